#!/bin/bash
# Compare the one-pass kernels on C4 and C2: streamed residual planes (AR_RL_RESMODE=1,
# fused_rl_kernel) vs gathered residual sectors (default, fused_rg_kernel).
for wl in c4 c2; do
  for mode in 1 0; do
    AR_RL_RESMODE=$mode timeout 600 python bench.py --workload $wl --only --no-cpu --e2e-steps 0 --no-parity \
      --steps 500 --replays 3 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); print(json.dumps({'wl':'$wl','mode':$mode,'kernel':d['roofline']['kernel'],'ms':d['ms_per_step'],'frac':d['roofline']['frac'],'rep':d['ms_per_step_replays']}))"
  done
done
