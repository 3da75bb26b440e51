#!/bin/bash
# Result-ring fused kernel: its GPU tests, the headline bench line per (NW, BPT) config, one ncu capture.
timeout 600 python -m pytest tests/test_gpu_fused_rl.py -x -q > gpurun_out/gpu_tests_rl.log 2>&1
for c in ${CFGS:-0 3}; do
  AR_RL_CFG=$c timeout 200 python bench.py --steps 300 --only --no-cpu --e2e-steps 0 > gpurun_out/rl_cfg$c.json 2> gpurun_out/rl_cfg$c.err
done
VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on -k regex:fused_rl_kernel -s 2 -c 1 \
   -o gpurun_out/rl python tools/profile_step.py > gpurun_out/rl_prof.log 2>&1
