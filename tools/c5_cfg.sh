#!/bin/bash
# C5 per-GPU share (split h = 4 host residual, fused_rg_kernel) under tile / CTA configurations.
run() {
  name=$1; shift
  env "$@" timeout 900 python bench.py --workload c5 --steps 6 --no-cpu --no-parity 2>/dev/null | tail -1 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); print(json.dumps({'run':'$name','ms':round(d['ms_per_step'],3),'link_frac':round(d['host_link']['frac'],3)}))"
}
run base
run cfg4c3 AR_RL_CFG=4 AR_RL_CTAS=3
run cfg4c4 AR_RL_CFG=4 AR_RL_CTAS=4
run cfg3 AR_RL_CFG=3
run cfg1 AR_RL_CFG=1
run st4 AR_STAGES=4
