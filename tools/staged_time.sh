#!/bin/bash
# The staged path (ar_approx_select -> ar_refine_sum) on C4 and C2: per-kernel times and fractions.
for wl in c4 c2; do
  timeout 600 python bench.py --workload $wl --variant staged --only --no-cpu --e2e-steps 0 --no-parity \
      --steps 300 --replays 2 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); r=d['roofline']; print(json.dumps({'wl':'$wl','ms':d['ms_per_step'],'per_kernel':{k:(v['ms'],round(v['gbs']/6455.3,3)) for k,v in r['per_kernel'].items()},'step_frac':r['step_frac']}))"
done
