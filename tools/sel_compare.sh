#!/bin/bash
# The staged path's select at 1/2/3 tile buffers per persistent CTA (AR_SEL_BUFS), C4 and C2.
for wl in c4 c2; do
  for b in 1 2 3; do
    AR_SEL_BUFS=$b timeout 600 python bench.py --workload $wl --variant staged --only --no-cpu --e2e-steps 0 --no-parity \
      --steps 300 --replays 2 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); r=d['roofline']; print(json.dumps({'wl':'$wl','bufs':$b,'ms':d['ms_per_step'],'per_kernel':{k:(v['ms'],round(v['gbs']/6455.3,3)) for k,v in r['per_kernel'].items()},'step_frac':r['step_frac']}))"
  done
done
