#!/bin/bash
# C5 per-GPU share with the l_shipdate residual in pinned host memory: split layouts h = 0 (one SLICED
# part), 2, 3, 4 high planes stored apart.
for h in 0 2 3 4; do
  timeout 900 python bench.py --workload c5 --steps 6 --no-cpu --c5-split $h | tail -1 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); print(json.dumps({'split':$h,'kernel':d['kernel'],'ms':d['ms_per_step'],'link_frac':d['host_link']['frac'],'link':d['host_link']['peak'],'parity':d['parity']['match']}))"
done
