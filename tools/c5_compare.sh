#!/bin/bash
# C5 per-GPU share (750 M rows, l_shipdate residual in pinned host memory): general one-pass kernel
# vs the gathered-residual kernel with / without the .L2::64B hint on host reads.
run() { env "$@" timeout 900 python bench.py --workload c5 --steps 6 --no-cpu | tail -1 | python -c "import sys,json; d=json.loads(sys.stdin.readline()); print(json.dumps({'env':'$*','kernel':d['kernel'],'ms':d['ms_per_step'],'link_frac':d['host_link']['frac'],'link':d['host_link']['peak'],'parity':d['parity']['match']}))"; }
run AR_FUSED_LEGACY=1
run AR_HOST_HINT=1
run AR_HOST_HINT=0
