#!/bin/bash
# One ncu --set full capture of the C4 one-pass kernel ($1 = split h, default 0) and its hot-block summary.
h=${1:-0}
SF=100 SEED=4 SPLIT=$h VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel|fused_rg_kernel" -s 2 -c 1 -o gpurun_out/pf_c4_$h python tools/profile_step.py \
    > gpurun_out/pf_c4_$h.log 2>&1
python tools/ncu_summary.py gpurun_out/pf_c4_$h.ncu-rep > gpurun_out/pf_c4_$h.txt 2>&1
python -c "
import sys; sys.path.insert(0, 'tools')
import ncu_summary as n
n.hot_blocks('gpurun_out/pf_c4_$h.ncu-rep', 'fused_r', top=40)
" >> gpurun_out/pf_c4_$h.txt 2>&1
