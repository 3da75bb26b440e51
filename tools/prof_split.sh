#!/bin/bash
# ncu --set full of the C4 one-pass kernel with the l_shipdate residual split ($1 high planes) and unsplit.
for h in "$@"; do
SF=100 SEED=4 SPLIT=$h VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel" -s 2 -c 1 -o gpurun_out/full_fused_c4_split$h python tools/profile_step.py \
    > gpurun_out/full_fused_c4_split$h.log 2>&1
done
