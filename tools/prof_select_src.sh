#!/bin/bash
# Source-level ncu view of the staged select (C4): per CUDA line and per SASS block,
# instructions executed and stall samples.
SF=100 SEED=4 VARIANTS=staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"select_tile_kernel|compact_kernel|refine_sum" -s 3 -c 3 -o gpurun_out/pss_c4 python tools/profile_step.py \
    > gpurun_out/pss_c4.log 2>&1
python tools/ncu_summary.py gpurun_out/pss_c4.ncu-rep > gpurun_out/pss_c4.txt 2>&1
for k in select_tile refine_sum compact; do
python -c "
import sys; sys.path.insert(0, 'tools')
import ncu_summary as n
print('== $k by source line'); n.hot_src('gpurun_out/pss_c4.ncu-rep', '$k', top=40)
print('== $k by SASS block'); n.hot_blocks('gpurun_out/pss_c4.ncu-rep', '$k', top=25)
" >> gpurun_out/pss_c4.txt 2>&1
done
[ -n "$KEEP" ] || rm -f gpurun_out/pss_c4.ncu-rep
