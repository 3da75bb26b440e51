#!/bin/bash
# ncu --set full of the C4 staged kernels (select tile + compaction + refine+SUM) and their summaries.
SF=100 SEED=4 VARIANTS=staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"select_tile_kernel|compact_kernel|refine_sum" -s 3 -c 3 -o gpurun_out/ps_c4 python tools/profile_step.py \
    > gpurun_out/ps_c4.log 2>&1
python tools/ncu_summary.py gpurun_out/ps_c4.ncu-rep > gpurun_out/ps_c4.txt 2>&1
python -c "
import sys; sys.path.insert(0, 'tools')
import ncu_summary as n
n.hot_blocks('gpurun_out/ps_c4.ncu-rep', 'select_tile', top=25)
" >> gpurun_out/ps_c4.txt 2>&1
[ -n "$KEEP" ] || rm -f gpurun_out/ps_c4.ncu-rep
