#!/bin/bash
# ncu --set full of the one-kernel ordered select (select_rr_kernel) at C4, source-level summary.
SF=100 SEED=4 VARIANTS=staged AR_SEL_RR_BUFS=${BUFS:-1} timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"select_rr" -s 1 -c 1 -o gpurun_out/prr python tools/profile_step.py > gpurun_out/prr.log 2>&1
python tools/ncu_summary.py gpurun_out/prr.ncu-rep > gpurun_out/prr.txt 2>&1
python -c "
import sys; sys.path.insert(0, 'tools')
import ncu_summary as n
n.hot_src('gpurun_out/prr.ncu-rep', 'select_rr', top=40)
" >> gpurun_out/prr.txt 2>&1
