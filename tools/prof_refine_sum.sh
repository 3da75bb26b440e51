#!/bin/bash
# ncu --set full of the C4 staged refine + SUM kernels: the default (pipe) and AR_REF_PIPE=0 (sliced).
for v in 1 0; do
AR_REF_PIPE=$v SF=100 SEED=4 VARIANTS=staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"refine_sum" -s 1 -c 1 -o gpurun_out/prs_$v python tools/profile_step.py > gpurun_out/prs_$v.log 2>&1
python tools/ncu_summary.py gpurun_out/prs_$v.ncu-rep > gpurun_out/prs_$v.txt 2>&1
python -c "
import sys; sys.path.insert(0, 'tools')
import ncu_summary as n
n.hot_src('gpurun_out/prs_$v.ncu-rep', 'refine_sum', top=30)
" >> gpurun_out/prs_$v.txt 2>&1
done
