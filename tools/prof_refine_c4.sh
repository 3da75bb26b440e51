#!/bin/bash
# ncu --set full of the ordered refine (ar_refine, positions out) at C4 and its summary.
SF=100 SEED=4 VARIANTS=refine timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"refine_kernel" -s 1 -c 1 -o gpurun_out/prf_c4 python tools/profile_step.py > gpurun_out/prf_c4.log 2>&1
python tools/ncu_summary.py gpurun_out/prf_c4.ncu-rep > gpurun_out/prf_c4.txt 2>&1
