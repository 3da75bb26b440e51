#!/bin/bash
# Iteration check on one B200: GPU tests, the default bench line, one full ncu
# capture per hot kernel (select_rl + compact of the staged path, the fused kernel).
set -x
timeout 900 python -m pytest tests -m gpu -q -x > gpurun_out/gpu_tests.log 2>&1
timeout 600 python bench.py --no-cpu > gpurun_out/bench.json 2> gpurun_out/bench.err
VARIANTS=staged timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"select_rl_kernel|select_tile_kernel|compact_kernel|refine_sum_kernel" -s 3 -c 3 -o gpurun_out/full_staged python tools/profile_step.py \
    > gpurun_out/full_staged.log 2>&1
VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel" -s 2 -c 1 -o gpurun_out/full_fused python tools/profile_step.py \
    > gpurun_out/full_fused.log 2>&1
