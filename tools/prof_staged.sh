#!/bin/bash
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
VARIANTS=staged timeout 600 ncu --set full --clock-control none --import-source on -k regex:"refine_sum_kernel" -s 2 -c 1 -o gpurun_out/staged2 python tools/profile_step.py > gpurun_out/staged2.log 2>&1
