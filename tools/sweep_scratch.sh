#!/bin/bash
timeout 600 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 10 > gpurun_out/sw_fused.json 2> gpurun_out/sw_fused.err
VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on -k regex:"fused_kernel" -s 2 -c 1 -o gpurun_out/prof22 python tools/profile_step.py > gpurun_out/prof22.log 2>&1
