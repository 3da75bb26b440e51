#!/bin/bash
timeout 400 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
for c in 0 2 3; do
AR_CTAS=$c timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --variant fused > gpurun_out/sw_fused_c$c.json 2> gpurun_out/sw_fused_c$c.err
done
VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on -k regex:"fused_kernel" -s 2 -c 1 -o gpurun_out/prof13 python tools/profile_step.py > gpurun_out/prof13.log 2>&1
