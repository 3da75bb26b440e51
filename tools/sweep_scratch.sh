#!/bin/bash
timeout 600 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
for c in 0 3; do
AR_CTAS=$c timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --only > gpurun_out/sw_fused_c$c.json 2> gpurun_out/sw_fused.err
done
VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on -k regex:"fused_kernel" -s 2 -c 1 -o gpurun_out/prof20 python tools/profile_step.py > gpurun_out/prof20.log 2>&1
