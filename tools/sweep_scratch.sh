#!/bin/bash
timeout 400 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --variant fused > gpurun_out/sw_fused.json 2> gpurun_out/sw_fused.err
timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 > gpurun_out/sw_staged.json 2> gpurun_out/sw_staged.err
VARIANTS=fused,staged timeout 600 ncu --set full --clock-control none --import-source on -k regex:"fused_kernel|select_kernel" -s 2 -c 2 -o gpurun_out/prof11 python tools/profile_step.py > gpurun_out/prof11.log 2>&1
