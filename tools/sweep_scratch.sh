#!/bin/bash
timeout 600 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --variant staged --only > gpurun_out/sw_staged.json 2> gpurun_out/sw_staged.err
VARIANTS=staged timeout 600 ncu --set full --clock-control none --import-source on -k regex:"select_tile_kernel|compact" -s 2 -c 2 -o gpurun_out/prof18 python tools/profile_step.py > gpurun_out/prof18.log 2>&1
