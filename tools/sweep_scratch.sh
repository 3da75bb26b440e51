#!/bin/bash
timeout 600 python -m pytest tests -m gpu -x -q > gpurun_out/gpu_tests.log 2>&1
timeout 300 python bench.py --steps 200 --no-cpu --e2e-steps 10 > gpurun_out/sw_all.json 2> gpurun_out/sw_all.err
