#!/bin/bash
timeout 300 python bench.py --steps 300 --no-cpu --e2e-steps 0 > gpurun_out/bench_sel.json 2> gpurun_out/bench_sel.err
./tools/stream_probe 180 > gpurun_out/stream_probe180.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "refine or q6 or sum" > gpurun_out/gpu_tests_parity.log 2>&1
