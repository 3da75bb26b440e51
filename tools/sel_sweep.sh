#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x > gpurun_out/gpu_tests.log 2>&1
timeout 600 python tools/bench_configs.py c3 --widths 16 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
timeout 300 python tools/time_staged.py >> gpurun_out/ts.jsonl 2>> gpurun_out/ts.err
