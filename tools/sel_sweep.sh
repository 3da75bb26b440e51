#!/bin/bash
set -x
timeout 300 python tools/time_staged.py >> gpurun_out/sel_sweep.jsonl 2>> gpurun_out/sel_sweep.err
timeout 600 python tools/bench_configs.py c3 --widths 8 24 --sels 0.01 0.5 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
timeout 900 python -m pytest tests -m gpu -q -x -k "select or refine or q6 or c1 or fullsize or minmax" > gpurun_out/gpu_tests.log 2>&1
