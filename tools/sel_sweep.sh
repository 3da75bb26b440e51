#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x -k "refine or q6 or c1 or fullsize or minmax or group or spatial or segmented" > gpurun_out/gpu_tests.log 2>&1
timeout 300 python tools/profile_refine.py > gpurun_out/pr.log 2>&1
S=0.01 timeout 300 python tools/profile_refine.py >> gpurun_out/pr.log 2>&1
M=8 timeout 300 python tools/profile_refine.py >> gpurun_out/pr.log 2>&1
timeout 600 python tools/bench_configs.py c3 --widths 8 24 --sels 0.01 0.5 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
