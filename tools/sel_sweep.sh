#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x -k "refine or select or minmax or spatial" > gpurun_out/gpu_tests.log 2>&1
timeout 600 python tools/bench_configs.py c3 --widths 8 24 --sels 0.01 0.5 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
