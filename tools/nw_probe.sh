#!/bin/bash
timeout 900 python -m pytest tests -m gpu -q -x -k "select or q6 or refine or c1 or fullsize" > gpurun_out/t.log 2>&1
timeout 300 python tools/time_staged.py > gpurun_out/ts.jsonl 2>&1
timeout 600 python tools/bench_configs.py c3 --widths 8 16 24 --sels 0.01 0.5 --reps 5 > gpurun_out/c3.jsonl 2> gpurun_out/c3.err
