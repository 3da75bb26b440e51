#!/bin/bash
set -x
for cfg in "AR_SEL_TPC=1" "AR_SEL_TPC=2"; do
  env $cfg timeout 300 python tools/time_staged.py >> gpurun_out/sel_sweep.jsonl 2>> gpurun_out/sel_sweep.err
  env $cfg timeout 600 python tools/bench_configs.py c3 --widths 8 16 24 --sels 0.01 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
done
AR_SEL_TPC=2 timeout 900 python -m pytest tests -m gpu -q -x -k "select or refine or q6 or c1 or fullsize or minmax" > gpurun_out/gpu_tests.log 2>&1
