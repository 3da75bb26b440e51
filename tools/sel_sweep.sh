#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x -k "select or refine or minmax or spatial or q6 or c1 or fullsize" > gpurun_out/gpu_tests.log 2>&1
for cfg in "AR_SELECT_TILE=1" "AR_SELECT_TILE=0"; do
  env $cfg timeout 300 python tools/time_staged.py >> gpurun_out/sel_sweep.jsonl 2>> gpurun_out/sel_sweep.err
done
timeout 600 python tools/bench_configs.py c3 --widths 8 24 --sels 0.01 0.5 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
