#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x -k "select or refine or q6 or c1 or fullsize or minmax or group or spatial" > gpurun_out/gpu_tests.log 2>&1
for cfg in "AR_SELECT_RING=0" "AR_SELECT_RING=1"; do
  env $cfg timeout 300 python tools/time_staged.py >> gpurun_out/ts.jsonl 2>> gpurun_out/ts.err
  env $cfg timeout 600 python tools/bench_configs.py c3 --widths 8 16 24 --sels 0.01 0.5 --reps 5 >> gpurun_out/c3.jsonl 2>> gpurun_out/c3.err
done
