#!/bin/bash
set -x
for cfg in "AR_REFINE_GENERIC=0"; do
  env $cfg timeout 300 python tools/time_staged.py >> gpurun_out/sel_sweep.jsonl 2>> gpurun_out/sel_sweep.err
done
timeout 900 python -m pytest tests -m gpu -q -x -k "refine or q6 or c2 or fullsize" > gpurun_out/gpu_tests.log 2>&1
