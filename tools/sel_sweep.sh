#!/bin/bash
set -x
for cfg in "AR_SEL_BPT=2" "AR_SEL_BPT=4"; do
  env $cfg timeout 300 python tools/time_staged.py >> gpurun_out/sel_sweep.jsonl 2>> gpurun_out/sel_sweep.err
done
AR_SEL_BPT=4 timeout 900 python -m pytest tests -m gpu -q -x -k "select or refine or q6 or c1 or fullsize or c2" > gpurun_out/gpu_tests.log 2>&1
