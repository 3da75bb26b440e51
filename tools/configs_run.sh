#!/bin/bash
# Secondary configurations (tools/bench_configs.py) in one GPU call
set -x
for c in mm c1 c5 c3; do
  timeout 900 python tools/bench_configs.py $c --reps 10 >> gpurun_out/configs.jsonl 2>> gpurun_out/configs.err
done
