#!/bin/bash
set -x
timeout 900 python -m pytest tests -m gpu -q -x -k "segmented or q6 or refine or select" > gpurun_out/gpu_tests.log 2>&1
timeout 300 python tools/time_staged.py >> gpurun_out/ts.jsonl 2>> gpurun_out/ts.err
timeout 300 python tools/time_staged.py --segmented >> gpurun_out/ts.jsonl 2>> gpurun_out/ts.err
