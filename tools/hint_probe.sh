#!/bin/bash
# Gather prefetch-size hint probe: library with .L2::64B (A) vs without (B) on the host-link
# bound paths (C5 per-GPU share, e2e of bench.py) and the HBM headline.
set -x
run() {
  timeout 600 python tools/bench_configs.py c5 --reps 5 > gpurun_out/c5_$1.jsonl 2> gpurun_out/c5_$1.err
  timeout 300 python bench.py --only --steps 300 --no-cpu --e2e-steps 10 > gpurun_out/bench_$1.json 2> gpurun_out/bench_$1.err
}
run A
cp probe_b/libar_b200.so paper_conf_icde_pirkmk14_b200/libar_b200.so
run B
