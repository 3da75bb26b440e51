#!/bin/bash
# Copy the round measurement (gpurun_out/, written by tools/round_bench.sh on the box) to profiles/$1 and
# install the traffic.json computed there.
R=${1:-r02}
mkdir -p profiles/$R
cp gpurun_out/bench.json profiles/$R/bench_line.json
cp gpurun_out/bench_ref.json profiles/$R/bench_reference_arm.json
cp gpurun_out/smi.txt profiles/$R/smi.txt
tail -3 gpurun_out/gpu_tests.log > profiles/$R/gpu_tests_tail.txt
cat gpurun_out/smoke.log > profiles/$R/smoke.txt
cp gpurun_out/launches.csv profiles/$R/launches.csv
cp gpurun_out/round/launches_summary.txt profiles/$R/launches_summary.txt
for rep in full_fused_c4 full_staged_c4 full_c2 full_refine_c4; do
  cp gpurun_out/round/ncu_$rep.txt profiles/$R/ncu_$rep.txt
done
cp gpurun_out/round/traffic.json profiles/traffic.json
