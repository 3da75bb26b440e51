#!/bin/bash
# Copy the round measurement's summaries from gpurun_out/ to profiles/$1 and refresh traffic.json.
R=${1:-r02}
mkdir -p profiles/$R
cp gpurun_out/bench.json profiles/$R/bench_line.json
cp gpurun_out/bench_ref.json profiles/$R/bench_reference_arm.json
cp gpurun_out/smi.txt profiles/$R/smi.txt
tail -3 gpurun_out/gpu_tests.log > profiles/$R/gpu_tests_tail.txt
cat gpurun_out/smoke.log > profiles/$R/smoke.txt
python tools/launch_summary.py gpurun_out/launches.csv "python bench.py --steps 20 --warmup 3 --no-cpu --e2e-steps 0 --no-c5 --latency-reps 3 --replays 0" > profiles/$R/launches_summary.txt
cp gpurun_out/launches.csv profiles/$R/launches.csv
for rep in full_fused_c4 full_staged_c4 full_c2; do
  python tools/ncu_summary.py gpurun_out/$rep.ncu-rep > profiles/$R/ncu_$rep.txt
done
python tools/ncu_traffic.py c4 gpurun_out/full_fused_c4.ncu-rep gpurun_out/full_staged_c4.ncu-rep > /dev/null
python tools/ncu_traffic.py c2 gpurun_out/full_c2.ncu-rep > /dev/null
