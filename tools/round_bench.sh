#!/bin/bash
# Round measurement on one B200: GPU tests, smoke, the default bench line, the
# reference (oracle) arm, the ncu launch list of the same bench command (cold,
# serialised: compare shares), one full ncu capture of each hot kernel, and the
# secondary configurations.  Outputs land in gpurun_out/; summaries are copied
# to profiles/ by hand.
set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,clocks.mem,power.draw --format=csv > gpurun_out/smi.txt
timeout 900 python -m pytest tests -m gpu -q > gpurun_out/gpu_tests.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1
timeout 600 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err
timeout 300 python bench.py --impl reference --steps 5 --warmup 3 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 20 --warmup 3 --no-cpu --e2e-steps 0 > gpurun_out/bench_under_ncu.json 2>&1
VARIANTS=fused,staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel|select_tile_kernel|compact_kernel|refine_sum" -s 3 -c 4 -o gpurun_out/full python tools/profile_step.py \
    > gpurun_out/full.log 2>&1
for c in mm grp c1 c5 c3; do
  timeout 900 python tools/bench_configs.py $c --reps 10 >> gpurun_out/configs.jsonl 2>> gpurun_out/configs.err
done
