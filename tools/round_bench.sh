#!/bin/bash
# Round measurement on one B200: GPU tests, smoke, the default bench line, the reference (oracle)
# arm, the ncu launch list of the bench command (cold, serialised: compare shares), full ncu captures
# of the hot kernels at C4 (the headline) and C2, and the traffic.json they give.  Outputs land in
# gpurun_out/; summaries are copied to profiles/rNN/ (tools/collect_round.sh).
set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,clocks.mem,power.draw,power.limit,enforced.power.limit --format=csv > gpurun_out/smi.txt
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_tests.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke.log 2>&1
timeout 900 python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err
timeout 300 python bench.py --impl reference --steps 5 --warmup 3 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 20 --warmup 3 --no-cpu --e2e-steps 0 --no-c5 --latency-reps 3 --replays 0 \
    > gpurun_out/bench_under_ncu.json 2>&1
SF=100 SEED=4 VARIANTS=fused timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel|fused_rg_kernel" -s 2 -c 1 -o gpurun_out/full_fused_c4 python tools/profile_step.py \
    > gpurun_out/full_fused_c4.log 2>&1
SF=100 SEED=4 VARIANTS=staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"select_rr_kernel|select_tile_kernel|compact_kernel|refine_sum" -s 2 -c 2 -o gpurun_out/full_staged_c4 python tools/profile_step.py \
    > gpurun_out/full_staged_c4.log 2>&1
SF=100 SEED=4 VARIANTS=refine timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"refine_kernel" -s 1 -c 1 -o gpurun_out/full_refine_c4 python tools/profile_step.py \
    > gpurun_out/full_refine_c4.log 2>&1
SF=10 SEED=2 VARIANTS=fused,staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel|select_rr_kernel|select_tile_kernel|compact_kernel|refine_sum" -s 3 -c 3 -o gpurun_out/full_c2 python tools/profile_step.py \
    > gpurun_out/full_c2.log 2>&1
# summaries on the box (gpurun merges at most 64 MiB of gpurun_out/ back): ncu summaries, the launch-list
# summary and traffic.json (bench.py reads profiles/traffic.json; tools/collect_round.sh installs it);
# only the C4 fused report is kept
mkdir -p gpurun_out/round
for rep in full_fused_c4 full_staged_c4 full_c2 full_refine_c4; do
  python tools/ncu_summary.py gpurun_out/$rep.ncu-rep > gpurun_out/round/ncu_$rep.txt 2>&1
done
cp profiles/traffic.json gpurun_out/round/traffic.json 2>/dev/null
TRAFFIC_JSON=gpurun_out/round/traffic.json python tools/ncu_traffic.py c4 gpurun_out/full_fused_c4.ncu-rep gpurun_out/full_staged_c4.ncu-rep > /dev/null
TRAFFIC_JSON=gpurun_out/round/traffic.json python tools/ncu_traffic.py c2 gpurun_out/full_c2.ncu-rep > /dev/null
python tools/launch_summary.py gpurun_out/launches.csv "python bench.py --steps 20 --warmup 3 --no-cpu --e2e-steps 0 --no-c5 --latency-reps 3 --replays 0" > gpurun_out/round/launches_summary.txt 2>&1
rm -f gpurun_out/full_staged_c4.ncu-rep gpurun_out/full_c2.ncu-rep gpurun_out/full_refine_c4.ncu-rep
