set -x
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 20 --warmup 3 --no-cpu --e2e-steps 0 > gpurun_out/bench_under_ncu.json 2>&1
VARIANTS=fused,staged timeout 900 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_kernel|select_tile_kernel|compact_kernel|refine_sum_kernel" -s 4 -c 4 -o gpurun_out/full python tools/profile_step.py \
    > gpurun_out/full.log 2>&1
timeout 300 python bench.py --impl reference --steps 5 --warmup 1 > gpurun_out/bench_ref.json 2> gpurun_out/bench_ref.err
