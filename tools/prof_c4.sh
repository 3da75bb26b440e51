set -x
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tools/stream_probe tools/stream_probe.cu
timeout 300 tools/stream_probe 2048 > gpurun_out/stream_probe_2g.jsonl 2>&1
SF=100 SEED=4 VARIANTS=fused timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"fused_rl_kernel" -s 2 -c 1 -o gpurun_out/full_fused_c4 python tools/profile_step.py > gpurun_out/full_fused_c4.log 2>&1
SF=100 SEED=4 VARIANTS=staged timeout 600 ncu --set full --clock-control none --import-source on \
    -k regex:"select_tile_kernel|compact_kernel|refine_sum" -s 3 -c 3 -o gpurun_out/full_staged_c4 python tools/profile_step.py > gpurun_out/full_staged_c4.log 2>&1
