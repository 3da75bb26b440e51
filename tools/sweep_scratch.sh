#!/bin/bash
for c in 0 2 3; do
AR_CTAS=$c timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --only > gpurun_out/sw_fused_c$c.json 2> gpurun_out/sw_fused.err
done
