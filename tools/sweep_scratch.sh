#!/bin/bash
timeout 200 python bench.py --steps 200 --no-cpu --e2e-steps 0 --only > gpurun_out/sw_fused.json 2> gpurun_out/sw_fused.err
