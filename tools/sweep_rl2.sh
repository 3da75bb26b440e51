#!/bin/bash
# one-pass kernel: (warps, blocks) x ring x CTAs with the PDL early-read workspace call
run() { echo "== $*"; env "${@:2}" timeout 120 python tools/rl_probe.py --reps 30 --srs $1; }
{
run pdl_early AR_RL_CFG=0
run pdl_early AR_RL_CFG=0 AR_RL_RING=128 AR_RL_CTAS=3
run pdl_early AR_RL_CFG=3 AR_RL_RING=64
run pdl_early AR_RL_CFG=5 AR_RL_RING=64
run pdl_early AR_RL_CFG=4 AR_RL_RING=64 AR_RL_CTAS=4
run pdl_early AR_RL_CFG=4 AR_RL_RING=64 AR_RL_CTAS=5
run pdl_early AR_RL_CFG=1 AR_RL_RING=64 AR_RL_CTAS=3
} > gpurun_out/sweep_rl6.txt 2>&1
