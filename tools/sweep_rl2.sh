#!/bin/bash
# one-pass kernel knob sweep on C2 (rl_probe: count / disc / q6 modes)
run() { echo "== $*"; env "$@" timeout 120 python tools/rl_probe.py --reps 20; }
{
run AR_RL_CFG=0
run AR_RL_CFG=0 AR_RL_RING=64
run AR_RL_CFG=0 AR_RL_RING=64 AR_RL_CTAS=3
run AR_RL_CFG=0 AR_RL_RING=64 AR_STAGES=4
run AR_RL_CFG=4 AR_RL_RING=64 AR_RL_CTAS=4
run AR_RL_CFG=4 AR_RL_RING=64 AR_RL_CTAS=5
run AR_RL_CFG=1 AR_RL_RING=64 AR_RL_CTAS=3
run AR_RL_CFG=3 AR_RL_RING=64
run AR_FUSED_LEGACY=1
} > gpurun_out/sweep_rl2.txt 2>&1
