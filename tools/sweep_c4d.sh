#!/bin/bash
# C4 one-pass kernel: more resident consumer warps per SM at 3 stages (4-warp CTAs, smaller rings).
source tools/sweep_lib.sh
run base
run cfg4c5st3r64 AR_RL_CFG=4 AR_RL_CTAS=5 AR_STAGES=3 AR_RL_RING=64
run cfg4c4st3r64 AR_RL_CFG=4 AR_RL_CTAS=4 AR_STAGES=3 AR_RL_RING=64
run cfg4c4st3 AR_RL_CFG=4 AR_RL_CTAS=4 AR_STAGES=3
run r64 AR_RL_RING=64
BARGS="--workload c2" run c2base
BARGS="--workload c2" run c2cfg4c5 AR_RL_CFG=4 AR_RL_CTAS=5 AR_STAGES=3 AR_RL_RING=64
BARGS="--workload c2" run c2cfg4c4 AR_RL_CFG=4 AR_RL_CTAS=4 AR_STAGES=3
run base2
