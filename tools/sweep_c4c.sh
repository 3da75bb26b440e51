#!/bin/bash
# C4 / C2 one-pass kernel: gather depth (AR_RL_DEPTH 4 / 8) at the 3-stage default.
source tools/sweep_lib.sh
run base
run d8 AR_RL_DEPTH=8
run d8r256 AR_RL_DEPTH=8 AR_RL_RING=256
run st4 AR_STAGES=4
BARGS="--split 4" run sp4
BARGS="--split 4" run sp4d8 AR_RL_DEPTH=8
BARGS="--workload c2" run c2base
BARGS="--workload c2" run c2d8 AR_RL_DEPTH=8
run base2
