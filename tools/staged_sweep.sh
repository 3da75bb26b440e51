#!/bin/bash
# C4 staged step under select knobs.
run() { name=$1; shift; env "$@" RUNS=$name bash tools/staged_c4.sh; }
run base
run bpt4 AR_SEL_BPT=4
run bufs2 AR_SEL_BUFS=2
run base2
