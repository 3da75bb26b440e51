#!/bin/bash
# C4 one-pass kernel: producer / consumer mbarrier wait modes.
source tools/sweep_lib.sh
run base
run pw1 AR_PROD_WAIT=1
run pw2000 AR_PROD_WAIT=2000
run pw20000 AR_PROD_WAIT=20000
run sus1000 AR_SUSPEND_NS=1000
run pw1sus1000 AR_PROD_WAIT=1 AR_SUSPEND_NS=1000
run base2
