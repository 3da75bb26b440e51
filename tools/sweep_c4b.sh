#!/bin/bash
# C4 one-pass kernel: pipeline depth sweep (stages x CTAs per SM x tile size), unsplit and split residuals.
run() {
  name=$1; shift
  env "$@" timeout 300 python bench.py --only --no-cpu --no-parity --e2e-steps 0 --latency-reps 0 --steps 200 $BARGS \
      > gpurun_out/sw_$name.json 2> gpurun_out/sw_$name.err
  python - "$name" <<'PY'
import sys, json
n = sys.argv[1]
try:
    d = json.loads(open(f"gpurun_out/sw_{n}.json").read().strip().splitlines()[-1])
    print(json.dumps({"run": n, "ms": round(d["ms_per_step"], 4), "med": round(d["ms_per_step_replays"]["median"], 4),
                      "min": round(d["ms_per_step_replays"]["min"], 4), "frac": round(d["roofline"]["frac"], 4)}))
except Exception as e:
    print(n, "failed", open(f"gpurun_out/sw_{n}.err").read()[-600:])
PY
}
run base
run st3 AR_STAGES=3
run st2 AR_STAGES=2
run st4 AR_STAGES=4
run c3st2 AR_RL_CTAS=3 AR_STAGES=2
run cfg4c4st3 AR_RL_CFG=4 AR_RL_CTAS=4 AR_STAGES=3
run cfg4c4st2 AR_RL_CFG=4 AR_RL_CTAS=4 AR_STAGES=2
run cfg4c5st2 AR_RL_CFG=4 AR_RL_CTAS=5 AR_STAGES=2
run cfg3st2 AR_RL_CFG=3 AR_STAGES=2
run st3b AR_STAGES=3
BARGS="--split 4" run sp4 AR_STAGES=4
BARGS="--split 4" run sp4st3 AR_STAGES=3
BARGS="--split 4" run sp4st2 AR_STAGES=2
BARGS="--workload c2" run c2base
BARGS="--workload c2" run c2st3 AR_STAGES=3
BARGS="--workload c2" run c2st2 AR_STAGES=2
