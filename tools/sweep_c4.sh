#!/bin/bash
# C4 one-pass kernel configuration sweep (consumer warps x blocks per thread, CTAs per SM, ring, stages).
run() {
  name=$1; shift
  env "$@" timeout 300 python bench.py --only --no-cpu --no-parity --e2e-steps 0 --latency-reps 0 --steps 200 \
      > gpurun_out/sw_$name.json 2> gpurun_out/sw_$name.err
  python - "$name" <<'PY'
import sys, json
n = sys.argv[1]
try:
    d = json.loads(open(f"gpurun_out/sw_{n}.json").read().strip().splitlines()[-1])
    print(json.dumps({"run": n, "ms": round(d["ms_per_step"], 4), "med": round(d["ms_per_step_replays"]["median"], 4),
                      "frac": round(d["roofline"]["frac"], 4)}))
except Exception as e:
    print(n, "failed", open(f"gpurun_out/sw_{n}.err").read()[-600:])
PY
}
run base
run cfg5 AR_RL_CFG=5
run cfg5r64 AR_RL_CFG=5 AR_RL_RING=64
run cfg1 AR_RL_CFG=1
run cfg3 AR_RL_CFG=3 AR_RL_RING=64
run cfg4c3 AR_RL_CFG=4 AR_RL_CTAS=3
run cfg4c4 AR_RL_CFG=4 AR_RL_CTAS=4 AR_RL_RING=64
run ctas3 AR_RL_CTAS=3 AR_RL_RING=64
run st3 AR_STAGES=3
run ring64 AR_RL_RING=64
run ring256 AR_RL_RING=256
run base2
