#!/bin/bash
# C4 staged step (ar_approx_select -> ar_refine_sum): step time, per-kernel times and fractions.
for v in ${RUNS:-a b}; do
  timeout 300 python bench.py --only --variant staged --no-cpu --no-parity --e2e-steps 0 --latency-reps 0 --steps 100 \
      > gpurun_out/st_$v.json 2> gpurun_out/st_$v.err
  python - "$v" <<'PY'
import sys, json
v = sys.argv[1]
try:
    d = json.loads(open(f"gpurun_out/st_{v}.json").read().strip().splitlines()[-1])
    r = d["roofline"]
    print(json.dumps({"run": v, "ms": round(d["ms_per_step"], 4), "step_frac": round(r["step_frac"], 4),
                      "kernels": {k: [round(x["ms"], 4), round(x["gbs"] / r["peak"], 3)] for k, x in r["per_kernel"].items()}}))
except Exception as e:
    print(v, "failed", e, open(f"gpurun_out/st_{v}.err").read()[-800:])
PY
done
