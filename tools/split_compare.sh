#!/bin/bash
# C4 (and C2) headline with the l_shipdate residual split h = 0 (one part), 2, 3, 4: the one-pass kernel
# streams the h high planes and gathers the low planes of the rows they leave undecided (DESIGN s6.3d).
for h in 0 4 3 2; do
  timeout 900 python bench.py --only --no-cpu --e2e-steps 0 --latency-reps 0 --split $h --steps 200 \
    > gpurun_out/split_$h.json 2> gpurun_out/split_$h.err
  python - "$h" <<'PY'
import sys, json
h = sys.argv[1]
try:
    d = json.loads(open(f"gpurun_out/split_{h}.json").read().strip().splitlines()[-1])
    r = d["roofline"]
    print(json.dumps({"split": int(h), "ms": d["ms_per_step"], "rows_per_s": d["value"], "frac": r["frac"],
                      "alg_bytes": r["algorithmic_bytes_per_launch"], "kernel": d["gpu_kernels"],
                      "replays": d["ms_per_step_replays"], "parity": (d.get("parity") or {}).get("match"),
                      "clocks": d["clocks"]["sm_mhz"]}))
except Exception as e:
    print("split", h, "failed", e, open(f"gpurun_out/split_{h}.err").read()[-2000:])
PY
done
