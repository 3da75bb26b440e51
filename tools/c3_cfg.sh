#!/bin/bash
# C3 (1 G rows) one-pass COUNT under the gathered-residual kernel's tile configurations.
for cfg in 0 1 3 4; do
  AR_RL_CFG=$cfg timeout 600 python tools/bench_configs.py c3 > gpurun_out/c3cfg_$cfg.jsonl 2>/dev/null
  python - $cfg <<'PY'
import json, sys
c = sys.argv[1]
for l in open(f"gpurun_out/c3cfg_{c}.jsonl"):
    d = json.loads(l)
    if d["selectivity"] in (0.0001, 0.01):
        print(json.dumps({"cfg": int(c), "M": d["major_bits"], "s": d["selectivity"], "fused_ms": round(d["fused_count_ms"], 4),
                          "frac": round(d["fused_count_frac"], 3)}))
PY
done
