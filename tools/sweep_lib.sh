# run NAME [ENV=V ...]: one headline bench line (no parity / cpu / e2e / latency), summarised as JSON
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
