"""Print one line per bench JSON file: value, ms/step, per-kernel times, roofline fraction."""
import glob
import json
import sys

for f in sorted(sum([glob.glob(p) for p in sys.argv[1:]], [])):
    try:
        d = json.loads(open(f).read().strip().splitlines()[-1])
    except Exception as e:
        print(f, "ERR", e)
        continue
    r = d.get("roofline") or {}
    pk = {k: round(v["ms"] * 1e3, 1) for k, v in (r.get("per_kernel") or {}).items()}
    ok = (d.get("counts") or {}).get("gpu_sum")
    print(f"{f.split('/')[-1]:28s} {d['value']:.3e} rows/s  {d['ms_per_step']*1e3:7.1f} us/step  "
          f"frac {r.get('frac', 0):.3f} step_frac {r.get('step_frac', 0):.3f}  {pk}  sum={ok}")
