"""Write profiles/traffic.json from `ncu --set full` captures of the bench's kernels.

    python tools/ncu_traffic.py <workload> <report.ncu-rep> [<report.ncu-rep> ...]

For every kernel in the reports: dram__bytes_read.sum + dram__bytes_write.sum per
launch (averaged over the captured launches), keyed the way bench.py names its
roofline kernels ("fused_rl_kernel", "select_tile_kernel+compact_kernel" = the
sum of the two launches of ar_approx_select, "refine_sum_sliced_kernel", ...),
with the git commit and report names it was taken from.  bench.py copies the
entry of the kernel it reports into roofline.traffic.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def kernels(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv", "--metrics",
                          "dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum"],
                         capture_output=True, text=True, check=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units = rows[0], rows[1]
    name_i = hdr.index("Kernel Name")
    res = []
    for r in rows[2:]:
        if len(r) != len(hdr):
            continue
        d = {"name": r[name_i]}
        for m in ("dram__bytes_read.sum", "dram__bytes_write.sum", "gpu__time_duration.sum"):
            i = hdr.index(m)
            v = float(r[i].replace(",", ""))
            u = units[i]
            scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "ns": 1e-3, "us": 1, "ms": 1e3}.get(u, 1)
            d[m] = v * scale
        res.append(d)
    return res


def short(name):
    base = name.split("(")[0].split("<")[0].strip()
    return base.replace("void ", "").split("::")[-1]


def main():
    wl, reps = sys.argv[1], sys.argv[2:]
    # the GPU box has no .git: the caller passes the commit in COMMIT
    commit = os.environ.get("COMMIT") or subprocess.run(["git", "rev-parse", "--short", "HEAD"], cwd=ROOT,
                                                        capture_output=True, text=True).stdout.strip()
    acc = {}
    for rep in reps:
        for k in kernels(rep):
            s = short(k["name"])
            a = acc.setdefault(s, {"bytes": 0.0, "read": 0.0, "write": 0.0, "us": 0.0, "n": 0})
            a["bytes"] += k["dram__bytes_read.sum"] + k["dram__bytes_write.sum"]
            a["read"] += k["dram__bytes_read.sum"]
            a["write"] += k["dram__bytes_write.sum"]
            a["us"] += k["gpu__time_duration.sum"]
            a["n"] += 1
    src = f"ncu --set full, commit {commit}, {', '.join(os.path.basename(r) for r in reps)}"
    entry = {}
    for s, a in acc.items():
        entry[s] = {"bytes_per_launch": a["bytes"] / a["n"], "read_per_launch": a["read"] / a["n"],
                    "write_per_launch": a["write"] / a["n"], "us_per_launch_cold": a["us"] / a["n"],
                    "launches": a["n"], "source": src}
    if "select_tile_kernel" in entry and "compact_kernel" in entry:
        e1, e2 = entry["select_tile_kernel"], entry["compact_kernel"]
        entry["select_tile_kernel+compact_kernel"] = {
            "bytes_per_launch": e1["bytes_per_launch"] + e2["bytes_per_launch"],
            "read_per_launch": e1["read_per_launch"] + e2["read_per_launch"],
            "write_per_launch": e1["write_per_launch"] + e2["write_per_launch"],
            "us_per_launch_cold": e1["us_per_launch_cold"] + e2["us_per_launch_cold"], "source": src}
    path = os.environ.get("TRAFFIC_JSON") or os.path.join(ROOT, "profiles", "traffic.json")
    allt = {}
    if os.path.exists(path):
        try:
            allt = json.load(open(path))
        except Exception:
            allt = {}
    allt = {k: v for k, v in allt.items() if isinstance(v, dict) and k in ("c2", "c4", "c5")}
    allt.setdefault(wl, {}).update(entry)
    json.dump(allt, open(path, "w"), indent=1, sort_keys=True)
    print(json.dumps({wl: entry}, indent=1))


if __name__ == "__main__":
    main()
