"""Summarise an ncu launch list (`ncu --metrics gpu__time_duration.sum --csv`):
launches, mean and total time and share per kernel.

    python tools/launch_summary.py gpurun_out/launches.csv "python bench.py ..."
"""
import collections
import csv
import re
import sys


def main(path, cmd=""):
    rows = list(csv.reader(open(path)))
    hi = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
    h = rows[hi]
    ik, iv, im = h.index("Kernel Name"), h.index("Metric Value"), h.index("Metric Name")
    tot = collections.defaultdict(float)
    cnt = collections.Counter()
    for r in rows[hi + 1:]:
        if len(r) != len(h) or r[im] != "gpu__time_duration.sum":
            continue
        name = re.sub(r"<.*>", "<..>", r[ik].split("(")[0]).replace("void ", "")
        tot[name] += float(r[iv]) / 1e3
        cnt[name] += 1
    allt = sum(tot.values()) or 1.0
    print(f"# ncu launch list: {cmd}")
    print("# ncu --metrics gpu__time_duration.sum --clock-control none (cold-cache, serialised launches)")
    print(f"{'kernel':40s} {'launches':>9s} {'mean_us':>10s} {'total_us':>10s} {'share':>7s}")
    for k in sorted(tot, key=lambda k: -tot[k]):
        print(f"{k[:40]:40s} {cnt[k]:9d} {tot[k] / cnt[k]:10.2f} {tot[k]:10.1f} {tot[k] / allt * 100:6.1f}%")


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2] if len(sys.argv) > 2 else "")
