"""Probe of the one-pass kernel on the C2 workload (SF10 Q6, 60 M rows): time
ar_select_refine_sum per SUM-factor mode with the L2 flushed before every call.

    AR_RL_CFG=0 python tools/rl_probe.py [--reps R]

Modes: count (no factors: the scan alone, majors + streamed residual),
disc (one predicate-column factor, no gathers), q6 (l_extendedprice gathered
x l_discount).  One JSON line per mode.
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))

import torch  # noqa: E402

import datagen  # noqa: E402
from bench_configs import timed, PEAK  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--reps", type=int, default=30)
    ap.add_argument("--sf", type=float, default=10.0)
    args = ap.parse_args()
    c = datagen.q6_columns(2, args.sf)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    flush = torch.empty(512 * 1024 * 1024, dtype=torch.uint8, device="cuda")
    out = torch.zeros(4, dtype=torch.int64, device="cuda")
    scan_bytes = n * (4 + 4 + 6 + 8) / 8
    for mode, aggs in (("count", []), ("disc", [dc]), ("q6", [ep, dc])):
        ms, mn = timed(lambda: cu.select_refine_sum(preds, aggs, out), args.reps, flush)
        print(json.dumps({"mode": mode, "kernel": _ar.ar_last_scan_kernel(), "cfg": os.environ.get("AR_RL_CFG"),
                          "us_mean": ms * 1e3, "us_min": mn * 1e3,
                          "scan_stream_gbs": scan_bytes / (mn / 1e3) / 1e9, "peak": PEAK,
                          "out": out.tolist()}), flush=True)


if __name__ == "__main__":
    main()
