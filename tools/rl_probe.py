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
from bench_configs import PEAK  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--reps", type=int, default=30)
    ap.add_argument("--sf", type=float, default=10.0)
    ap.add_argument("--srs", choices=["plain", "ws", "pdl", "pdl_early"], default="plain",
                    help="ar_select_refine_sum (memset + kernel) or the _ws call without / with PDL")
    args = ap.parse_args()
    c = datagen.q6_columns(2, args.sf)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    # inputs rotated over 3 copies (3 x 345 MB > L2) instead of a flush: a flush leaves dirty
    # lines in L2 whose write-back would be charged to the timed kernel
    sets = [(sd, dc, qt, ep)] + [tuple(x.copy() for x in (sd, dc, qt, ep)) for _ in range(2)]
    out = torch.zeros(4, dtype=torch.int64, device="cuda")
    scan_bytes = n * (4 + 4 + 6 + 8) / 8
    it = [0]
    ws = cu.SrsWorkspace()
    flags = {"plain": 0, "ws": 0, "pdl": _ar.AR_SRS_PDL, "pdl_early": _ar.AR_SRS_PDL_EARLY_READ}[args.srs]

    def call(mode):
        a, b, c_, e = sets[it[0] % 3]
        it[0] += 1
        preds = [(a, *datagen.Q6_SHIPDATE), (b, *datagen.Q6_DISCOUNT), (c_, *datagen.Q6_QUANTITY)]
        aggs = {"count": [], "disc": [b], "q6": [e, b]}[mode]
        if args.srs == "plain":
            cu.select_refine_sum(preds, aggs, out)
        else:
            cu.select_refine_sum(preds, aggs, out, ws=ws, flags=flags)
    def timed(fn, reps):
        """Back-to-back calls (the host enqueues faster than the kernels run): mean and best of 3
        batches, ms per call."""
        for _ in range(3):
            fn()
        torch.cuda.synchronize()
        res = []
        for _ in range(3):
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a.record()
            for _ in range(reps):
                fn()
            b.record()
            torch.cuda.synchronize()
            res.append(a.elapsed_time(b) / reps)
        return sum(res) / len(res), min(res)

    for mode in ("count", "disc", "q6"):
        ms, mn = timed(lambda: call(mode), args.reps)
        print(json.dumps({"mode": mode, "kernel": _ar.ar_last_scan_kernel(), "cfg": os.environ.get("AR_RL_CFG"), "srs": args.srs,
                          "us_mean": ms * 1e3, "us_min": mn * 1e3,
                          "scan_stream_gbs": scan_bytes / (mn / 1e3) / 1e9, "peak": PEAK,
                          "out": out.tolist()}), flush=True)


if __name__ == "__main__":
    main()
