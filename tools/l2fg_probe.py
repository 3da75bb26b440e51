"""Probe: C4 one-pass query time with cudaLimitMaxL2FetchGranularity set (L2FG = 0/32/64/128 bytes)
before the library runs -- does a smaller L2 fetch granularity cut the gathers' DRAM traffic?

    L2FG=32 python tools/l2fg_probe.py
"""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    torch.cuda.init()
    fg = os.environ.get("L2FG")
    got = None
    if fg:
        from cuda.bindings import runtime as rt
        torch.zeros(1, device="cuda")
        err, = rt.cudaDeviceSetLimit(rt.cudaLimit.cudaLimitMaxL2FetchGranularity, int(fg))
        got = rt.cudaDeviceGetLimit(rt.cudaLimit.cudaLimitMaxL2FetchGranularity)
    cols = datagen.q6_columns(4, float(os.environ.get("SF", "100")))
    sd = cu.BWDColumn(cols["shipdate"], 24)
    dc, qt = cu.BWDColumn(cols["discount"], 32), cu.BWDColumn(cols["quantity"], 32)
    ep = cu.BWDColumn(cols["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    out = torch.zeros(4, dtype=torch.int64, device="cuda")
    for _ in range(5):
        cu.select_refine_sum(preds, [ep, dc], out)
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    reps = int(os.environ.get("REPS", "50"))
    a.record()
    for _ in range(reps):
        cu.select_refine_sum(preds, [ep, dc], out)
    b.record()
    torch.cuda.synchronize()
    print(json.dumps({"l2fg": fg, "limit": str(got), "ms": a.elapsed_time(b) / reps, "out": out.tolist(),
                      "kernel": _ar.ar_last_scan_kernel()}))


if __name__ == "__main__":
    main()
