"""Time the staged A&R calls on the C2 workload (SF10 Q6, 60 M rows), inputs
rotated over 3 copies (> L2): ar_approx_select (with the approximation tuple)
and ar_refine_sum, each back to back, and check the SUM against the fused call.

    AR_SEL_CTAS=3 python tools/time_staged.py [--reps R]

One JSON line: us per call (mean / best of 3 batches) and GB/s of the
algorithmic bytes of each step (DESIGN s6).
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def timed(fn, reps):
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
    return sum(res) / len(res) * 1e3, min(res) * 1e3


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--reps", type=int, default=30)
    ap.add_argument("--sf", type=float, default=10.0)
    args = ap.parse_args()
    c = datagen.q6_columns(2, args.sf)
    n = c["shipdate"].size
    base = (cu.BWDColumn(c["shipdate"], 24), cu.BWDColumn(c["discount"], 32), cu.BWDColumn(c["quantity"], 32),
            cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED))
    sets = [base] + [tuple(x.copy() for x in base) for _ in range(2)]
    preds = [[(a, *datagen.Q6_SHIPDATE), (b, *datagen.Q6_DISCOUNT), (q, *datagen.Q6_QUANTITY)]
             for a, b, q, _ in sets]
    cands = [cu.CandidateList(n) for _ in range(3)]
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    out = torch.zeros(4, dtype=torch.int64, device="cuda")
    it = [0]

    def sel():
        i = it[0] % 3
        it[0] += 1
        cu.approx_select(preds[i], cands[i], ws, carry=True)

    def ref():
        i = it[0] % 3
        it[0] += 1
        cu.refine_sum(cands[i], preds[i], [sets[i][3], sets[i][1]], out[0:1], out[1:2])

    for i in range(3):
        cu.approx_select(preds[i], cands[i], ws, carry=True)
    torch.cuda.synchronize()
    ncand = cands[0].count()
    sel_ms = timed(sel, args.reps)
    kern = _ar.ar_last_scan_kernel()
    ref_ms = timed(ref, args.reps)
    got = out[:2].tolist()
    chk = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds[0], [sets[0][3], sets[0][1]], chk)
    ok = got == chk[:2].tolist()
    scan_bytes = n * 14 / 8 + 8 * ncand
    print(json.dumps({"select_kernel": kern, "cands": ncand, "select_us": sel_ms, "refine_sum_us": ref_ms,
                      "select_gbs": scan_bytes / (sel_ms[1] * 1e-6) / 1e9, "sum_count": got, "match_fused": ok,
                      "env": {k: v for k, v in os.environ.items() if k.startswith("AR_")}}), flush=True)


if __name__ == "__main__":
    main()
