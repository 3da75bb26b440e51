"""Profiling driver for the ordered refine (ar_refine, positions out) on a C3-shaped
column: N uniform u32 rows, M major bits, one range of selectivity S.

    ncu --set full -k regex:refine_kernel -s 1 -c 1 python tools/profile_refine.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    n = int(float(os.environ.get("N", "2e8")))
    M = int(os.environ.get("M", "24"))
    sel = float(os.environ.get("S", "0.5"))
    v = datagen.uniform_u32(3, n)
    col = cu.BWDColumn(v, M)
    lo = 0x1234567
    preds = [(col, lo, lo + int(sel * 2**32) - 1)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)), carry=False)
    pos = cu.PositionList(n)
    wr = cu.Workspace(_ar.ar_refine_ws_bytes(n))
    for _ in range(3):
        cu.refine(cands, preds, pos, wr)
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    cu.refine(cands, preds, pos, wr)
    b.record()
    torch.cuda.synchronize()
    print("cands", cands.count(), "results", pos.count(), "refine_ms", a.elapsed_time(b), flush=True)


if __name__ == "__main__":
    main()
