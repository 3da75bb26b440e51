"""Profiling driver: build the C2 workload (SF10 Q6, 60 M rows) and run a few
eager steps of each variant, so that ncu can capture single launches:

  ncu --set full --clock-control none --import-source on -k regex:'select_kernel|refine_sum_kernel|fused_kernel' \
      -s 6 -c 3 -o gpurun_out/prof python tools/profile_step.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    sf = float(os.environ.get("SF", "10"))
    steps = int(os.environ.get("STEPS", "4"))
    variants = os.environ.get("VARIANTS", "staged,fused").split(",")
    if os.environ.get("L2FG"):
        from cuda.bindings import runtime as rt
        torch.cuda.init()
        err, = rt.cudaDeviceSetLimit(rt.cudaLimit.cudaLimitMaxL2FetchGranularity, int(os.environ["L2FG"]))
        print("set L2 fetch granularity", os.environ["L2FG"], err, rt.cudaDeviceGetLimit(rt.cudaLimit.cudaLimitMaxL2FetchGranularity))
    cols = datagen.q6_columns(int(os.environ.get("SEED", "2")), sf)
    n = cols["shipdate"].size
    # RES_LOC=1: the l_shipdate residual in pinned host memory (the C5 mechanism, read over the host link)
    sd = cu.BWDColumn(cols["shipdate"], 24, residual_loc=int(os.environ.get("RES_LOC", "0")),
                      split=int(os.environ.get("SPLIT", "0")))
    dc = cu.BWDColumn(cols["discount"], 32)
    qt = cu.BWDColumn(cols["quantity"], 32)
    ep = cu.BWDColumn(cols["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    out = torch.zeros(4, dtype=torch.int64, device="cuda")
    pos = cu.PositionList(n) if "refine" in variants else None
    wr = cu.Workspace(_ar.ar_refine_ws_bytes(n)) if "refine" in variants else None
    flush = torch.empty(512 * 1024 * 1024, dtype=torch.uint8, device="cuda")
    for v in variants:
        for _ in range(steps):
            flush.zero_()
            if v == "staged":
                cu.approx_select(preds, cands, ws, carry=True)
                cu.refine_sum(cands, preds, [ep, dc], out[0:1], out[1:2])
            elif v == "refine":   # a5 as its own step: ordered positions out (ar_refine)
                cu.approx_select(preds, cands, ws, carry=True)
                cu.refine(cands, preds, pos, wr)
                out[1] = pos.count_t[0]
            else:
                cu.select_refine_sum(preds, [ep, dc], out)
        torch.cuda.synchronize()
        print(v, out.tolist(), flush=True)


if __name__ == "__main__":
    main()
