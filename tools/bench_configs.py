"""Secondary measurements (BASELINE.json configs other than the headline C2):

  C1  1 M-row u32 column, 24/8 split, 1 % range      (latency / L2-resident; not a roofline point)
  C3  1 G-row u32 column: major-bit width {8,16,24} x selectivity sweep, positions out
  C5  SF1000-shaped Q6 per GPU share (750 M rows = SF125) with the l_shipdate residual in
      pinned host memory: HBM + host-link rooflines
  C4  the N = 1 point of C4: TPC-H SF100-shaped Q6 (600 M rows) on one GPU, one pass and staged
  MM  C2 (SF10 Q6 predicates) MIN / MAX(l_extendedprice): ar_approx_select + ar_minmax (s IV-F)
  GRP C2 shipdate + quantity predicates, SUM(l_extendedprice), COUNT group by l_discount (s IV-E)

    python tools/bench_configs.py c1|c3|c4|c5|mm|grp [--reps R]

One JSON line per point.  Timing as in bench.py: inputs resident, warm-up, CUDA
events on the launching stream around R back-to-back repetitions, L2 flushed
(512 MB write) before each repetition for the HBM-bound configs.
"""
import argparse
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402

PEAK = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json"))).get("hbm_gbs", 6650.0) \
    if os.path.exists(os.path.join(ROOT, "MEASURED_PEAKS.json")) else 6650.0


def timed(fn, reps, flush=None):
    """Mean ms per call over `reps` calls, each preceded by an (untimed) L2 flush."""
    for _ in range(2):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        if flush is not None:
            flush.zero_()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return statistics.mean(ts), min(ts)


def sectors(idx, bits_per_row, gran=32):
    b0 = idx.astype(np.int64) * bits_per_row
    return np.unique(np.concatenate([b0 // (gran * 8), (b0 + bits_per_row - 1) // (gran * 8)])).size


def c1(args):
    n = datagen.C1_N
    v = datagen.uniform_u32(1, n)
    col = cu.BWDColumn(v, 24)
    preds = [(col, datagen.C1_LO, datagen.C1_HI)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    pos = cu.PositionList(n)
    wr = cu.Workspace(_ar.ar_refine_ws_bytes(n))
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")

    def staged():
        cu.approx_select(preds, cands, ws)
        cu.refine(cands, preds, pos, wr)

    ms_s, _ = timed(staged, args.reps)
    ms_f, _ = timed(lambda: cu.select_refine_sum(preds, [], o4), args.reps)
    print(json.dumps({"config": "C1", "rows": n, "staged_select_refine_us": ms_s * 1e3,
                      "fused_count_us": ms_f * 1e3, "results": pos.count(),
                      "note": "L2-resident, latency-bound (not a roofline point)"}), flush=True)


def c3(args):
    n = 1_000_000_000
    v = datagen.uniform_u32(3, n)
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    for M in args.widths:
        col = cu.BWDColumn(v, M)
        k = 32 - M
        w = col.w_major
        cands = cu.CandidateList(n)
        ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
        pos = cu.PositionList(n)
        wr = cu.Workspace(_ar.ar_refine_ws_bytes(n))
        o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
        for s in args.sels:
            lo = 0x1234567
            hi = lo + int(s * 2**32) - 1
            preds = [(col, lo, hi)]
            # carry the approximation (4 B per candidate written + read) when many candidates are
            # non-definite (M = 8: 2/256 of the rows), else let refine gather the few majors it needs
            carry = M <= 8

            def sel():
                cu.approx_select(preds, cands, ws, carry=carry)

            def ref():
                cu.refine(cands, preds, pos, wr)

            ms_sel, _ = timed(sel, args.reps, flush)
            sel()
            ms_ref, _ = timed(ref, args.reps, flush)
            ms_fus, _ = timed(lambda: cu.select_refine_sum(preds, [], o4), args.reps, flush)
            torch.cuda.synchronize()
            nc, nr = cands.count(), pos.count()
            nd = int(o4[3].item())
            # two independent GPU paths must agree (staged select -> refine vs the one-pass kernel)
            consistent = nr == int(o4[1].item()) and nc == int(o4[2].item())
            # algorithmic bytes: majors scanned + candidate list (8 B) + non-definite residual
            # sectors + positions out (4 B)
            nondef = nc - nd
            scan = n * w / 8
            res_bytes = min(n * k / 8, 32.0 * max(1, nondef) * 1.0) if k else 0.0
            sel_bytes = scan + 8.0 * nc
            ref_bytes = 8.0 * nc + res_bytes + 4.0 * nr
            rows_s = n / ((ms_sel + ms_ref) / 1e3)
            print(json.dumps({
                "config": "C3", "rows": n, "major_bits": M, "k": k, "w_major": w, "selectivity": s, "carry": carry,
                "candidates": nc, "definite": nd, "results": nr, "staged_equals_one_pass": consistent,
                "select_ms": ms_sel, "refine_ms": ms_ref, "fused_count_ms": ms_fus,
                "select_refine_rows_per_s": rows_s,
                "select_frac": sel_bytes / (ms_sel / 1e3) / 1e9 / PEAK,
                "refine_frac": ref_bytes / (ms_ref / 1e3) / 1e9 / PEAK,
                "fused_count_frac": (scan + (res_bytes if k else 0)) / (ms_fus / 1e3) / 1e9 / PEAK,
                "peak_gbs": PEAK}), flush=True)
        del col, cands, pos, ws, wr


def c5(args):
    sf = 125                                    # SF1000 / 8 GPUs: 750 M rows per GPU
    c = datagen.q6_columns(5, 1000, n=sf * datagen.ROWS_PER_SF)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24, residual_loc=_ar.AR_LOC_HOST_PINNED)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")

    def staged():
        cu.approx_select(preds, cands, ws)
        cu.refine_sum(cands, preds, [ep, dc], s2[0:1], s2[1:2])

    ms_f, _ = timed(lambda: cu.select_refine_sum(preds, [ep, dc], o4), args.reps, flush)
    ms_s, _ = timed(staged, args.reps, flush)
    # host link: measured pinned -> device copy bandwidth
    h = torch.empty(1 << 30, dtype=torch.uint8).pin_memory()
    d = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
    ms_h2d, _ = timed(lambda: d.copy_(h, non_blocking=True), 5)
    link_gbs = (1 << 30) / (ms_h2d / 1e3) / 1e9
    # host bytes the refine must read: residual sectors of non-definite candidates (32 B and 64 B granules)
    sdv = c["shipdate"]
    major = sdv >> 8
    other = (c["discount"] >= 5) & (c["discount"] <= 7) & (c["quantity"] <= 23)
    nondef = np.nonzero(other & (major >= 2) & (major <= 4) & (major != 3))[0]
    host32 = 32.0 * sectors(nondef, 8, 32)
    host64 = 64.0 * sectors(nondef, 8, 64)
    print(json.dumps({
        "config": "C5 (per-GPU share)", "rows": n, "residual": "pinned host memory (zero-copy over PCIe)",
        "fused_ms": ms_f, "staged_ms": ms_s, "result_sum": int(o4[0].item()), "result_count": int(o4[1].item()),
        "fused_rows_per_s": n / (ms_f / 1e3), "staged_rows_per_s": n / (ms_s / 1e3),
        "h2d_link_gbs_measured": link_gbs,
        "host_bytes_32B_sectors": host32, "host_bytes_64B_granules": host64,
        "host_link_frac_fused": host32 / (ms_f / 1e3) / 1e9 / link_gbs,
        "host_link_frac_staged": host32 / (ms_s / 1e3) / 1e9 / link_gbs}), flush=True)


def c4(args):
    c = datagen.q6_columns(4, 100)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    srs_ws = cu.SrsWorkspace()

    def staged():
        cu.approx_select(preds, cands, ws)
        cu.refine_sum(cands, preds, [ep, dc], s2[0:1], s2[1:2])

    ms_f, mn_f = timed(lambda: cu.select_refine_sum(preds, [ep, dc], o4, ws=srs_ws), args.reps)
    ms_s, mn_s = timed(staged, args.reps)
    torch.cuda.synchronize()
    # algorithmic bytes (DESIGN s6): majors 1.75 B/row + touched residual / l_extendedprice sectors + 8 B
    sdv = c["shipdate"]
    oth = (c["discount"] >= 5) & (c["discount"] <= 7) & (c["quantity"] <= 23)
    major = sdv >> 8
    nondef = np.nonzero(oth & (major >= 2) & (major <= 4) & (major != 3))[0]
    res = np.nonzero(oth & (sdv >= datagen.Q6_SHIPDATE[0]) & (sdv <= datagen.Q6_SHIPDATE[1]))[0]
    alg = n * 14 / 8 + 32.0 * sectors(nondef, 8, 32) + 32.0 * sectors(res, 24, 32) + 8
    print(json.dumps({"config": "C4 (N=1 point: SF100 Q6, 600 M rows, one GPU)", "rows": n,
                      "fused_ms": ms_f, "staged_ms": ms_s, "fused_rows_per_s": n / (ms_f / 1e3),
                      "staged_rows_per_s": n / (ms_s / 1e3), "fused_frac": alg / (ms_f / 1e3) / 1e9 / PEAK,
                      "parity_staged_equals_one_pass": s2.tolist() == o4[:2].tolist(),
                      "sum": int(o4[0].item()), "count": int(o4[1].item()), "peak_gbs": PEAK,
                      "l2": "inputs 3.5 GB >> 126 MB L2 (no flush needed)"}), flush=True)


def mm(args):
    c = datagen.q6_columns(2, 10)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    wm = cu.Workspace(_ar.ar_minmax_ws_bytes(n))
    o7 = torch.zeros(7, dtype=torch.int64, device="cuda")
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    cu.approx_select(preds, cands, ws)
    torch.cuda.synchronize()
    pos = cands.positions()
    for mode in ("min", "max"):
        ms_sel, _ = timed(lambda: cu.approx_select(preds, cands, ws), args.reps, flush)
        ms_mm, _ = timed(lambda: cu.minmax(cands, preds, ep, mode, o7, wm), args.reps, flush)
        torch.cuda.synchronize()
        r = o7.cpu().tolist()
        # algorithmic bytes of ar_minmax: candidate list read (8 B), l_extendedprice sectors at
        # every candidate (the approximate pass needs every candidate's major), the kept majors
        # written and read back (8 B); the refined rows' gathers are a few rows (ignored)
        ep_bytes = 32.0 * sectors(pos, 24, 32)
        mm_bytes = 16.0 * pos.size + ep_bytes
        print(json.dumps({"config": "MM (C2 Q6, %s(l_extendedprice))" % mode.upper(), "rows": n,
                          "answer": r[0], "survivors": r[1], "approx_bounds": r[2:4], "refined": r[4],
                          "definite": r[5], "candidates": r[6], "select_us": ms_sel * 1e3, "minmax_us": ms_mm * 1e3,
                          "rows_per_s": n / ((ms_sel + ms_mm) / 1e3),
                          "minmax_frac": mm_bytes / (ms_mm / 1e3) / 1e9 / PEAK, "peak_gbs": PEAK}), flush=True)


def grp(args):
    c = datagen.q6_columns(2, 10)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24)
    qt = cu.BWDColumn(c["quantity"], 32)
    dc = cu.BWDColumn(c["discount"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, *datagen.Q6_SHIPDATE), (qt, *datagen.Q6_QUANTITY)]
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    cu.approx_select(preds, cands, ws)
    torch.cuda.synchronize()
    pos = cands.positions()
    ms_sel, _ = timed(lambda: cu.approx_select(preds, cands, ws), args.reps, flush)
    res = {}
    ms_grp, _ = timed(lambda: res.__setitem__("o", cu.refine_group_sum(cands, preds, dc, [ep], 16)), args.reps, flush)
    torch.cuda.synchronize()
    out = res["o"].cpu().numpy()
    # algorithmic bytes: candidate list (8 B), residual sectors of the non-definite candidates, the
    # key (l_discount, 4 b) and l_extendedprice sectors at the refined rows, 256 B out
    sdv = c["shipdate"]
    other = (c["quantity"] <= 23)
    major = sdv >> 8
    nondef = np.nonzero(other & (major >= 2) & (major <= 4) & (major != 3))[0]
    res_rows = np.nonzero(other & (sdv >= datagen.Q6_SHIPDATE[0]) & (sdv <= datagen.Q6_SHIPDATE[1]))[0]
    gb = 8.0 * pos.size + 32.0 * sectors(nondef, 8, 32) + 32.0 * sectors(res_rows, 4, 32) \
        + 32.0 * sectors(res_rows, 24, 32) + 256
    print(json.dumps({"config": "GRP (C2 shipdate+quantity, SUM(l_extendedprice) GROUP BY l_discount)", "rows": n,
                      "candidates": int(pos.size), "groups": int((out[1] > 0).sum()), "result_rows": int(out[1].sum()),
                      "select_us": ms_sel * 1e3, "group_sum_us": ms_grp * 1e3,
                      "rows_per_s": n / ((ms_sel + ms_grp) / 1e3),
                      "group_sum_frac": gb / (ms_grp / 1e3) / 1e9 / PEAK, "peak_gbs": PEAK}), flush=True)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("config", choices=["c1", "c3", "c4", "c5", "mm", "grp"])
    ap.add_argument("--reps", type=int, default=10)
    ap.add_argument("--widths", type=int, nargs="+", default=[8, 16, 24], help="C3 major bits")
    ap.add_argument("--sels", type=float, nargs="+", default=[0.0001, 0.001, 0.01, 0.1, 0.5], help="C3 selectivities")
    args = ap.parse_args()
    torch.cuda.set_device(0)
    {"c1": c1, "c3": c3, "c4": c4, "c5": c5, "mm": mm, "grp": grp}[args.config](args)


if __name__ == "__main__":
    main()
