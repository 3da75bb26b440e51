"""Small-size driver for compute-sanitizer (racecheck / synccheck / memcheck): one call of every
hot-path entry point on Q6-shaped data, each result checked against the oracle so a run that
skipped a kernel cannot pass silently.  Kernel selection knobs are environment variables read
once per process (AR_RL_RESMODE, AR_FUSED_LEGACY, AR_SEL_BUFS; SPLIT = the l_shipdate residual in the
split layout with that many high planes apart), so tools/sanitize.sh runs this
driver once per configuration.

    compute-sanitizer --tool racecheck python tools/sanitize_driver.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import datagen  # noqa: E402
import oracle  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    n = int(os.environ.get("N", "70001"))
    c = datagen.q6_columns(81, 1.0, n=n)
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    res_loc = int(os.environ.get("RES_LOC", "0"))
    sd = cu.BWDColumn(c["shipdate"], 24, residual_loc=res_loc, split=int(os.environ.get("SPLIT", "0")))
    dc, qt = cu.BWDColumn(c["discount"], 32), cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, los[0], his[0]), (dc, los[1], his[1]), (qt, los[2], his[2])]
    ref_pos, ref_cnt, ref_sum = oracle.select_sum(vals, los, his, [c["extprice"], c["discount"]])
    cpos, cdef = oracle.approx_select(vals, [8, 0, 0], los, his)
    ran = []

    # one pass (fused_rl / fused_rg / fused_kernel), plain and workspace + PDL
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [ep, dc], o4)
    torch.cuda.synchronize()
    ran.append(_ar.ar_last_scan_kernel())
    assert o4.tolist() == [ref_sum, ref_cnt, cpos.size, int(cdef.sum())], o4.tolist()
    ws = cu.SrsWorkspace()
    for _ in range(3):
        cu.select_refine_sum(preds, [ep, dc], o4, ws=ws, flags=_ar.AR_SRS_PDL_EARLY_READ)
    torch.cuda.synchronize()
    assert o4.tolist() == [ref_sum, ref_cnt, cpos.size, int(cdef.sum())], o4.tolist()

    # staged: select (tile kernel + compaction), refine (positions), refine + SUM, SUM
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    ran.append(_ar.ar_last_scan_kernel())
    pos = cu.PositionList(n)
    cu.refine(cands, preds, pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    ran.append(_ar.ar_last_scan_kernel())
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, [ep, dc], s2[0:1], s2[1:2])
    ran.append(_ar.ar_last_scan_kernel())
    s1 = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.sum_at(pos, [ep, dc], s1)
    torch.cuda.synchronize()
    assert np.array_equal(cands.positions(), cpos) and np.array_equal(cands.definite(), cdef)
    assert np.array_equal(pos.positions(), ref_pos)
    assert s2.tolist() == [ref_sum, ref_cnt] and int(s1.item()) == ref_sum

    # MIN / MAX and grouping (dense key, hashed ids)
    out7 = torch.zeros(7, dtype=torch.int64, device="cuda")
    cu.minmax(cands, preds, ep, "min", out7)
    ran.append(_ar.ar_last_scan_kernel())
    want = oracle.select_minmax(vals, los, his, c["extprice"], "min")
    torch.cuda.synchronize()
    assert int(out7[0].item()) == want[0]
    g = cu.refine_group_sum(cands, preds, dc, [ep], 16)
    ran.append(_ar.ar_last_scan_kernel())
    gr = cu.group_ids(cands, qt, cu.Grouping(n, 64))
    gs = cu.refine_group_sum_ids(cands, preds, gr, [ep, dc])
    torch.cuda.synchronize()
    sums, cnts = oracle.select_group_sum(vals, los, his, c["discount"], 16, [c["extprice"]])
    assert g[1].cpu().tolist() == cnts.tolist() and g[0].cpu().tolist() == sums.tolist()
    keys = gr.group_keys()
    got = {int(keys[i]): int(gs[1, i].item()) for i in range(gr.ngroups()) if gs[1, i].item() > 0}
    k2, c2, _ = oracle.select_group_sum_keys(vals, los, his, c["quantity"])
    assert got == dict(zip(k2.tolist(), c2.tolist()))

    # one pass over a bit-packed residual (k = 24, C3 at M = 8): check entries, COUNT and SUM
    v = datagen.uniform_u32(91, n)
    col = cu.BWDColumn(v, 8)
    lo, hi = 0x5A5A5A37, 0x5A5A5A37 + (1 << 32) // 100
    _, pc, ps = oracle.select_sum([v], [lo], [hi], [c["extprice"]], positions=False)
    pcp, pcd = oracle.approx_select([v], [24], [lo], [hi])
    for aggs, want in (([], 0), ([ep], ps)):
        cu.select_refine_sum([(col, lo, hi)], aggs, o4)
        torch.cuda.synchronize()
        assert o4.tolist() == [want, pc, pcp.size, int(pcd.sum())], o4.tolist()
    ran.append(_ar.ar_last_scan_kernel() + "(packed)")
    print("sanitize driver ok:", ",".join(ran), flush=True)


if __name__ == "__main__":
    main()
