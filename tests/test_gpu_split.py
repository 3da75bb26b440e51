"""GPU parity of the split residual layout (ar_column_desc.residual_split, DESIGN s6.3d): the
residual's h high planes stored apart from its low planes, so that refinement can decide most
non-definite candidates from the high planes alone (the bucket rule at granularity 2^(k-h), the
A&R approximation applied to the residual itself) and read the low planes only for the rest.
Every consumer of residuals -- ar_refine, ar_refine_sum, the one-pass kernels (gathered-residual
kernel; general kernel), MIN / MAX, exact grouping, projection -- must return results identical to
the oracle for any split, in HBM and in pinned host memory."""
import numpy as np
import pytest

import datagen
import oracle
from tests._layout import unpack_split

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")

LOS = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
HIS = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


@pytest.mark.parametrize("k,h", [(8, 1), (8, 2), (8, 3), (8, 7), (4, 2), (6, 5)])
@pytest.mark.parametrize("n", [1, 1023, 1025, 70_001])
def test_gpu_split_decompose_layout(cu, k, h, n):
    v = datagen.uniform_u32(80 + k, n)
    col = cu.BWDColumn(v, 32 - k, split=h)
    assert col.desc.residual_split == h and col.desc.residual_bytes == -(-n // 8192) * 1024 * k
    _, residual, _ = oracle.decompose(v, k)
    got = unpack_split(col.residual.cpu().numpy().tobytes(), n, k, h)
    assert np.array_equal(got, residual.astype(np.uint64))


def test_gpu_split_rejected(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.uniform_u32(88, 1000)
    for bits, h in [(24, 8), (20, 2), (31, 1)]:   # h >= k, k > 8 (PACKED residual), h >= k
        with pytest.raises(_ar.ARError):
            cu.BWDColumn(v, bits, split=h)


@pytest.mark.parametrize("loc", [0, 1])
@pytest.mark.parametrize("h", [1, 2, 3, 7])
def test_gpu_split_q6_every_path(cu, loc, h):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 300_017
    c = datagen.q6_columns(83, 1.0, n=n)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    sd = cu.BWDColumn(vals[0], 24, residual_loc=loc, split=h)
    dc, qt = cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, LOS[0], HIS[0]), (dc, LOS[1], HIS[1]), (qt, LOS[2], HIS[2])]
    ref_pos, ref_cnt, ref_sum = oracle.select_sum(vals, LOS, HIS, [c["extprice"], c["discount"]])
    cpos, cdef = oracle.approx_select(vals, [8, 0, 0], LOS, HIS)
    # one pass (progressive refinement from the high planes): HBM residual with a compiled split shape ->
    # the result-ring kernel streaming the high planes; otherwise the gathered-residual kernel
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [ep, dc], o4)
    torch.cuda.synchronize()
    assert _ar.ar_last_scan_kernel() == ("fused_rl_kernel" if loc == 0 and h in (2, 3, 4) else "fused_rg_kernel")
    assert o4.cpu().tolist() == [ref_sum, ref_cnt, cpos.size, int(cdef.sum())]
    o1 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [], o1)   # COUNT: no result ring -> gathered-residual kernel
    torch.cuda.synchronize()
    assert _ar.ar_last_scan_kernel() == "fused_rg_kernel"
    assert o1.cpu().tolist() == [0, ref_cnt, cpos.size, int(cdef.sum())]

    # staged
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    pos = cu.PositionList(n)
    cu.refine(cands, preds, pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, [ep, dc], s2[0:1], s2[1:2])
    torch.cuda.synchronize()
    assert np.array_equal(pos.positions(), ref_pos)
    assert s2.cpu().tolist() == [ref_sum, ref_cnt]
    # MIN / MAX of the split column itself, exact projection, exact grouping by it
    out7 = torch.zeros(7, dtype=torch.int64, device="cuda")
    cu.minmax(cands, preds, sd, "max", out7)
    torch.cuda.synchronize()
    assert int(out7[0].item()) == oracle.select_minmax(vals, LOS, HIS, vals[0], "max")[0]
    ex = cu.project(pos, sd, exact=True)
    torch.cuda.synchronize()
    assert np.array_equal(ex[:ref_cnt].cpu().numpy().view(np.uint32), vals[0][ref_pos])
    gr = cu.group_ids(cands, sd, cu.Grouping(n, 1024), exact=True)
    out = cu.refine_group_sum_ids(cands, preds, gr, [ep, dc]).cpu().numpy()
    keys = gr.group_keys()
    got = {int(keys[g]): (int(out[1, g]), int(out[0, g])) for g in range(gr.ngroups()) if out[1, g] > 0}
    k2, c2, s2k = oracle.select_group_sum_keys(vals, LOS, HIS, vals[0], [c["extprice"], c["discount"]])
    assert got == {int(a): (int(b), int(d)) for a, b, d in zip(k2, c2, s2k)}


def test_gpu_split_general_kernel_and_spatial(cu):
    # two decomposed signed predicates with split residuals (FOR base): gathered-residual kernel when the
    # shape is compiled, the general kernel otherwise -- both must match the oracle
    n = 200_003
    s = datagen.spatial_columns(84, n)
    lon, lat = np.asarray(s["lon"], dtype=np.int32), np.asarray(s["lat"], dtype=np.int32)
    cl = [cu.BWDColumn(lon, 24, signed=True, base="min", split=3), cu.BWDColumn(lat, 24, signed=True, split=2)]
    los, his = [-900_000, 4_000_000], [600_000, 6_000_000]
    preds = [(c, lo & 0xFFFFFFFF, hi & 0xFFFFFFFF) for c, lo, hi in zip(cl, los, his)]
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [], o4)
    torch.cuda.synchronize()
    _, cnt, _ = oracle.select_sum([lon, lat], los, his, signed=[True, True], positions=False)
    cpos, cdef = oracle.approx_select([lon, lat], [8, 8], los, his, base=[int(c.desc.base) for c in cl],
                                      signed=[True, True])
    assert o4.cpu().tolist() == [0, cnt, cpos.size, int(cdef.sum())]


@pytest.mark.parametrize("h", [2, 3, 4])
@pytest.mark.parametrize("bounds", [(731, 1095), (800, 805), (768, 1023), (0, 0xFFFFFFFF), (1, 2526), (1000, 1000),
                                    (1024, 1040), (2520, 5000), (1, 5), (3, 20), (2500, 2510), (0, 0)])
@pytest.mark.parametrize("loc", [0, 1])
def test_gpu_split_stream_bounds(cu, h, bounds, loc):
    """Check entries of the split residual at bound placements the check code must get right: both bounds
    inside one fine bucket (code 3), bucket-aligned bounds (no undecided rows), the whole domain, a point
    predicate, a bound past the data; 8192-row tiles with a ragged tail.  HBM residual: the result-ring
    kernel streaming the high planes; pinned host residual: the gathered-residual kernel (high planes
    gathered in phase A, low planes with the aggregate)."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 3 * 8192 + 77_777
    c = datagen.q6_columns(90 + h, 1.0, n=n)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    los, his = [bounds[0], LOS[1], LOS[2]], [bounds[1], HIS[1], HIS[2]]
    sd = cu.BWDColumn(vals[0], 24, split=h, residual_loc=loc)
    dc, qt = cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, los[0], his[0]), (dc, los[1], his[1]), (qt, los[2], his[2])]
    _, ref_cnt, ref_sum = oracle.select_sum(vals, los, his, [c["extprice"], c["discount"]], positions=False)
    cpos, cdef = oracle.approx_select(vals, [8, 0, 0], los, his)
    for aggs, want in (([ep, dc], ref_sum), ([ep], None)):
        o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
        cu.select_refine_sum(preds, aggs, o4)
        torch.cuda.synchronize()
        assert _ar.ar_last_scan_kernel() == ("fused_rl_kernel" if loc == 0 else "fused_rg_kernel")
        if want is None:
            _, _, want = oracle.select_sum(vals, los, his, [c["extprice"]], positions=False)
        assert o4.cpu().tolist() == [want, ref_cnt, cpos.size, int(cdef.sum())]
