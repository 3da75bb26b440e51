"""Parity at BASELINE.json's full sizes, in the launch configurations bench.py
times: C2 (SF10 Q6, 60 M rows), C3 (1 G-row u32 column, 24/8 split, 1 %), and the
C5 mechanism (shipdate residual in pinned host memory) at SF10.  The oracle runs
the plain definition over the whole table (multi-threaded C, seconds)."""
import numpy as np
import pytest

import datagen
import oracle

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")

Q6_LO = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
Q6_HI = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def _q6(cu, sf, residual_loc):
    from paper_conf_icde_pirkmk14_b200 import _ar
    c = datagen.q6_columns(2, sf)
    n = c["shipdate"].size
    sd = cu.BWDColumn(c["shipdate"], 24, residual_loc=residual_loc)
    dc = cu.BWDColumn(c["discount"], 32)
    qt = cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, Q6_LO[0], Q6_HI[0]), (dc, Q6_LO[1], Q6_HI[1]), (qt, Q6_LO[2], Q6_HI[2])]
    values = [c["shipdate"], c["discount"], c["quantity"]]
    ref_pos, ref_cnt, ref_sum = oracle.select_sum(values, Q6_LO, Q6_HI, [c["extprice"], c["discount"]], threads=0)
    # staged: approximate select -> refine positions, refine + SUM
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    pos = cu.PositionList(n)
    cu.refine(cands, preds, pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, [ep, dc], s2[0:1], s2[1:2])
    # one pass
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [ep, dc], o4)
    torch.cuda.synchronize()
    assert np.array_equal(pos.positions(), ref_pos)
    assert s2.tolist() == [ref_sum, ref_cnt]
    cpos, cdef = oracle.approx_select(values, [8, 0, 0], Q6_LO, Q6_HI)
    assert o4.tolist() == [ref_sum, ref_cnt, cpos.size, int(cdef.sum())]
    # candidate relation: compare on a deterministic sample of entries (the full list is 2.4 M)
    got = cands.positions()
    assert got.size == cpos.size
    idx = np.unique(np.linspace(0, cpos.size - 1, 4096).astype(np.int64))
    assert np.array_equal(got[idx], cpos[idx]) and np.array_equal(cands.definite()[idx], cdef[idx])


def test_gpu_c2_sf10_full(cu):
    _q6(cu, 10, 0)


def test_gpu_c5_mechanism_host_residual_sf10(cu):
    _q6(cu, 10, 1)


def test_gpu_c3_1g_rows_24_8_one_percent(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 1_000_000_000
    v = datagen.uniform_u32(3, n)
    lo = 0x3C3C3C37
    hi = lo + int(0.01 * 2**32) - 1
    col = cu.BWDColumn(v, 24)
    cands = cu.CandidateList(n)
    cu.approx_select([(col, lo, hi)], cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    pos = cu.PositionList(n)
    cu.refine(cands, [(col, lo, hi)], pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum([(col, lo, hi)], [], o4)
    torch.cuda.synchronize()
    ref_pos, ref_cnt, _ = oracle.select_sum([v], [lo], [hi], threads=0)
    got = pos.positions()
    assert got.size == ref_cnt and np.array_equal(got, ref_pos)
    assert int(o4[1].item()) == ref_cnt
    # candidate and definite counts from the oracle's bucket rule (k = 24)
    cpos, cdef = oracle.approx_select([v], [8], [lo], [hi])
    assert cands.count() == cpos.size and int(o4[2].item()) == cpos.size and int(o4[3].item()) == int(cdef.sum())
    idx = np.unique(np.linspace(0, cpos.size - 1, 4096).astype(np.int64))
    assert np.array_equal(cands.positions()[idx], cpos[idx])


def test_gpu_max_rows_u32_positions(cu):
    """Maximum size: positions are u32 per column (ar.h), so a column holds < 2^32 rows.  A ragged
    column of 2^32 - 2^20 - 5 rows (4.29 G; 17 GB of values) through select -> refine -> SUM and
    the one-pass COUNT: every 64-bit index / offset path past 2^31 and the ragged last tile."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    free, _ = torch.cuda.mem_get_info()
    n = 2**32 - 2**20 - 5
    if free < 110 * 2**30:
        pytest.skip("needs ~110 GB of free device memory")
    v = datagen.uniform_u32(41, n)
    lo, hi = 0xF0000123, 0xF0000123 + (2**32 // 1000)   # 0.1 %, near the top of the domain
    col = cu.BWDColumn(v, 24)
    ref_pos, ref_cnt, ref_sum = oracle.select_sum([v], [lo], [hi], [v], threads=0)
    cpos, cdef = oracle.approx_select([v], [8], [lo], [hi])
    preds = [(col, lo, hi)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    torch.cuda.synchronize()
    got = cands.positions()
    assert got.size == cpos.size and np.array_equal(got, cpos)
    assert np.array_equal(cands.definite(), cdef)
    pos = cu.PositionList(cands.c.capacity)
    cu.refine(cands, preds, pos, cu.Workspace(_ar.ar_refine_ws_bytes(cands.c.capacity)))
    s2 = torch.zeros(2, dtype=torch.int64, device="cuda")
    # SUM of a 32-bit column over up to 2^32 rows could overflow int64: the ABI refuses it (ar.h)
    with pytest.raises(_ar.ARError, match="AR_ERR_RANGE"):
        cu.refine_sum(cands, preds, [col], s2[0:1], s2[1:2])
    cu.refine_sum(cands, preds, [], s2[0:1], s2[1:2])
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [], o4)
    torch.cuda.synchronize()
    assert np.array_equal(pos.positions(), ref_pos)
    assert s2.tolist() == [0, ref_cnt]
    assert oracle.sum_at(ref_pos, [v]) == ref_sum and ref_sum > 0
    assert o4.tolist() == [0, ref_cnt, cpos.size, int(cdef.sum())]
    assert ref_pos[-1] > 2**31   # results past 2^31 really exercised
