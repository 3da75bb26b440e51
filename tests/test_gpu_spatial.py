"""GPU parity for signed / frame-of-reference decomposition and the spatial range
count of Table I: int32 lon/lat in 1e-5
degrees, bwdecompose(lon, 24), bwdecompose(lat, 24), two BETWEEN predicates,
COUNT.  Everything is checked against the oracle's plain int32 definition."""
import numpy as np
import pytest

import datagen
import oracle
from tests._layout import unpack_packed, unpack_sliced

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")

FLIP = 0x80000000


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def _key(v):
    """Order-preserving key of int32 values as uint32, computed test-side."""
    return (np.asarray(v, dtype=np.int32).view(np.uint32) ^ np.uint32(FLIP)).astype(np.uint32)


def _bytes(t):
    return t.cpu().numpy().tobytes()


@pytest.mark.parametrize("major_bits,layout", [(24, 0), (24, 1), (20, 0), (28, 1)])
def test_gpu_decompose_signed_base_min(cu, major_bits, layout):
    c = datagen.spatial_columns(3, 300_001)
    v = c["lon"]
    col = cu.BWDColumn(v, major_bits, layout=layout, signed=True, base="min")
    key = _key(v)
    assert col.desc.value_signed == 1 and col.desc.base == int(key.min())
    k = 32 - major_bits
    major, residual, w = oracle.decompose(key, k, int(key.min()))
    assert col.w_major == w
    dec = unpack_sliced if layout == 0 else unpack_packed
    assert np.array_equal(dec(_bytes(col.major), v.size, w), major)
    rdec = unpack_sliced if col.desc.residual_layout == 0 else unpack_packed
    assert np.array_equal(rdec(_bytes(col.residual), v.size, k), residual)


def test_gpu_base_above_min_rejected(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = np.arange(100, 5000, dtype=np.uint32)
    with pytest.raises(_ar.ARError) as e:
        cu.BWDColumn(v, 24, base=101)
    assert e.value.status == _ar.AR_ERR_RANGE
    cu.BWDColumn(v, 24, base=100)


def _run_all(cu, cols, los, his, values, signed):
    """approx_select -> refine, refine_sum (COUNT), fused COUNT, project; all vs the oracle."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = cols[0].n
    preds = [(c, lo & 0xFFFFFFFF, hi & 0xFFFFFFFF) for c, lo, hi in zip(cols, los, his)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    out = cu.PositionList(n)
    cu.refine(cands, preds, out, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, [], torch.zeros(1, dtype=torch.int64, device="cuda"), cnt)
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [], o4)
    b4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.sum_approximate(cands, [], b4)
    torch.cuda.synchronize()
    ref_pos, ref_cnt, _ = oracle.select_sum(values, los, his, signed=signed)
    assert out.count() == ref_cnt and np.array_equal(out.positions(), ref_pos)
    assert int(cnt.item()) == ref_cnt
    # candidates / definite flags: the oracle's bucket rule on the keys with the keys' bounds
    keys = [_key(v) if s else np.asarray(v, dtype=np.uint32) for v, s in zip(values, signed)]
    klo = [(lo & 0xFFFFFFFF) ^ (FLIP if s else 0) for lo, s in zip(los, signed)]
    khi = [(hi & 0xFFFFFFFF) ^ (FLIP if s else 0) for hi, s in zip(his, signed)]
    bases = [int(c.desc.base) for c in cols]
    cpos, cdef = oracle.approx_select(keys, [c.k for c in cols], klo, khi, base=bases)
    assert np.array_equal(cands.positions(), cpos) and np.array_equal(cands.definite(), cdef)
    assert o4.cpu().tolist() == [0, ref_cnt, cpos.size, int(cdef.sum())]
    assert b4.cpu().tolist() == [0, 0, int(cdef.sum()), cpos.size]
    # projection of the signed column back to int32 values at the refined rows
    ex = cu.project(out, cols[0], exact=True)
    torch.cuda.synchronize()
    assert np.array_equal(ex[:ref_cnt].cpu().numpy(), np.asarray(values[0], dtype=np.int32)[ref_pos])
    return ref_cnt, cpos.size, int(cdef.sum())


@pytest.mark.parametrize("n", [1, 4097, 2_000_003])
def test_gpu_spatial_table1(cu, n):
    c = datagen.spatial_columns(6, n)
    cols = [cu.BWDColumn(c["lon"], 24, signed=True, base="min"), cu.BWDColumn(c["lat"], 24, signed=True, base="min")]
    los = [datagen.SPATIAL_LON[0], datagen.SPATIAL_LAT[0]]
    his = [datagen.SPATIAL_LON[1], datagen.SPATIAL_LAT[1]]
    cnt, ncand, ndef = _run_all(cu, cols, los, his, [c["lon"], c["lat"]], [True, True])
    if n > 1_000_000:
        assert cnt > 1000 and ncand > cnt > ndef > 0


@pytest.mark.parametrize("lo,hi", [(-5, 5), (-2**31, -1), (0, 2**31 - 1), (-2**31, 2**31 - 1), (7, 3),
                                   (-1_262_427, -1_262_427)])
def test_gpu_signed_ranges(cu, lo, hi):
    # ranges across zero, the whole negative / positive half, everything, empty, one value
    v = datagen.spatial_columns(9, 300_000)["lon"].copy()
    v[:64] = np.array([-5, 5, -6, 6, 0, -1, -2**31, 2**31 - 1] * 8, dtype=np.int32)
    for base in (0, "min"):
        col = cu.BWDColumn(v, 24, signed=True, base=base)
        _run_all(cu, [col], [lo], [hi], [v], [True])


def test_gpu_signed_sum_unsupported(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.spatial_columns(4, 10_000)["lon"]
    col = cu.BWDColumn(v, 24, signed=True, base="min")
    cands = cu.CandidateList(col.n)
    cu.approx_select([(col, 0, 2**31 - 1)], cands, cu.Workspace(_ar.ar_select_ws_bytes(col.n)))
    with pytest.raises(_ar.ARError) as e:
        cu.sum_approximate(cands, [col], torch.zeros(4, dtype=torch.int64, device="cuda"))
    assert e.value.status == _ar.AR_ERR_UNSUPPORTED
