"""GPU parity of ar_minmax (MIN / MAX with the selection's error bounds
propagated to the aggregation, s IV-F, Fig. 6) against the
oracle, bit-exact on every output word: the refined answer, survivors, the
approximate bounds, the number of refined candidates, |D| and |C|."""
import numpy as np
import pytest

import datagen
import oracle

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def run_minmax(cu, pcols, los, his, ycol, mode, carry=True):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = pcols[0].n
    preds = [(c, lo & 0xFFFFFFFF, hi & 0xFFFFFFFF) for c, lo, hi in zip(pcols, los, his)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)), carry=carry)
    out7 = torch.full((7,), -99, dtype=torch.int64, device="cuda")
    cu.minmax(cands, preds, ycol, mode, out7)
    torch.cuda.synchronize()
    return out7.cpu().tolist()


def expect(pvals, pcols, los, his, yvals, ycol, mode, y_signed=False, pred_signed=None):
    r = oracle.minmax_ar(pvals, [c.k for c in pcols], los, his, yvals, ycol.k, mode,
                         pred_bases=[int(c.desc.base) for c in pcols], y_base=int(ycol.desc.base), y_signed=y_signed,
                         pred_signed=pred_signed)
    exact = oracle.select_minmax(pvals, los, his, yvals, mode, signed=pred_signed, y_signed=y_signed)
    assert (r["value"], r["survivors"] > 0) == (exact[0], exact[1] > 0)   # A&R reaches the plain answer
    return [r["value"], r["survivors"], r["lo"], r["hi"], r["refined"], r["definite"], r["candidates"]]


def test_gpu_minmax_fig6(cu, golden):
    g = golden("fig6_minmax_table.txt")
    k = int(g["k"])
    x = np.array([int(v) for v in g["x"].split(",")], dtype=np.uint32)
    y = np.array([int(v) for v in g["y"].split(",")], dtype=np.uint32)
    xc, yc = cu.BWDColumn(x, 32 - k), cu.BWDColumn(y, 32 - k)
    got = run_minmax(cu, [xc], [int(g["precise_lo"])], [0xFFFFFFFF], yc, "min")
    assert got[0] == int(g["precise_min"])
    assert got[2:4] == [int(g["approx_lo"]), int(g["approx_hi"])]
    assert got == expect([x], [xc], [int(g["precise_lo"])], [0xFFFFFFFF], y, yc, "min")


@pytest.mark.parametrize("mode", ["min", "max"])
@pytest.mark.parametrize("n,xk,yk", [(1, 8, 8), (1000, 4, 12), (65_537, 8, 8), (300_001, 12, 4), (300_001, 0, 16)])
def test_gpu_minmax_random(cu, mode, n, xk, yk):
    x = datagen.uniform_u32(11 + n, n, 0, 1 << 20)
    y = datagen.uniform_u32(13 + n, n)
    xc, yc = cu.BWDColumn(x, 32 - xk), cu.BWDColumn(y, 32 - yk)
    lo, hi = 300_001, 650_000
    assert run_minmax(cu, [xc], [lo], [hi], yc, mode) == expect([x], [xc], [lo], [hi], y, yc, mode)


@pytest.mark.parametrize("mode", ["min", "max"])
def test_gpu_minmax_of_predicate_column(cu, mode):
    # Y is the (decomposed) predicate column itself: its major comes from the carried
    # approximation, its residual is gathered at the refined rows
    n = 200_003
    x = datagen.uniform_u32(21, n)
    xc = cu.BWDColumn(x, 24)
    lo, hi = 0x5A5A5A37, 0x5A5A5A37 + 40_000_000
    for carry in (True, False):
        assert run_minmax(cu, [xc], [lo], [hi], xc, mode, carry) == expect([x], [xc], [lo], [hi], x, xc, mode)


@pytest.mark.parametrize("mode", ["min", "max"])
def test_gpu_minmax_q6_extendedprice(cu, mode):
    # MIN / MAX(l_extendedprice) under the Q6 predicates; l_extendedprice whole or decomposed 24/8
    # with its residual in pinned host memory
    c = datagen.q6_columns(31, 0.3)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    cols = [cu.BWDColumn(vals[0], 24), cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)]
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    for ep in (cu.BWDColumn(c["extprice"], 32, layout=1), cu.BWDColumn(c["extprice"], 24, residual_loc=1)):
        assert run_minmax(cu, cols, los, his, ep, mode) == expect(vals, cols, los, his, c["extprice"], ep, mode)


@pytest.mark.parametrize("mode", ["min", "max"])
def test_gpu_minmax_signed_for_base(cu, mode):
    # signed Y (int32 longitudes of the spatial workload) with a frame-of-reference base
    n = 100_001
    s = datagen.spatial_columns(8, n)
    x = datagen.uniform_u32(9, n, 0, 999)
    xc = cu.BWDColumn(x, 28)
    yc = cu.BWDColumn(s["lon"], 24, signed=True, base="min")
    got = run_minmax(cu, [xc], [100], [350], yc, mode)
    assert got == expect([x], [xc], [100], [350], np.asarray(s["lon"], dtype=np.int32), yc, mode, y_signed=True)


@pytest.mark.parametrize("mode", ["min", "max"])
@pytest.mark.parametrize("n", [4097, 300_001])
def test_gpu_minmax_signed_predicates(cu, mode, n):
    # the spatial query's signed lon / lat predicates (FOR base, 24/8) select the rows; MIN / MAX of a
    # third column and of the signed lon itself (its major carried in the approximation tuple)
    s = datagen.spatial_columns(14, n)
    lon, lat = np.asarray(s["lon"], dtype=np.int32), np.asarray(s["lat"], dtype=np.int32)
    pcols = [cu.BWDColumn(lon, 24, signed=True, base="min"), cu.BWDColumn(lat, 24, signed=True, base="min")]
    y = datagen.uniform_u32(15, n)
    yc = cu.BWDColumn(y, 20)
    # Table I's box, and a box whose longitude range crosses zero (negative lower bound)
    for los, his in (([datagen.SPATIAL_LON[0], datagen.SPATIAL_LAT[0]], [datagen.SPATIAL_LON[1], datagen.SPATIAL_LAT[1]]),
                     ([-900_000, 4_000_000], [600_000, 6_000_000])):
        got = run_minmax(cu, pcols, los, his, yc, mode)
        assert got == expect([lon, lat], pcols, los, his, y, yc, mode, pred_signed=[True, True])
        assert got[1] > 0
        got = run_minmax(cu, pcols, los, his, pcols[0], mode)
        assert got == expect([lon, lat], pcols, los, his, lon, pcols[0], mode, y_signed=True,
                             pred_signed=[True, True])


def test_gpu_minmax_empty_and_all(cu):
    n = 5000
    x = datagen.uniform_u32(3, n, 0, 1000)
    y = datagen.uniform_u32(4, n)
    xc, yc = cu.BWDColumn(x, 28), cu.BWDColumn(y, 24)
    assert run_minmax(cu, [xc], [2000], [3000], yc, "min") == [0] * 7
    got = run_minmax(cu, [xc], [0], [0xFFFFFFFF], yc, "max")   # every row, all definite
    assert got[0] == int(y.max()) and got[1] >= 1 and got[5] == got[6] == n
    assert got == expect([x], [xc], [0], [0xFFFFFFFF], y, yc, "max")


def test_gpu_minmax_c2_full(cu):
    # C2 (SF10, 60 M rows): MIN / MAX(l_extendedprice) under Q6
    c = datagen.q6_columns(2, 10)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    cols = [cu.BWDColumn(vals[0], 24), cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)]
    ep = cu.BWDColumn(c["extprice"], 32, layout=1)
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    for mode in ("min", "max"):
        assert run_minmax(cu, cols, los, his, ep, mode) == expect(vals, cols, los, his, c["extprice"], ep, mode)
