"""GPU parity: every C-ABI call vs the CPU oracle, bit-exact (positions, definite
flags, approximation words, counts, int64 sums).  Runs on a B200 (sm_100a)."""
import numpy as np
import pytest

import datagen
import oracle
from tests._layout import unpack_packed, unpack_sliced

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def _col(cu, v, major_bits, layout=0, loc=0, base=0):
    return cu.BWDColumn(np.ascontiguousarray(v, dtype=np.uint32), major_bits, layout=layout, residual_loc=loc,
                        base=base)


def _bytes(t):
    return t.cpu().numpy().tobytes()


def _residual(c, n):
    """Decode a column's residual part per its layout (ar.h: SLICED for k <= 8, else PACKED)."""
    dec = unpack_sliced if c.desc.residual_layout == 0 else unpack_packed
    return dec(_bytes(c.residual), n, c.k)


# ----------------------------------------------------------------- a1 decompose

def test_gpu_decompose_fig2(cu, golden):
    g = golden("fig2_decomposition.txt")
    v = np.array([int(g["value"])], dtype=np.uint32)
    k = int(g["cpu_bits"])
    c = _col(cu, v, 32 - k)
    assert c.w_major == int(g["gpu_bits"]) and c.k == k
    assert int(unpack_sliced(_bytes(c.major), 1, c.w_major)[0]) == int(g["major_bits_string"], 2)
    assert c.desc.residual_layout == 0                 # k = 7 <= 8: bit-sliced residual planes
    assert int(_residual(c, 1)[0]) == int(g["residual_bits_string"], 2)


@pytest.mark.parametrize("n", [0, 1, 31, 32, 33, 127, 128, 129, 4095, 4096, 4097, 2**20 - 1, 2**20 + 1])
@pytest.mark.parametrize("major_bits", [8, 24, 32, 1])
@pytest.mark.parametrize("layout", [0, 1])
def test_gpu_decompose_matches_oracle(cu, n, major_bits, layout):
    v = datagen.uniform_u32(1000 + n, n)
    c = _col(cu, v, major_bits, layout)
    major, residual, w = oracle.decompose(v, 32 - major_bits)
    assert c.w_major == w and c.k == 32 - major_bits
    dec = unpack_sliced if layout == 0 else unpack_packed
    got_major = dec(_bytes(c.major), n, w)
    assert np.array_equal(got_major, major.astype(np.uint64))
    if c.k:
        assert c.desc.residual_layout == (0 if c.k <= 8 else 1)
        assert np.array_equal(_residual(c, n), residual.astype(np.uint64))
    if layout == 0 and n % 128:
        # padding rows of the last 128-row group are zero planes
        words = np.frombuffer(_bytes(c.major), dtype="<u4")
        tail_blocks = words[((n + 31) // 32) * w:]
        assert not tail_blocks.any()


def test_gpu_decompose_base(cu):
    v = np.array([1000, 1001, 1255, 1256, 5000], dtype=np.uint32)
    c = _col(cu, v, 24, base=1000)
    major, residual, w = oracle.decompose(v, 8, base=1000)
    assert c.w_major == w
    assert np.array_equal(unpack_sliced(_bytes(c.major), 5, w), major.astype(np.uint64))
    assert np.array_equal(_residual(c, 5), residual.astype(np.uint64))


# ------------------------------------------------------------ a2+a3 approx select

def run_select(cu, cols, los, his, carry=True):
    n = cols[0].n
    cands = cu.CandidateList(n)
    ws = cu.Workspace(__import__("paper_conf_icde_pirkmk14_b200")._ar.ar_select_ws_bytes(n))
    cu.approx_select(list(zip(cols, los, his)), cands, ws, carry=carry)
    torch.cuda.synchronize()
    return cands


def check_select(cu, values, ks, los, his, carry=True):
    cols = [_col(cu, v, 32 - k) for v, k in zip(values, ks)]
    cands = run_select(cu, cols, los, his, carry)
    ref_pos, ref_def = oracle.approx_select(values, ks, los, his)
    got = cands.positions()
    assert cands.count() == ref_pos.size
    assert np.array_equal(got, ref_pos)
    assert np.array_equal(cands.definite(), ref_def)
    if carry and ref_pos.size:
        aux = cands.aux_words().astype(np.uint64)
        shift = 0
        for v, k, c in zip(values, ks, cols):
            major, _, w = oracle.decompose(v, k)
            got_m = (aux >> np.uint64(shift)) & np.uint64((1 << w) - 1)
            assert np.array_equal(got_m, major[ref_pos].astype(np.uint64))
            shift += w
    return cols, cands


def test_gpu_select_c1(cu):
    # config C1: 1M uniform u32, 24/8 split, 1 % range with an unaligned lower bound
    v = datagen.uniform_u32(1, datagen.C1_N)
    check_select(cu, [v], [8], [datagen.C1_LO], [datagen.C1_HI])


@pytest.mark.parametrize("n", [1, 31, 32, 33, 4095, 4096, 4097, 8192 * 3 + 5, 2**20 - 1, 2**20 + 1])
def test_gpu_select_ragged(cu, n):
    v = datagen.uniform_u32(7 + n, n, 0, 4095)
    check_select(cu, [v], [4], [700], [2900])


@pytest.mark.parametrize("k", [0, 1, 7, 8, 16, 24, 31])
def test_gpu_select_widths(cu, k):
    n = 300_001
    v = datagen.uniform_u32(50 + k, n)
    lo = 0x31234567
    check_select(cu, [v], [k], [lo], [lo + 0x10000000], carry=(32 - k) <= 31)


def test_gpu_select_edge_ranges(cu):
    n = 100_000
    v = datagen.uniform_u32(3, n, 0, 2**20)
    for lo, hi in [(0, 2**32 - 1), (500, 400), (0, 0), (2**20, 2**20), (2**32 - 1, 2**32 - 1),
                   (2**21, 2**31), (256, 511), (255, 512)]:
        check_select(cu, [v], [8], [lo], [hi])


def test_gpu_select_all_and_none(cu):
    n = 50_000
    v = np.full(n, 1234, dtype=np.uint32)
    cols, cands = check_select(cu, [v], [4], [1234], [1234])
    assert cands.count() == n
    # 1234 = 77 * 16 + 2: bucket [1232, 1247] meets [0, 1233] -> every row a candidate, none definite
    cols, cands = check_select(cu, [v], [4], [0], [1233])
    assert cands.count() == n and not cands.definite().any()
    cols, cands = check_select(cu, [v], [4], [0], [1231])
    assert cands.count() == 0


def test_gpu_select_conjunction_q6(cu):
    c = datagen.q6_columns(2, 0.5)                       # 3 M rows, Q6-shaped
    values = [c["shipdate"], c["discount"], c["quantity"]]
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    check_select(cu, values, [8, 0, 0], los, his)
    check_select(cu, values, [8, 0, 0], los, his, carry=False)


def test_gpu_select_base(cu):
    v = datagen.uniform_u32(4, 70_000, 10_000, 20_000)
    col = _col(cu, v, 24, base=10_000)
    cands = run_select(cu, [col], [12_345], [17_000])
    # with base b, buckets are [b + m 2^k, ...]: oracle on u = v - b with bounds shifted
    ref_pos, ref_def = oracle.approx_select([v - 10_000], [8], [2_345], [7_000])
    assert np.array_equal(cands.positions(), ref_pos) and np.array_equal(cands.definite(), ref_def)


# ------------------------------------------------------------------- a5 refine

def check_refine_and_sums(cu, values, ks, los, his, agg_values, agg_layouts, carry=True, loc=0, agg_ks=None,
                          agg_loc=0):
    from paper_conf_icde_pirkmk14_b200 import _ar
    cols = [_col(cu, v, 32 - k, loc=loc) for v, k in zip(values, ks)]
    n = cols[0].n
    cands = run_select(cu, cols, los, his, carry)
    preds = list(zip(cols, los, his))
    out = cu.PositionList(n)
    ws = cu.Workspace(_ar.ar_refine_ws_bytes(n))
    cu.refine(cands, preds, out, ws)
    torch.cuda.synchronize()
    ref_pos, ref_cnt, _ = oracle.select_sum(values, los, his)
    assert out.count() == ref_cnt
    assert np.array_equal(out.positions(), ref_pos)
    # aggregate columns: reuse a predicate column object when it is the same data
    aggs, aks = [], []
    agg_ks = agg_ks or [0] * len(agg_values)
    for av, lay, ak in zip(agg_values, agg_layouts, agg_ks):
        same = [(c, k) for c, v, k in zip(cols, values, ks) if v is av]
        aggs.append(same[0][0] if same else _col(cu, av, 32 - ak, layout=lay, loc=agg_loc))
        aks.append(same[0][1] if same else ak)
    ref_sum = oracle.sum_at(ref_pos, agg_values)
    s = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.sum_at(out, aggs, s)
    s2 = torch.zeros(1, dtype=torch.int64, device="cuda")
    c2 = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, aggs, s2, c2)
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, aggs, o4)
    torch.cuda.synchronize()
    assert int(s.item()) == ref_sum
    assert int(s2.item()) == ref_sum and int(c2.item()) == ref_cnt
    cpos, cdef = oracle.approx_select(values, ks, los, his)
    assert o4.cpu().tolist() == [ref_sum, ref_cnt, cpos.size, int(cdef.sum())]
    # bwd.sumapproximate: bounds from the candidates and the majors only
    b4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.sum_approximate(cands, aggs, b4)
    torch.cuda.synchronize()
    ref_b = oracle.sum_bounds(values, ks, los, his, agg_values, aks)
    assert tuple(b4.cpu().tolist()) == ref_b
    assert ref_b[0] <= ref_sum <= ref_b[1] and ref_b[2] <= ref_cnt <= ref_b[3]
    return ref_cnt, ref_sum


def test_gpu_refine_c1(cu):
    v = datagen.uniform_u32(1, datagen.C1_N)
    check_refine_and_sums(cu, [v], [8], [datagen.C1_LO], [datagen.C1_HI], [v], [1])


@pytest.mark.parametrize("k", [1, 8, 16, 24])
def test_gpu_refine_many_boundary_rows(cu, k):
    # narrow value domain so that many rows fall in the two boundary buckets
    n = 400_003
    v = datagen.uniform_u32(80 + k, n, 0, (1 << (k + 3)) - 1)
    lo, hi = (1 << k) + 3, 5 * (1 << k) - 2
    check_refine_and_sums(cu, [v], [k], [lo], [hi], [v], [1])
    check_refine_and_sums(cu, [v], [k], [lo], [hi], [v], [1], carry=False)


def test_gpu_q6_small(cu):
    c = datagen.q6_columns(2, 0.5)
    values = [c["shipdate"], c["discount"], c["quantity"]]
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    cnt, s = check_refine_and_sums(cu, values, [8, 0, 0], los, his, [c["extprice"], c["discount"]], [1, 0])
    assert cnt > 0 and s > 0


def test_gpu_q6_host_pinned_residual(cu):
    c = datagen.q6_columns(5, 0.2)
    values = [c["shipdate"], c["discount"], c["quantity"]]
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    check_refine_and_sums(cu, values, [8, 0, 0], los, his, [c["extprice"], c["discount"]], [1, 0], loc=1)


@pytest.mark.parametrize("agg_loc", [0, 1])
@pytest.mark.parametrize("ep_k", [4, 8, 12])
def test_gpu_q6_decomposed_extprice(cu, ep_k, agg_loc):
    # the aggregate column itself is decomposed (residual in HBM or pinned host
    # memory); SUM(refine) rebuilds ((major << k) | residual) before multiplying
    c = datagen.q6_columns(12, 0.3)
    values = [c["shipdate"], c["discount"], c["quantity"]]
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    for lay in (0, 1):
        check_refine_and_sums(cu, values, [8, 0, 0], los, his, [c["extprice"], c["discount"]], [lay, 0],
                              agg_ks=[ep_k, 0], agg_loc=agg_loc)


def test_gpu_sum_approximate_edges(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.uniform_u32(21, 50_001)
    col = _col(cu, v, 24)
    # empty candidate relation: all bounds 0
    cands = run_select(cu, [col], [10], [5])
    b4 = torch.full((4,), -1, dtype=torch.int64, device="cuda")
    cu.sum_approximate(cands, [col], b4)
    torch.cuda.synchronize()
    assert b4.cpu().tolist() == [0, 0, 0, 0]
    # COUNT only (ncols = 0)
    cands = run_select(cu, [col], [datagen.C1_LO], [datagen.C1_HI])
    cu.sum_approximate(cands, [], b4)
    torch.cuda.synchronize()
    pos, dfn = oracle.approx_select([v], [8], [datagen.C1_LO], [datagen.C1_HI])
    assert b4.cpu().tolist() == [0, 0, int(dfn.sum()), pos.size]
    with pytest.raises(_ar.ARError):
        cu.sum_approximate(cands, [col, col, col], b4)


@pytest.mark.parametrize("k,loc,lay", [(0, 0, 1), (8, 0, 0), (8, 1, 1), (12, 0, 1), (20, 1, 0)])
def test_gpu_project(cu, k, loc, lay):
    # positional projection of the exact value (leftjoinrefine) and of the approximation
    # (leftjoinapproximate) at candidate and at refined positions
    v = datagen.uniform_u32(30 + k, 200_003, 1_000, 2**31)
    base = 1_000 if k == 12 else 0
    col = cu.BWDColumn(v, 32 - k, layout=lay, residual_loc=loc, base=base)
    sel = _col(cu, v, 24)
    lo, hi = 2**30, 2**30 + 2**27
    cands = run_select(cu, [sel], [lo], [hi])
    n = cands.count()
    ex = cu.project(cands, col, exact=True)
    ap = cu.project(cands, col, exact=False)
    torch.cuda.synchronize()
    pos = cands.positions()
    assert n > 1000
    assert np.array_equal(ex[:n].cpu().numpy().view(np.uint32), v[pos])
    major, _, _ = oracle.decompose(v, k, base)
    want = ((major[pos].astype(np.uint64) << k) + base).astype(np.uint32)
    assert np.array_equal(ap[:n].cpu().numpy().view(np.uint32), want)
    out = cu.PositionList(sel.n)
    from paper_conf_icde_pirkmk14_b200 import _ar
    cu.refine(cands, [(sel, lo, hi)], out, cu.Workspace(_ar.ar_refine_ws_bytes(sel.n)))
    ex2 = cu.project(out, col, exact=True)
    torch.cuda.synchronize()
    m = out.count()
    assert np.array_equal(ex2[:m].cpu().numpy().view(np.uint32), v[out.positions()])


def test_gpu_sum_closed_form(cu):
    n = 123_457
    ep = np.arange(1, n + 1, dtype=np.uint32)
    col = _col(cu, ep, 32, layout=1)
    scol = _col(cu, ep, 24)
    from paper_conf_icde_pirkmk14_b200 import _ar
    cands = run_select(cu, [scol], [0], [2**32 - 1])
    pos = cu.PositionList(n)
    cu.refine(cands, [(scol, 0, 2**32 - 1)], pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    s = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.sum_at(pos, [col], s)
    torch.cuda.synchronize()
    assert int(s.item()) == n * (n + 1) // 2


def test_gpu_errors(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.uniform_u32(9, 1000)
    a = _col(cu, v, 24)
    b = _col(cu, v[:999], 24)
    cands = cu.CandidateList(1000)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(1000))
    with pytest.raises(_ar.ARError) as e:
        cu.approx_select([(a, 0, 10), (b, 0, 10)], cands, ws)
    assert e.value.status == _ar.AR_ERR_INVALID
    small = cu.CandidateList(10)
    with pytest.raises(_ar.ARError) as e:
        cu.approx_select([(a, 0, 10)], small, ws)
    assert e.value.status == _ar.AR_ERR_RANGE
    packed = _col(cu, v, 24, layout=1)
    with pytest.raises(_ar.ARError) as e:
        cu.approx_select([(packed, 0, 10)], cands, ws)
    assert e.value.status == _ar.AR_ERR_INVALID
    big = _col(cu, np.full(10, 2**32 - 1, dtype=np.uint32), 32, layout=1)
    s = torch.zeros(1, dtype=torch.int64, device="cuda")
    with pytest.raises(_ar.ARError) as e:
        cu.sum_at(cu.PositionList(10), [big, big], s)
    assert e.value.status == _ar.AR_ERR_RANGE


def test_gpu_wrap_rejects_short_or_misaligned_buffers(cu):
    # a descriptor promising fewer bytes than its geometry, or a part buffer that is not 16-B
    # aligned, is refused at wrap time instead of faulting inside a TMA copy later
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.uniform_u32(10, 5000)
    a = _col(cu, v, 24)
    d = _ar.ar_column_get_desc(a.handle)
    maj, res = a.major.data_ptr(), a.residual.data_ptr()
    h = _ar.ar_column_wrap(d, maj, res)
    _ar.ar_column_free(h)
    for field in ("major_bytes", "residual_bytes"):
        short = _ar.ar_column_get_desc(a.handle)
        setattr(short, field, getattr(short, field) - 16)
        with pytest.raises(_ar.ARError) as e:
            _ar.ar_column_wrap(short, maj, res)
        assert e.value.status == _ar.AR_ERR_RANGE
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_column_wrap(d, maj + 4, res)
    assert e.value.status == _ar.AR_ERR_INVALID
    with pytest.raises(_ar.ARError) as e:
        _ar.ar_column_wrap(d, maj, res + 8)
    assert e.value.status == _ar.AR_ERR_INVALID


def test_gpu_refine_cooperative_launch(cu):
    # ar_refine's look-back needs every CTA resident: it is launched cooperatively and sized from
    # this device's occupancy; a large candidate list (many tiles per CTA) still refines exactly
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 3_000_017
    v = datagen.uniform_u32(12, n)
    col = _col(cu, v, 24)
    lo, hi = 0x10000000, 0xB0000000
    cands = cu.CandidateList(n)
    cu.approx_select([(col, lo, hi)], cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    pos = cu.PositionList(n)
    cu.refine(cands, [(col, lo, hi)], pos, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    torch.cuda.synchronize()
    ref, cnt, _ = oracle.select_sum([v], [lo], [hi])
    assert pos.count() == cnt and np.array_equal(pos.positions(), ref)
