"""GPU parity of ar_refine_group_sum (grouped COUNT / SUM over the refined rows,
PAPER.md:742-778, s IV-E/F) against the oracle, bit-exact per group."""
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


def grouped(cu, pcols, los, his, key, cols, G, carry=True):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = pcols[0].n
    preds = [(c, lo, hi) for c, lo, hi in zip(pcols, los, his)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)), carry=carry)
    out = cu.refine_group_sum(cands, preds, key, cols, G)
    torch.cuda.synchronize()
    return out.cpu().numpy()


def test_gpu_group_fig4(cu, golden):
    g = golden("fig4_groupby.txt")
    a = np.array([int(v) for v in g["A"].split(",")], dtype=np.uint32)
    b = np.array([int(v) for v in g["B"].split(",")], dtype=np.uint32)
    ac, bc = cu.BWDColumn(a, 31), cu.BWDColumn(b, 32)      # A: 31 GPU bits + 1 CPU bit; B whole on the GPU
    out = grouped(cu, [ac], [0], [4], bc, [], 8)
    assert list(np.nonzero(out[1])[0]) == [int(g["groups_with_rows"])] and int(out[1].sum()) == int(g["counts"])
    _, cnts = oracle.select_group_sum([a], [0], [4], b, 8)
    assert np.array_equal(out[1], cnts) and not out[0].any()


@pytest.mark.parametrize("sf", [0.01, 0.3])
def test_gpu_group_q6_by_discount(cu, sf):
    # SUM(l_extendedprice), COUNT per l_discount (11 groups) under the shipdate / quantity predicates
    c = datagen.q6_columns(17, sf)
    sd, qt = cu.BWDColumn(c["shipdate"], 24), cu.BWDColumn(c["quantity"], 32)
    dc = cu.BWDColumn(c["discount"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=1)
    los, his = [Q6_LO[0], Q6_LO[2]], [Q6_HI[0], Q6_HI[2]]
    for carry in (True, False):
        out = grouped(cu, [sd, qt], los, his, dc, [ep], 16, carry)
        sums, cnts = oracle.select_group_sum([c["shipdate"], c["quantity"]], los, his, c["discount"], 16,
                                             [c["extprice"]])
        assert np.array_equal(out[0], sums) and np.array_equal(out[1], cnts)


def test_gpu_group_q6_by_quantity_key_is_predicate(cu):
    # group by l_quantity, itself a predicate column (its value comes from the carried approximation);
    # SUM(l_extendedprice * l_discount) with l_extendedprice decomposed 24/8 (residual in pinned host memory)
    c = datagen.q6_columns(19, 0.2)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    cols = [cu.BWDColumn(vals[0], 24), cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)]
    ep = cu.BWDColumn(c["extprice"], 24, residual_loc=1)
    out = grouped(cu, cols, Q6_LO, Q6_HI, cols[2], [ep, cols[1]], 64)
    sums, cnts = oracle.select_group_sum(vals, Q6_LO, Q6_HI, c["quantity"], 64, [c["extprice"], c["discount"]])
    assert np.array_equal(out[0], sums) and np.array_equal(out[1], cnts)
    assert int(cnts.sum()) > 0


@pytest.mark.parametrize("n", [1, 2049, 100_003])
def test_gpu_group_ragged_many_groups(cu, n):
    x = datagen.uniform_u32(5 + n, n)
    key = datagen.uniform_u32(6 + n, n, 0, 4095)
    xc, kc = cu.BWDColumn(x, 20), cu.BWDColumn(key, 32)
    lo, hi = 0x10000000, 0x9fffffff
    out = grouped(cu, [xc], [lo], [hi], kc, [xc], 4096)
    sums, cnts = oracle.select_group_sum([x], [lo], [hi], key, 4096, [x])
    assert np.array_equal(out[0], sums) and np.array_equal(out[1], cnts)


def test_gpu_group_empty_and_errors(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 3000
    x = datagen.uniform_u32(1, n, 0, 100)
    key = datagen.uniform_u32(2, n, 0, 9)
    xc, kc = cu.BWDColumn(x, 28), cu.BWDColumn(key, 32)
    assert not grouped(cu, [xc], [500], [600], kc, [xc], 16).any()
    with pytest.raises(_ar.ARError, match="AR_ERR_RANGE"):       # key values up to 15 need 16 groups
        grouped(cu, [xc], [0], [50], kc, [], 10)
    with pytest.raises(_ar.ARError, match="AR_ERR_UNSUPPORTED"):  # a decomposed key
        grouped(cu, [xc], [0], [50], cu.BWDColumn(key, 30), [], 16)


# ---- the approximation group operator (hash ids) + refinement by ids

def hashed(cu, pcols, los, his, key, cols, G, exact=False, carry=True):
    """approx_select -> ar_group_ids over the candidates -> ar_refine_group_sum_ids; returns the
    (value -> (count, sum)) map of the non-empty groups, the number of ids and the per-row ids."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = pcols[0].n
    preds = [(c, lo & 0xFFFFFFFF, hi & 0xFFFFFFFF) for c, lo, hi in zip(pcols, los, his)]
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)), carry=carry)
    gr = cu.group_ids(cands, key, cu.Grouping(n, G), exact=exact)
    out = cu.refine_group_sum_ids(cands, preds, gr, cols).cpu().numpy()
    torch.cuda.synchronize()
    assert gr.overflow() == 0
    ng = gr.ngroups()
    keys = gr.group_keys()
    ids = gr.gids[:cands.count()].cpu().numpy().view(np.uint32)
    res = {int(keys[g]): (int(out[1, g]), int(out[0, g])) for g in range(ng) if out[1, g] > 0}
    return res, ng, ids, cands


def expect_keys(values, los, his, keyvals, aggs, signed=None):
    k, c, s = oracle.select_group_sum_keys(values, los, his, keyvals, aggs, signed=signed)
    return {int(a): (int(b), int(d)) for a, b, d in zip(k, c, s)}


@pytest.mark.parametrize("n", [1, 4097, 300_001])
def test_gpu_hash_group_sparse_key(cu, n):
    # Q6 predicates, GROUP BY a GPU-resident (k = 0) key whose values are sparse 32-bit numbers (not ids)
    c = datagen.q6_columns(61, 1.0, n=n)
    key = ((c["quantity"].astype(np.uint64) * 2654435761) & 0xFFFFFFFF).astype(np.uint32)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    pcols = [cu.BWDColumn(vals[0], 24), cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)]
    ep = cu.BWDColumn(c["extprice"], 32, layout=1)
    kc = cu.BWDColumn(key, 32, layout=1)
    got, ng, ids, cands = hashed(cu, pcols, Q6_LO, Q6_HI, kc, [ep, pcols[1]], 64)
    assert got == expect_keys(vals, Q6_LO, Q6_HI, key, [c["extprice"], c["discount"]])
    # the ids are a bijection between the candidates' key values and 0 .. ngroups - 1
    ck = key[cands.positions()]
    assert ng == np.unique(ck).size and (ids < ng).all()
    pairs = set(zip(ck.tolist(), ids.tolist()))
    assert len(pairs) == ng and len({a for a, _ in pairs}) == ng and len({b for _, b in pairs}) == ng


def test_gpu_hash_group_false_positive_only_groups(cu):
    # groups that only false positives reach end with count 0 after the refinement
    n = 200_003
    x = datagen.uniform_u32(71, n, 0, 1 << 20)
    key = (x >> 8).astype(np.uint32) * 7919                   # 16 keys per 4096-value bucket of x
    xc = cu.BWDColumn(x, 20)                                   # k = 12: buckets of 4096
    kc = cu.BWDColumn(key, 32)
    lo, hi = 100_000, 700_000                                  # inside the boundary buckets [98304, 102399],
    got, ng, ids, _ = hashed(cu, [xc], [lo], [hi], kc, [], 4096)   # [696320, 700415]: some keys only below lo / above hi
    want = expect_keys([x], [lo], [hi], key, [])
    assert {k: v[0] for k, v in got.items()} == {k: v[0] for k, v in want.items()}
    assert ng > len(want)


@pytest.mark.parametrize("exact", [False, True])
def test_gpu_hash_group_decomposed_key(cu, exact):
    # GROUP BY l_shipdate decomposed 24/8: approximate ids group by bucket (the pre-grouping on
    # approximate values), exact ids by day (the residual read per candidate)
    n = 300_001
    c = datagen.q6_columns(62, 1.0, n=n)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    pcols = [cu.BWDColumn(vals[0], 24), cu.BWDColumn(vals[1], 32), cu.BWDColumn(vals[2], 32)]
    ep = cu.BWDColumn(c["extprice"], 32, layout=1)
    got, ng, _, _ = hashed(cu, pcols, Q6_LO, Q6_HI, pcols[0], [ep, pcols[1]], 1024, exact=exact)
    if exact:
        keyvals = c["shipdate"]
    else:
        major, _, _ = oracle.decompose(c["shipdate"], 8)
        keyvals = (major << 8).astype(np.uint32)               # the bucket minimum (base 0)
    assert got == expect_keys(vals, Q6_LO, Q6_HI, keyvals, [c["extprice"], c["discount"]])
    assert (len(got) > 300) == exact


def test_gpu_hash_group_signed_key(cu):
    # spatial box, GROUP BY the signed latitude's 1e-2-degree cell (decomposed 24/8 with a FOR base):
    # approximate values are bucket minima in the key domain, mapped back to int32
    n = 400_009
    s = datagen.spatial_columns(63, n)
    lon, lat = np.asarray(s["lon"], dtype=np.int32), np.asarray(s["lat"], dtype=np.int32)
    lc = cu.BWDColumn(lon, 24, signed=True, base="min")
    tc = cu.BWDColumn(lat, 24, signed=True, base="min")
    los, his = [-900_000, 5_000_000], [600_000, 5_300_000]
    got, _, _, _ = hashed(cu, [lc, tc], los, his, tc, [], 4096)
    b = int(tc.desc.base)
    kdom = lat.view(np.uint32) ^ np.uint32(0x80000000)
    major, _, _ = oracle.decompose(kdom, 8, b)
    appr = ((major.astype(np.uint64) << 8) + b).astype(np.uint32) ^ np.uint32(0x80000000)
    want = expect_keys([lon, lat], los, his, appr, [], signed=[True, True])
    assert {k: v[0] for k, v in got.items()} == {k: v[0] for k, v in want.items()}


def test_gpu_hash_group_overflow_flag(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 50_000
    x = datagen.uniform_u32(72, n, 0, 999)
    key = datagen.uniform_u32(73, n)                           # ~50 K distinct values
    xc, kc = cu.BWDColumn(x, 32), cu.BWDColumn(key, 32)
    cands = cu.CandidateList(n)
    cu.approx_select([(xc, 0, 999)], cands, cu.Workspace(_ar.ar_select_ws_bytes(n)))
    gr = cu.group_ids(cands, kc, cu.Grouping(n, 64))
    torch.cuda.synchronize()
    assert gr.overflow() & 1 and gr.ngroups() > 64
