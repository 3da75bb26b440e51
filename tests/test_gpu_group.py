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
