"""Pins for the approximate-select intermediates of the oracle
(relaxation PAPER.md:615-632 s IV-B; superset PAPER.md:372-374; Fig. 4, Fig. 6)."""
import numpy as np
import pytest

import oracle
from tests.conftest import read_golden


def test_relax_fig4():
    g = read_golden("fig4_integrated_example.txt")
    k = int(g["k"])
    A = np.array([int(x) for x in g["A"].split(",")], dtype=np.uint32)
    major, residual, _ = oracle.decompose(A, k)
    # A < 5  ==  0 <= A <= 4
    cand, dfn = oracle.bucket_flags(major, k, 0, 4)
    ids = [i + 1 for i in np.nonzero(cand)[0].tolist()]
    assert ids == [int(x) for x in g["candidate_ids"].split(",")]
    approx = (major.astype(np.int64) << k)[cand]                 # "Approx A" in value units
    assert approx.tolist() == [int(x) for x in g["candidate_approx"].split(",")]
    assert int(approx.max()) == int(g["approx_bound"])            # "Approx A <= 4"
    assert not dfn.any()                                          # both need refinement
    pos, cnt, _ = oracle.select_sum([A], [0], [4])
    assert [p + 1 for p in pos.tolist()] == [int(x) for x in g["refined_ids"].split(",")]
    assert A[pos].tolist() == [int(g["refined_A"])]


def test_relax_fig6():
    g = read_golden("fig6_minmax.txt")
    k = int(g["k"])
    # x > 6  ==  7 <= x <= 2^32-1 ; the approximate condition is x >= 4 (value units)
    majors = np.arange(0, 64, dtype=np.uint32)
    cand, _ = oracle.bucket_flags(majors, k, 7, 2**32 - 1)
    approx_values = (majors.astype(np.int64) << k)[cand]
    assert int(approx_values.min()) == 4
    assert np.all(approx_values >= 4) and cand[1:].all() and not cand[0]


def _brute(m, k, lo, hi):
    vals = [(m << k) | r for r in range(1 << k)]
    inside = [lo <= v <= hi for v in vals]
    return any(inside), all(inside)


@pytest.mark.parametrize("k", list(range(0, 9)))
def test_relax_bruteforce_small_domain(k):
    # cand <=> exists r < 2^k with (m<<k | r) in [lo,hi];  def <=> for all r
    rng = np.random.default_rng(7 + k)
    dom = 1 << (k + 4)
    for _ in range(60):
        lo, hi = sorted(rng.integers(0, dom, 2).tolist())
        if rng.random() < 0.1:
            lo, hi = hi + 1, lo            # empty range
        majors = np.arange(0, 1 << 4, dtype=np.uint32)
        cand, dfn = oracle.bucket_flags(majors, k, lo, hi)
        for m in range(1 << 4):
            c, d = _brute(m, k, lo, hi)
            assert cand[m] == c and dfn[m] == d, (m, k, lo, hi)


@pytest.mark.parametrize("k", [1, 4, 8])
def test_relax_bruteforce_top_of_domain(k):
    # buckets touching 2^32-1 (no 32-bit overflow in the bucket arithmetic)
    top = (1 << (32 - k)) - 1
    majors = np.array([top - 2, top - 1, top], dtype=np.uint32)
    for lo, hi in [(2**32 - 1, 2**32 - 1), (2**32 - 3, 2**32 - 1), (0, 2**32 - 1), (2**32 - 300, 2**32 - 2)]:
        cand, dfn = oracle.bucket_flags(majors, k, lo, hi)
        for i, m in enumerate(majors.tolist()):
            c, d = _brute(m, k, lo, hi)
            assert cand[i] == c and dfn[i] == d


def test_relax_paper_f_superset():
    # printed f(x) ('<<' restored) is a superset of the tight
    # rule, which is a superset of the exact result: exhaustive on a 6-bit domain
    v = np.arange(0, 64, dtype=np.uint32)
    looser = 0
    for k in range(0, 7):
        major, _, _ = oracle.decompose(v, k)
        for op in ["==", ">", ">=", "<", "<="]:
            for x in range(0, 64):
                exact = {"==": v == x, ">": v > x, ">=": v >= x, "<": v < x, "<=": v <= x}[op]
                lo, hi = {"==": (x, x), ">": (x + 1, 2**32 - 1), ">=": (x, 2**32 - 1),
                          "<": (0, x - 1), "<=": (0, x)}[op]
                if hi < lo or lo > 2**32 - 1:
                    tight = np.zeros(64, dtype=bool)
                else:
                    tight, dfn = oracle.bucket_flags(major, k, lo, hi)
                    assert not (dfn & ~exact).any()                # definite hits are hits
                paper = oracle.paper_f_flags(v, k, op, x)
                assert not (exact & ~tight).any(), (k, op, x)     # tight is a superset
                assert not (tight & ~paper).any(), (k, op, x)     # printed f is looser still
                looser += int((paper & ~tight).any())
    assert looser > 0          # the printed '<' and '<=' admit an extra bucket


def test_approx_select_superset_and_definite():
    rng = np.random.default_rng(11)
    a = rng.integers(0, 2**32, 20000, dtype=np.uint64).astype(np.uint32)
    b = rng.integers(0, 4096, 20000).astype(np.uint32)
    los, his = [0x40000000, 700], [0x4FFFFFFF, 1900]
    for ks in [(8, 4), (16, 0), (0, 8), (24, 11)]:
        cpos, cdef = oracle.approx_select([a, b], list(ks), los, his)
        exact, _, _ = oracle.select_sum([a, b], los, his)
        assert set(exact.tolist()) <= set(cpos.tolist())          # superset
        assert set(cpos[cdef].tolist()) <= set(exact.tolist())    # definite => hit
        # refine(approx) == exact: re-evaluate the exact predicate at candidates
        keep = cpos[(a[cpos] >= los[0]) & (a[cpos] <= his[0]) & (b[cpos] >= los[1]) & (b[cpos] <= his[1])]
        assert keep.tolist() == exact.tolist()


def test_approx_select_k0_is_exact():
    rng = np.random.default_rng(12)
    a = rng.integers(0, 1000, 5000).astype(np.uint32)
    cpos, cdef = oracle.approx_select([a], [0], [100], [350])
    exact, _, _ = oracle.select_sum([a], [100], [350])
    assert cpos.tolist() == exact.tolist() and cdef.all()


def test_approx_select_full_range_all_definite():
    a = np.random.default_rng(13).integers(0, 2**32, 3000, dtype=np.uint64).astype(np.uint32)
    for k in [0, 1, 8, 31, 32]:
        cpos, cdef = oracle.approx_select([a], [k], [0], [2**32 - 1])
        assert cpos.size == a.size and cdef.all()
