"""Pins for oracle.sum_bounds (bwd.sumapproximate, Fig. 7 PAPER.md:884-889;
strict error bounds of the approximate answer).

The pins do not re-type the bucket formula: the brute force enumerates every
residual a decomposed value could carry, the k = 0 case must collapse to the
exact answer of the (independently pinned) exact select, and the exact answer
must lie inside the bounds on Q6-shaped data."""
import numpy as np
import pytest

import datagen
import oracle


def _brute(pred_cols, pks, los, his, agg_cols, aks):
    """Per row, enumerate the 2^k values the approximation stands for (the
    major bits kept, every residual): candidate iff some value satisfies the
    predicate, definite iff all do; the aggregate factor ranges over the same
    enumerated values, so its bounds are their min and max (base 0)."""
    n = len(pred_cols[0])
    slo = shi = ndef = ncand = 0
    for i in range(n):
        cand = dfn = True
        for c, k, lo, hi in zip(pred_cols, pks, los, his):
            keep = int(c[i]) >> k << k
            vals = [keep + r for r in range(1 << k)]
            hits = [lo <= v <= hi for v in vals]
            cand &= any(hits)
            dfn &= all(hits)
        if not cand:
            continue
        ncand += 1
        ndef += dfn
        if not agg_cols:
            continue
        plo = phi = 1
        for a, k in zip(agg_cols, aks):
            keep = int(a[i]) >> k << k
            vals = [min(keep + r, 2**32 - 1) for r in range(1 << k)]
            plo *= min(vals)
            phi *= max(vals)
        shi += phi
        if dfn:
            slo += plo
    return slo, shi, ndef, ncand


@pytest.mark.parametrize("seed", range(10))
def test_sum_bounds_bruteforce_tiny(seed):
    rng = np.random.default_rng(100 + seed)
    n = int(rng.integers(0, 40))
    npred = int(rng.integers(1, 3))
    nagg = int(rng.integers(0, 3))
    dom = int(rng.choice([16, 300, 4096]))
    pc = [rng.integers(0, dom, n).astype(np.uint32) for _ in range(npred)]
    pks = [int(rng.integers(0, 5)) for _ in range(npred)]
    ac = [rng.integers(0, 5000, n).astype(np.uint32) for _ in range(nagg)]
    aks = [int(rng.integers(0, 6)) for _ in range(nagg)]
    los, his = [], []
    for _ in range(npred):
        lo, hi = sorted(rng.integers(0, dom, 2).tolist())
        los.append(lo)
        his.append(hi)
    got = oracle.sum_bounds(pc, pks, los, his, ac, aks)
    assert got == _brute(pc, pks, los, his, ac, aks)


def test_sum_bounds_top_bucket_clamped():
    # the bucket of 2^32 - 1 at k = 4 is [2^32 - 16, 2^32 - 1]: no value beyond 2^32 - 1
    v = np.array([2**32 - 1, 2**32 - 16], dtype=np.uint32)
    got = oracle.sum_bounds([v], [0], [0], [2**32 - 1], [v], [4])
    assert got == (2 * (2**32 - 16), 2 * (2**32 - 1), 2, 2) == _brute([v], [0], [0], [2**32 - 1], [v], [4])


def test_sum_bounds_k0_is_exact():
    # with nothing decomposed the approximation is the data: both bounds equal the exact SUM
    c = datagen.q6_columns(7, 0.05)
    sd, disc, qty, ep = c["shipdate"], c["discount"], c["quantity"], c["extprice"]
    los, his = [731, 5, 0], [1095, 7, 23]
    _, cnt, s = oracle.select_sum([sd, disc, qty], los, his, [ep, disc], positions=False)
    got = oracle.sum_bounds([sd, disc, qty], [0, 0, 0], los, his, [ep, disc], [0, 0])
    assert got == (s, s, cnt, cnt)


@pytest.mark.parametrize("ep_k", [0, 8, 12])
def test_sum_bounds_contain_exact_q6(ep_k):
    c = datagen.q6_columns(8, 0.05)
    sd, disc, qty, ep = c["shipdate"], c["discount"], c["quantity"], c["extprice"]
    los, his = [731, 5, 0], [1095, 7, 23]
    _, cnt, s = oracle.select_sum([sd, disc, qty], los, his, [ep, disc], positions=False)
    slo, shi, clo, chi = oracle.sum_bounds([sd, disc, qty], [8, 0, 0], los, his, [ep, disc], [ep_k, 0])
    assert clo <= cnt <= chi and slo <= s <= shi
    # count bounds are the approximate selection's definite / candidate counts
    pos, dfn = oracle.approx_select([sd, disc, qty], [8, 0, 0], los, his)
    assert (clo, chi) == (int(dfn.sum()), len(pos))
    if ep_k == 0:
        # undecomposed ep: the lower bound is the exact SUM over the definite rows
        assert slo == oracle.sum_at(pos[dfn], [ep, disc])


def test_sum_bounds_closed_form_constant():
    # ep == c (decomposed k), disc == d, one predicate that keeps every row definitely:
    # bounds = n d (c >> k << k)  and  n d ((c >> k << k) + 2^k - 1)
    n, c, d, k = 5000, 1_234_567, 3, 8
    ep = np.full(n, c, dtype=np.uint32)
    disc = np.full(n, d, dtype=np.uint32)
    keep = np.zeros(n, dtype=np.uint32)
    got = oracle.sum_bounds([keep], [0], [0], [0], [ep, disc], [k, 0])
    lo = (c >> k) << k
    assert got == (n * d * lo, n * d * (lo + 2**k - 1), n, n)
