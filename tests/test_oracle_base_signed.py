"""Pins of the oracle's prefix-base (b != 0) and signed-key branches.

The frame-of-reference base ("base" kept with the column;
PAPER.md:1172-1177 factoring out the high bytes of the spatial coordinates)
and the signed key domain d = v ^ 2^31 (DESIGN R8) are the checker
for the GPU's NEXT-3 / NEXT-4 intermediates, so every branch that uses them is
pinned here against brute force that never evaluates a bucket formula: a value
with stored major m stands for the 2^k values b + (m << k) + r, r < 2^k
(the residual bits are unknown to the approximation), and a
predicate holds "for some" (candidate) or "for all"
(definite) of them.  A dropped base, a wrong sign flip or a signed /
unsigned mix-up fails one of these.  CPU only."""
import random

import numpy as np
import pytest

import oracle

TOP = 2**32 - 1


def _as_signed(key):
    """int32 value of a key-domain word d (v = d ^ 2^31)."""
    v = key ^ 0x80000000
    return v - 2**32 if v >= 2**31 else v


def _bucket_values(m, k, b):
    """Every key a row with major m can hold: b + (m << k) + r, r < 2^k; keys past 2^32 - 1 do not exist."""
    return [b + (m << k) + r for r in range(1 << k) if b + (m << k) + r <= TOP]


def _exists_forall(keys, lo, hi, signed):
    vals = [_as_signed(x) for x in keys] if signed else keys
    inside = [lo <= v <= hi for v in vals]
    # a bucket whose top lies past 2^32 - 1 holds non-values: never "all inside"
    return any(inside), bool(inside) and all(inside)


def _key_bound(x, signed):
    return ((x & 0xFFFFFFFF) ^ 0x80000000) if signed else x


@pytest.mark.parametrize("signed", [False, True])
@pytest.mark.parametrize("k", [0, 1, 3, 5, 8])
def test_bucket_flags_base_bruteforce(k, signed):
    rng = random.Random(1000 * k + signed)
    for _ in range(40):
        b = rng.choice([1, 7, 1 << 20, rng.randrange(0, TOP - (64 << k)), TOP - (16 << k)])
        majors = list(range(16))
        keys_span = [b, b + (16 << k) - 1]
        if signed:
            span = [_as_signed(min(x, TOP)) for x in keys_span]
            a, c = rng.randint(min(span) - 4, max(span) + 4), rng.randint(min(span) - 4, max(span) + 4)
            a, c = (min(max(x, -2**31), 2**31 - 1) for x in (a, c))
            lo, hi = min(a, c), max(a, c)
        else:
            a, c = rng.randint(max(b - 4, 0), min(keys_span[1] + 4, TOP)), rng.randint(max(b - 4, 0), min(keys_span[1] + 4, TOP))
            lo, hi = min(a, c), max(a, c)
        if rng.random() < 0.1 and hi < (2**31 - 1 if signed else TOP):
            lo, hi = hi + 1, lo                                            # empty range
        cand, dfn = oracle.bucket_flags(np.array(majors, dtype=np.uint32), k,
                                        _key_bound(lo, signed), _key_bound(hi, signed), b)
        for m in majors:
            keys = _bucket_values(m, k, b)
            c_want, d_want = _exists_forall(keys, lo, hi, signed) if keys else (False, False)
            if lo > hi:
                c_want = d_want = False
            assert cand[m] == c_want and dfn[m] == d_want, (k, b, m, lo, hi, signed)


@pytest.mark.parametrize("signed", [False, True])
def test_approx_select_base_bruteforce(signed):
    # rows, not majors: decomposition with a base (the oracle's decompose) feeds the flags
    rng = np.random.default_rng(5 + signed)
    for trial in range(30):
        n = int(rng.integers(1, 60))
        k = int(rng.integers(0, 7))
        if signed:
            v = rng.integers(-3000, 3000, n).astype(np.int32)
            keys = (v.view(np.uint32) ^ np.uint32(0x80000000)).astype(np.uint64)
        else:
            v = rng.integers(10**6, 10**6 + 6000, n).astype(np.uint32)
            keys = v.astype(np.uint64)
        b = int(keys.min()) - int(rng.integers(0, 5))                      # base <= min (key domain)
        lo, hi = sorted(int(x) for x in rng.choice(v.astype(np.int64), 2))
        lo -= int(rng.integers(0, 3))
        pos, dfn = oracle.approx_select([v], [k], [lo], [hi], base=[b], signed=[signed])
        want_c, want_d = [], []
        for i in range(n):
            m = (int(keys[i]) - b) >> k
            c, d = _exists_forall(_bucket_values(m, k, b), lo, hi, signed)
            if c:
                want_c.append(i)
                want_d.append(d)
        assert pos.tolist() == want_c and dfn.tolist() == want_d, trial
        # refine(approx) == exact on the signed / based column
        ex, cnt, _ = oracle.select_sum([v], [lo], [hi], signed=[signed])
        keep = [int(p) for p in pos if lo <= int(v[p]) <= hi]
        assert keep == ex.tolist()


def _brute_bounds(pcols, pks, pbases, los, his, psigned, acols, aks, abases):
    slo = shi = nd = nc = 0
    n = len(pcols[0])
    for i in range(n):
        cand = dfn = True
        for c, k, b, lo, hi, sg in zip(pcols, pks, pbases, los, his, psigned):
            key = (int(c[i]) & TOP) ^ (0x80000000 if sg else 0)
            m = (key - b) >> k
            ce, de = _exists_forall(_bucket_values(m, k, b), lo, hi, sg)
            cand &= ce
            dfn &= de
        if not cand:
            continue
        nc += 1
        nd += dfn
        if not acols:
            continue
        plo = phi = 1
        for a, k, b in zip(acols, aks, abases):
            vals = _bucket_values((int(a[i]) - b) >> k, k, b)
            plo *= min(vals)
            phi *= max(vals)
        shi += phi
        if dfn:
            slo += plo
    return slo, shi, nd, nc


@pytest.mark.parametrize("seed", range(16))
def test_sum_bounds_base_signed_bruteforce(seed):
    rng = random.Random(300 + seed)
    n = rng.randint(0, 30)
    npred = rng.randint(1, 2)
    nagg = rng.randint(0, 2)
    pcols, pks, pbases, los, his, psg = [], [], [], [], [], []
    for _ in range(npred):
        sg = rng.random() < 0.5
        k = rng.randint(0, 4)
        if sg:
            vals = [rng.randint(-200, 200) for _ in range(n)]
            col = np.array(vals, dtype=np.int32)
            keys = [(x & TOP) ^ 0x80000000 for x in vals]
            lo, hi = sorted(rng.randint(-220, 220) for _ in range(2))
        else:
            vals = [rng.randint(70000, 70400) for _ in range(n)]
            col = np.array(vals, dtype=np.uint32)
            keys = vals
            lo, hi = sorted(rng.randint(69990, 70410) for _ in range(2))
        b = (min(keys) - rng.randint(0, 9)) if keys else rng.randint(0, 1000)
        pcols.append(col); pks.append(k); pbases.append(b); los.append(lo); his.append(hi); psg.append(sg)
    acols, aks, abases = [], [], []
    for _ in range(nagg):
        vals = [rng.randint(5000, 9000) for _ in range(n)]
        acols.append(np.array(vals, dtype=np.uint32))
        aks.append(rng.randint(0, 5))
        abases.append((min(vals) - rng.randint(0, 50)) if vals else 0)
    if n == 0:
        pcols = [np.zeros(0, dtype=np.int32 if s else np.uint32) for s in psg]
    got = oracle.sum_bounds(pcols, pks, los, his, acols, aks, pred_bases=pbases, agg_bases=abases,
                            pred_signed=psg)
    assert got == _brute_bounds(pcols, pks, pbases, los, his, psg, acols, aks, abases)


def _in_r(pcols, los, his, i):
    return all(lo <= int(c[i]) <= hi for c, lo, hi in zip(pcols, los, his))


@pytest.mark.parametrize("seed", range(24))
def test_minmax_ar_base_signed_bruteforce(seed):
    """s IV-F with bases and signed predicate / Y columns: the refined answer is the exact one, the
    approximate bounds contain it, and the refined set is exactly the candidates whose Y bucket can
    hold the answer (Y major <= the smallest Y major over definite candidates for MIN, >= the largest
    for MAX; every candidate without a definite one) -- candidate / definite by brute force."""
    rng = random.Random(900 + seed)
    n = rng.randint(0, 14)
    npred = rng.randint(1, 2)
    pcols, pks, pbases, los, his, psg = [], [], [], [], [], []
    for _ in range(npred):
        sg = rng.random() < 0.5
        vals = [rng.randint(-40, 40) if sg else rng.randint(5000, 5080) for _ in range(n)]
        col = np.array(vals, dtype=np.int32 if sg else np.uint32)
        keys = [((x & TOP) ^ 0x80000000) if sg else x for x in vals]
        lo, hi = sorted((rng.randint(-45, 45) if sg else rng.randint(4995, 5085)) for _ in range(2))
        pcols.append(col); pks.append(rng.randint(0, 3)); los.append(lo); his.append(hi); psg.append(sg)
        pbases.append((min(keys) - rng.randint(0, 6)) if keys else 0)
    ysg = rng.random() < 0.5
    yv = [rng.randint(-100, 100) if ysg else rng.randint(1000, 1200) for _ in range(n)]
    y = np.array(yv, dtype=np.int32 if ysg else np.uint32)
    ykeys = [((x & TOP) ^ 0x80000000) if ysg else x for x in yv]
    ky = rng.randint(0, 4)
    yb = (min(ykeys) - rng.randint(0, 6)) if ykeys else 0
    for mode in ("min", "max"):
        r = oracle.minmax_ar(pcols, pks, los, his, y, ky, mode, pred_bases=pbases, y_base=yb, y_signed=ysg,
                             flags=True, pred_signed=psg)
        in_r = [_in_r(pcols, los, his, i) for i in range(n)]
        vals = [yv[i] for i in range(n) if in_r[i]]
        want = (min(vals) if mode == "min" else max(vals)) if vals else 0
        assert (r["value"], r["survivors"] > 0) == (want, bool(vals))
        cand, dfn = [], []
        for i in range(n):
            c = d = True
            for col, k, b, lo, hi, sg in zip(pcols, pks, pbases, los, his, psg):
                key = (int(col[i]) & TOP) ^ (0x80000000 if sg else 0)
                ce, de = _exists_forall(_bucket_values((key - b) >> k, k, b), lo, hi, sg)
                c &= ce
                d &= de
            cand.append(c)
            dfn.append(c and d)
        ym = [(ykeys[i] - yb) >> ky for i in range(n)]
        dm = [ym[i] for i in range(n) if dfn[i]]
        want_set = []
        for i in range(n):
            if not cand[i]:
                continue
            if dm and (ym[i] > min(dm) if mode == "min" else ym[i] < max(dm)):
                continue
            want_set.append(i)
        assert list(np.nonzero(r["refine_flags"])[0]) == want_set
        assert (r["candidates"], r["definite"], r["refined"]) == (sum(cand), sum(dfn), len(want_set))
        if vals:
            assert r["lo"] <= want <= r["hi"]
            # the bounds are bucket ends of Y (values of the buckets, by enumeration)
            ends = set()
            for i in range(n):
                if cand[i]:
                    bv = _bucket_values(ym[i], ky, yb)
                    ends.update(_as_signed(x) if ysg else x for x in (bv[0], bv[-1]))
            assert r["lo"] in ends and r["hi"] in ends
