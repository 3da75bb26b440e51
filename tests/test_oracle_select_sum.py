"""Pins for oracle.select_sum / sum_at: brute force, closed forms, invariants."""
import numpy as np
import pytest

import oracle


def _brute(pred_cols, los, his, agg_cols):
    n = len(pred_cols[0])
    pos, s = [], 0
    for i in range(n):
        if all(lo <= int(c[i]) <= hi for c, lo, hi in zip(pred_cols, los, his)):
            pos.append(i)
            prod = 1
            for a in agg_cols:
                prod *= int(a[i])
            s += prod if agg_cols else 0
    return pos, s


@pytest.mark.parametrize("seed", range(12))
def test_select_sum_bruteforce_tiny(seed):
    rng = np.random.default_rng(seed)
    n = int(rng.integers(0, 65))
    npred = int(rng.integers(1, 4))
    nagg = int(rng.integers(0, 3))
    dom = int(rng.choice([4, 50, 2**12, 2**32]))
    pc = [rng.integers(0, dom, n, dtype=np.uint64).astype(np.uint32) for _ in range(npred)]
    ac = [rng.integers(0, 2**24, n).astype(np.uint32) for _ in range(nagg)]
    los, his = [], []
    for _ in range(npred):
        lo, hi = sorted(rng.integers(0, dom, 2, dtype=np.uint64).tolist())
        los.append(lo); his.append(hi)
    pos, cnt, s = oracle.select_sum(pc, los, his, ac)
    bpos, bs = _brute(pc, los, his, ac)
    assert pos.tolist() == bpos and cnt == len(bpos) and s == bs


def test_sum_closed_form_constant_columns():
    # ep == c, disc == d  =>  SUM = c * d * |R|
    rng = np.random.default_rng(3)
    n = 100000
    sd = rng.integers(1, 2527, n).astype(np.uint32)
    ep = np.full(n, 10_494_950, dtype=np.uint32)
    disc = np.full(n, 7, dtype=np.uint32)
    _, cnt, s = oracle.select_sum([sd], [731], [1095], [ep, disc], positions=False)
    assert cnt == int(((sd >= 731) & (sd <= 1095)).sum())
    assert s == 10_494_950 * 7 * cnt


def test_sum_closed_form_triangular():
    # ep_i = i + 1 over a predicate that keeps every row  =>  SUM = n (n + 1) / 2
    n = 123457
    ep = np.arange(1, n + 1, dtype=np.uint32)
    _, cnt, s = oracle.select_sum([ep], [0], [2**32 - 1], [ep], positions=False)
    assert cnt == n and s == n * (n + 1) // 2
    # every second row, closed form for the odd numbers 1,3,5,...
    odd = (np.arange(n) % 2).astype(np.uint32)
    _, cnt, s = oracle.select_sum([odd], [0], [0], [ep], positions=False)
    m = (n + 1) // 2
    assert cnt == m and s == m * m


def test_select_empty_and_full():
    a = np.arange(1000, dtype=np.uint32)
    pos, cnt, s = oracle.select_sum([a], [500], [400], [a])        # lo > hi: empty, OK
    assert cnt == 0 and s == 0 and pos.size == 0
    pos, cnt, _ = oracle.select_sum([a], [0], [2**32 - 1])
    assert cnt == 1000 and pos.tolist() == list(range(1000))
    pos, cnt, _ = oracle.select_sum([np.zeros(0, dtype=np.uint32)], [0], [10])
    assert cnt == 0


@pytest.mark.parametrize("threads", [1, 2, 3, 8])
def test_select_sum_thread_invariance(threads):
    rng = np.random.default_rng(5)
    n = 300001
    a = rng.integers(0, 2**32, n, dtype=np.uint64).astype(np.uint32)
    b = rng.integers(0, 50, n).astype(np.uint32)
    ref = oracle.select_sum([a, b], [0x10000000, 3], [0x9FFFFFFF, 30], [b, b], threads=1)
    got = oracle.select_sum([a, b], [0x10000000, 3], [0x9FFFFFFF, 30], [b, b], threads=threads)
    assert got[0].tolist() == ref[0].tolist() and got[1:] == ref[1:]


def test_sum_at_matches_select_sum():
    rng = np.random.default_rng(9)
    a = rng.integers(0, 2**24, 5000).astype(np.uint32)
    b = rng.integers(0, 11, 5000).astype(np.uint32)
    pos, _, s = oracle.select_sum([b], [5], [7], [a, b])
    assert oracle.sum_at(pos, [a, b]) == s
    assert oracle.sum_at(np.zeros(0, dtype=np.int64), [a]) == 0


def test_sum_overflow_detected():
    a = np.full(4, 2**32 - 1, dtype=np.uint32)
    with pytest.raises(OverflowError):
        oracle.select_sum([a], [0], [2**32 - 1], [a, a])


@pytest.mark.parametrize("seed", range(6))
def test_select_signed_bruteforce_tiny(seed):
    # int32 columns with int32 bounds (Table I longitudes are negative)
    rng = np.random.default_rng(50 + seed)
    n = int(rng.integers(0, 80))
    a = rng.integers(-2**31, 2**31, n, dtype=np.int64).astype(np.int32)
    b = rng.integers(-300, 300, n).astype(np.int32)
    lo_a, hi_a = sorted(rng.integers(-2**31, 2**31, 2, dtype=np.int64).tolist())
    lo_b, hi_b = sorted(rng.integers(-300, 300, 2).tolist())
    pos, cnt, _ = oracle.select_sum([a, b], [lo_a, lo_b], [hi_a, hi_b], signed=[True, True])
    want = [i for i in range(n) if lo_a <= int(a[i]) <= hi_a and lo_b <= int(b[i]) <= hi_b]
    assert pos.tolist() == want and cnt == len(want)


def test_select_signed_spans_zero():
    # [-5, 5] on int32: unsigned order would select nothing of the negatives
    v = np.array([-7, -5, -1, 0, 4, 5, 6, -2**31, 2**31 - 1], dtype=np.int32)
    pos, cnt, _ = oracle.select_sum([v], [-5], [5], signed=[True])
    assert pos.tolist() == [1, 2, 3, 4, 5]
