"""Pins of the grouped COUNT / SUM oracle (s IV-E/F; Fig. 4): the
figure's grouped count, pure-Python brute force on tiny tables, closed forms."""
import random

import numpy as np
import pytest

import oracle


def test_fig4_grouped_count(golden):
    g = golden("fig4_groupby.txt")
    a = np.array([int(v) for v in g["A"].split(",")], dtype=np.uint32)
    b = np.array([int(v) for v in g["B"].split(",")], dtype=np.uint32)
    sums, cnts = oracle.select_group_sum([a], [0], [4], b, 8)          # A < 5  ->  A in [0, 4]
    assert list(np.nonzero(cnts)[0]) == [int(g["groups_with_rows"])]
    assert int(cnts.sum()) == int(g["counts"])


@pytest.mark.parametrize("seed", range(30))
def test_group_brute_force(seed):
    rng = random.Random(seed)
    n = rng.randint(0, 15)
    G = rng.randint(1, 6)
    x = np.array([rng.randint(0, 20) for _ in range(n)], dtype=np.uint32)
    key = np.array([rng.randint(0, G - 1) for _ in range(n)], dtype=np.uint32)
    y = np.array([rng.randint(0, 1000) for _ in range(n)], dtype=np.uint32)
    z = np.array([rng.randint(0, 9) for _ in range(n)], dtype=np.uint32)
    lo, hi = sorted((rng.randint(0, 20), rng.randint(0, 20)))
    want_s, want_c = [0] * G, [0] * G
    for i in range(n):
        if lo <= int(x[i]) <= hi:
            want_c[int(key[i])] += 1
            want_s[int(key[i])] += int(y[i]) * int(z[i])
    sums, cnts = oracle.select_group_sum([x], [lo], [hi], key, G, [y, z])
    assert list(cnts) == want_c and list(sums) == want_s
    _, cnt1 = oracle.select_group_sum([x], [lo], [hi], key, G)
    assert list(cnt1) == want_c


def test_group_closed_forms():
    n, G = 10_000, 7
    i = np.arange(n, dtype=np.uint32)
    key = (i % G).astype(np.uint32)
    ones = np.ones(n, dtype=np.uint32)
    sums, cnts = oracle.select_group_sum([ones], [0], [5], key, G, [ones])
    assert list(cnts) == [len(range(g, n, G)) for g in range(G)] and list(sums) == list(cnts)
    sums, _ = oracle.select_group_sum([ones], [0], [5], key, G, [i])
    assert list(sums) == [sum(range(g, n, G)) for g in range(G)]   # arithmetic series per residue class
    _, cnts = oracle.select_group_sum([ones], [2], [5], key, G)      # nothing qualifies
    assert int(cnts.sum()) == 0


def test_group_key_out_of_range():
    with pytest.raises(ValueError):
        oracle.select_group_sum([np.zeros(3, np.uint32)], [0], [0], np.array([0, 5, 1], np.uint32), 4)


# ---- arbitrary (non-dense) keys: oracle.select_group_sum_keys

@pytest.mark.parametrize("seed", range(30))
def test_group_keys_brute_force(seed):
    rng = random.Random(500 + seed)
    n = rng.randint(0, 25)
    pool = [rng.randint(0, 2**32 - 1) for _ in range(rng.randint(1, 6))]
    x = np.array([rng.randint(0, 20) for _ in range(n)], dtype=np.uint32)
    key = np.array([rng.choice(pool) for _ in range(n)], dtype=np.uint32)
    y = np.array([rng.randint(0, 10**6) for _ in range(n)], dtype=np.uint32)
    z = np.array([rng.randint(0, 9) for _ in range(n)], dtype=np.uint32)
    lo, hi = sorted((rng.randint(0, 20), rng.randint(0, 20)))
    want = {}
    for i in range(n):
        if lo <= int(x[i]) <= hi:
            c, s = want.get(int(key[i]), (0, 0))
            want[int(key[i])] = (c + 1, s + int(y[i]) * int(z[i]))
    keys, cnts, sums = oracle.select_group_sum_keys([x], [lo], [hi], key, [y, z])
    assert keys.tolist() == sorted(want)
    assert cnts.tolist() == [want[k][0] for k in sorted(want)]
    assert sums.tolist() == [want[k][1] for k in sorted(want)]


def test_group_keys_dense_special_case_and_constant_key():
    rng = np.random.default_rng(4)
    n, G = 20_000, 37
    x = rng.integers(0, 100, n).astype(np.uint32)
    key = rng.integers(0, G, n).astype(np.uint32)
    y = rng.integers(0, 10**6, n).astype(np.uint32)
    # dense keys: the same answer as select_group_sum, restricted to the non-empty groups
    sums, cnts = oracle.select_group_sum([x], [10], [60], key, G, [y])
    k2, c2, s2 = oracle.select_group_sum_keys([x], [10], [60], key, [y])
    nz = np.nonzero(cnts)[0]
    assert k2.tolist() == nz.tolist() and c2.tolist() == cnts[nz].tolist() and s2.tolist() == sums[nz].tolist()
    # one key value: the single group is the ungrouped select + SUM
    const = np.full(n, 0xDEADBEEF, dtype=np.uint32)
    _, cnt, s = oracle.select_sum([x], [10], [60], [y], positions=False)
    assert [a.tolist() for a in oracle.select_group_sum_keys([x], [10], [60], const, [y])] == [[0xDEADBEEF], [cnt], [s]]


def test_group_keys_closed_form_and_limits():
    n = 3000
    i = np.arange(n, dtype=np.uint32)
    key = ((i % 10) * 1_000_003 + 7).astype(np.uint32)           # 10 sparse keys
    ones = np.ones(n, dtype=np.uint32)
    keys, cnts, sums = oracle.select_group_sum_keys([ones], [1], [1], key, [i])
    assert keys.tolist() == [g * 1_000_003 + 7 for g in range(10)]
    assert cnts.tolist() == [300] * 10 and sums.tolist() == [sum(range(g, n, 10)) for g in range(10)]
    assert [a.size for a in oracle.select_group_sum_keys([ones], [2], [5], key)] == [0, 0, 0]
    with pytest.raises(ValueError):
        oracle.select_group_sum_keys([ones], [1], [1], key, max_groups=5)
