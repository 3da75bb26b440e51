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
