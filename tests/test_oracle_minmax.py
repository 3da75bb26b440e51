"""Pins of the MIN / MAX oracle (s IV-F, Fig. 6): the worked
figure, pure-Python brute force on tiny tables, closed forms and the k = 0
collapse.  CPU only."""
import os
import random

import numpy as np
import pytest

import oracle

GOLD = os.path.join(os.path.dirname(__file__), "golden", "fig6_minmax_table.txt")


def _golden():
    d = {}
    for line in open(GOLD):
        line = line.strip()
        if line and not line.startswith("#"):
            k, v = line.split("=", 1)
            d[k] = v
    return d


def test_fig6_false_minimum_and_propagated_set():
    g = _golden()
    k = int(g["k"])
    x = np.array([int(v) for v in g["x"].split(",")], dtype=np.uint32)
    y = np.array([int(v) for v in g["y"].split(",")], dtype=np.uint32)
    lo, hi = int(g["precise_lo"]), 0xFFFFFFFF
    assert oracle.select_minmax([x], [lo], [hi], y, "min") == (int(g["precise_min"]), 2)
    r = oracle.minmax_ar([x], [k], [lo], [hi], y, k, "min", flags=True)
    # the single minimal approximation is the false positive ...
    ymaj = y >> k
    cands = [i for i in range(len(x)) if ((int(x[i]) >> k) << k) + (1 << k) - 1 >= lo]
    minimal = [i for i in cands if ymaj[i] == min(ymaj[j] for j in cands)]
    assert minimal == [int(v) for v in g["minimal_approximation_rows"].split(",")]
    assert not (x[minimal[0]] >= lo)
    # ... while the set with the selection's error bounds propagated holds the true minimum
    assert list(np.nonzero(r["refine_flags"])[0]) == [int(v) for v in g["propagated_rows"].split(",")]
    assert r["value"] == int(g["precise_min"])
    assert (r["lo"], r["hi"]) == (int(g["approx_lo"]), int(g["approx_hi"]))
    assert r["candidates"] == 3 and r["definite"] == 2


def _brute(xs, los, his, y, mode, y_signed=False):
    vals = []
    for i in range(len(y)):
        if all(lo <= int(c[i]) <= hi for c, lo, hi in zip(xs, los, his)):
            v = int(y[i])
            if y_signed and v >= 2 ** 31:
                v -= 2 ** 32
            vals.append(v)
    if not vals:
        return 0, 0
    return (min(vals) if mode == "min" else max(vals)), len(vals)


@pytest.mark.parametrize("seed", range(40))
def test_minmax_brute_force_tiny(seed):
    rng = random.Random(seed)
    n = rng.randint(0, 12)
    npred = rng.randint(1, 2)
    ks = [rng.randint(0, 3) for _ in range(npred)]
    xs = [np.array([rng.randint(0, 31) for _ in range(n)], dtype=np.uint32) for _ in range(npred)]
    los, his = [], []
    for _ in range(npred):
        a, b = rng.randint(0, 31), rng.randint(0, 31)
        los.append(min(a, b))
        his.append(max(a, b))
    y = np.array([rng.randint(0, 63) for _ in range(n)], dtype=np.uint32)
    ky = rng.randint(0, 4)
    for mode in ("min", "max"):
        want = _brute(xs, los, his, y, mode)
        assert oracle.select_minmax(xs, los, his, y, mode) == want
        r = oracle.minmax_ar(xs, ks, los, his, y, ky, mode, flags=True)
        assert (r["value"], r["survivors"] > 0) == (want[0], want[1] > 0)
        if want[1]:
            assert r["lo"] <= want[0] <= r["hi"]
            # every row of R that attains the answer is in the refined set
            for i in range(n):
                if all(lo <= int(c[i]) <= hi for c, lo, hi in zip(xs, los, his)) and int(y[i]) == want[0]:
                    assert r["refine_flags"][i]
        assert r["survivors"] <= r["refined"] <= r["candidates"]
        assert r["definite"] <= r["candidates"]


def test_minmax_k0_collapses_to_exact():
    rng = np.random.default_rng(7)
    x = rng.integers(0, 100, 500).astype(np.uint32)
    y = rng.integers(0, 1000, 500).astype(np.uint32)
    for mode in ("min", "max"):
        want, cnt = oracle.select_minmax([x], [20], [60], y, mode)
        r = oracle.minmax_ar([x], [0], [20], [60], y, 0, mode)
        # k = 0: D = C = R, the bounds are the answer, only the rows attaining it are refined
        assert r["definite"] == r["candidates"] == cnt
        assert r["lo"] == r["hi"] == r["value"] == want
        sel = (x >= 20) & (x <= 60)
        assert r["refined"] == r["survivors"] == int(np.sum(sel & (y == want)))


def test_minmax_closed_forms():
    # y_i = i over a full-range predicate: MIN = 0, MAX = n - 1; y constant: MIN = MAX = c
    n = 1000
    x = np.zeros(n, dtype=np.uint32)
    y = np.arange(n, dtype=np.uint32)
    assert oracle.select_minmax([x], [0], [0], y, "min") == (0, n)
    assert oracle.select_minmax([x], [0], [0], y, "max") == (n - 1, n)
    r = oracle.minmax_ar([x], [4], [0], [0xFFFFFFFF], y, 4, "max")
    assert r["value"] == n - 1 and r["hi"] == 1007 and r["lo"] == 992   # bucket of 999 at k = 4: [992, 1007]
    c = np.full(n, 77, dtype=np.uint32)
    assert oracle.select_minmax([x], [0], [0], c, "min") == (77, n)


def test_minmax_signed_y():
    rng = np.random.default_rng(3)
    x = rng.integers(0, 50, 300).astype(np.uint32)
    y = rng.integers(-2 ** 31, 2 ** 31 - 1, 300).astype(np.int32)
    for mode in ("min", "max"):
        want = _brute([x], [10], [30], y.view(np.uint32), mode, y_signed=True)
        assert oracle.select_minmax([x], [10], [30], y, mode, y_signed=True) == want
        r = oracle.minmax_ar([x], [3], [10], [30], y, 8, mode, y_signed=True, y_base=0)
        assert r["value"] == want[0]
        assert r["lo"] <= want[0] <= r["hi"]


def test_minmax_empty():
    x = np.array([1, 2, 3], dtype=np.uint32)
    y = np.array([4, 5, 6], dtype=np.uint32)
    assert oracle.select_minmax([x], [10], [20], y, "min") == (0, 0)
    r = oracle.minmax_ar([x], [1], [10], [20], y, 1, "min")
    assert (r["value"], r["survivors"], r["refined"], r["candidates"]) == (0, 0, 0, 0)
