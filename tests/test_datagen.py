"""Synthetic input generators: C == numpy mirror, shard independence, and the
value-domain facts the paper states for the Q6 columns."""
import math

import numpy as np

import datagen
import oracle


def test_uniform_c_matches_numpy():
    for lo, hi in [(0, 2**32 - 1), (5, 17), (1, 50)]:
        c = datagen.uniform_u32(42, 10007, lo, hi, row0=123, stream=3)
        p = datagen.uniform_u32_np(42, 10007, lo, hi, row0=123, stream=3)
        assert np.array_equal(c, p)


def test_q6_c_matches_numpy():
    c = datagen.q6_columns(2, 10, n=20011, row0=59_000_000)
    p = datagen.q6_columns_np(2, 10, n=20011, row0=59_000_000)
    for k in c:
        assert np.array_equal(c[k], p[k]), k


def test_shard_independence():
    full = datagen.q6_columns(4, 1, n=100000)
    a = datagen.q6_columns(4, 1, n=37000)
    b = datagen.q6_columns(4, 1, n=63000, row0=37000)
    for k in full:
        assert np.array_equal(full[k], np.concatenate([a[k], b[k]]))
    t1 = datagen.uniform_u32(1, 200000, threads=1)
    t8 = datagen.uniform_u32(1, 200000, threads=8)
    assert np.array_equal(t1, t8)


def test_bijection_is_permutation():
    for N in [1, 2, 3, 1000, 65537]:
        p = datagen.bijection_u32(3, N)
        assert np.array_equal(np.sort(p), np.arange(N, dtype=np.uint32))
    part = datagen.bijection_u32(3, 65537, n=1000, row0=500)
    assert np.array_equal(part, datagen.bijection_u32(3, 65537)[500:1500])


def test_datagen_shapes():
    c = datagen.q6_columns(2, 1)                          # SF1: 6 M rows
    n = c["shipdate"].size
    assert n == 6_000_000
    sd, q, d, ep = c["shipdate"], c["quantity"], c["discount"], c["extprice"]
    # "l_quantity: 50 values/6 bits, l_discount: 10 values/4 bits and l_shipdate: 2526 values/12 bits"
    assert q.min() == 1 and q.max() == 50 and np.unique(q).size == 50 and int(q.max()).bit_length() == 6
    assert d.min() == 0 and d.max() == 10 and int(d.max()).bit_length() == 4   # 11 values
    assert sd.min() >= 1 and sd.max() <= 2526 and int(sd.max()).bit_length() == 12
    assert np.unique(sd).size >= 2500
    assert int(ep.max()) < 2**24                          # 24-bit l_extendedprice
    # derived column: extprice is a multiple of quantity
    assert np.all(ep % q == 0)


def _within_5sigma(count, n, p):
    sigma = math.sqrt(n * p * (1 - p))
    return abs(count - n * p) <= 5 * sigma


def test_q6_selectivity_closed_form():
    c = datagen.q6_columns(2, 1)
    n = c["shipdate"].size
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    cols = [c["shipdate"], c["discount"], c["quantity"]]
    _, cnt, _ = oracle.select_sum(cols, los, his, positions=False, threads=0)
    p = 365 / 2406 * 3 / 11 * 23 / 50                      # 1.903 %, SURVEY s8(c) pins
    assert _within_5sigma(cnt, n, p)
    # candidates with shipdate decomposed 24/8 (k = 8): majors 2..4 -> 768 days; definite: major 3
    cpos, cdef = oracle.approx_select(cols, [8, 0, 0], los, his)
    assert _within_5sigma(cpos.size, n, 768 / 2406 * 3 / 11 * 23 / 50)   # 4.00 %
    assert _within_5sigma(int(cdef.sum()), n, 256 / 2406 * 3 / 11 * 23 / 50)  # 1.33 %


def test_spatial_c_matches_numpy():
    for row0 in (0, 1_000_003):
        c = datagen.spatial_columns(6, 50_000, row0=row0)
        m = datagen.spatial_columns_np(6, 50_000, row0=row0)
        assert np.array_equal(c["lon"], m["lon"]) and np.array_equal(c["lat"], m["lat"])


def test_spatial_shape():
    # inside the paper's bounding box; trips of 128 fixes; the Table I query
    # box holds a small, non-empty fraction of the fixes
    c = datagen.spatial_columns(6, 2_000_000)
    (lon_lo, lon_hi), (lat_lo, lat_hi) = datagen.SPATIAL_BOX
    assert c["lon"].min() >= lon_lo and c["lon"].max() <= lon_hi and c["lon"].min() < 0 < c["lon"].max()
    assert c["lat"].min() >= lat_lo and c["lat"].max() <= lat_hi
    hit = ((c["lon"] >= datagen.SPATIAL_LON[0]) & (c["lon"] <= datagen.SPATIAL_LON[1])
           & (c["lat"] >= datagen.SPATIAL_LAT[0]) & (c["lat"] <= datagen.SPATIAL_LAT[1]))
    assert 1e-4 < hit.mean() < 1e-2
    # consecutive fixes of one trip move by at most step + jitter
    d = np.abs(np.diff(c["lon"][:128].astype(np.int64)))
    assert d.max() <= 30 + 6
