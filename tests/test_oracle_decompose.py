"""Pins for oracle.decompose (BWD split, PAPER.md:143-160 s II-A, Fig. 2)."""
import numpy as np
import pytest

import oracle
from tests.conftest import read_golden


def test_oracle_decompose_fig2():
    g = read_golden("fig2_decomposition.txt")
    v = int(g["value"])
    assert format(v, "032b") == g["bits"]                      # the printed bit pattern
    k = int(g["cpu_bits"])
    major, residual, w = oracle.decompose(np.array([v], dtype=np.uint32), k)
    assert int(major[0]) == int(g["major_bits_string"], 2)    # 5843
    assert int(residual[0]) == int(g["residual_bits_string"], 2)  # 75
    assert w == int(g["gpu_bits"])                              # 13 stored major bits
    assert 32 - w - k == int(g["leading_zeros"])                # 12 leading zeros removed


EDGE = [0, 1, 2, 3, 127, 128, 255, 256, 2**16 - 1, 2**16, 2**24 - 1, 2**24, 2**31 - 1, 2**31,
        2**32 - 2, 2**32 - 1, 0x5A5A5A37, 747979]


@pytest.mark.parametrize("k", list(range(0, 33)))
def test_oracle_decompose_roundtrip(k):
    rng = np.random.default_rng(100 + k)
    v = np.concatenate([np.array(EDGE, dtype=np.uint64),
                        rng.integers(0, 2**32, 500, dtype=np.uint64)]).astype(np.uint32)
    major, residual, w = oracle.decompose(v, k)
    for x, m, r in zip(v.tolist(), major.tolist(), residual.tolist()):
        # reconstruction by bitwise concatenation (Alg. 2 "+bw")
        assert (m << k) | r == x
        assert r < (1 << k)                       # residual holds exactly k bits
    # non-redundant split: major width + residual width <= 32
    assert w + k <= 32
    assert w == max(major.tolist()).bit_length()  # leading zeros removed


def test_oracle_decompose_base():
    # prefix base (metadata "base for the prefix compression"): u = v - base
    v = np.array([1000, 1001, 1255, 1256, 5000], dtype=np.uint32)
    major, residual, w = oracle.decompose(v, 8, base=1000)
    assert [((m << 8) | r) + 1000 for m, r in zip(major.tolist(), residual.tolist())] == v.tolist()
    assert major.tolist() == [0, 0, 0, 1, 15]
    assert w == 4


def test_oracle_decompose_all_zero_major():
    v = np.array([0, 1, 200, 255], dtype=np.uint32)
    major, residual, w = oracle.decompose(v, 8)
    assert major.tolist() == [0, 0, 0, 0] and residual.tolist() == v.tolist() and w == 0
