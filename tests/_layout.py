"""Test-only decoders of the bit layouts documented in include/ar.h (ar_layout).

Written from the layout text, independently of the CUDA packers, so that the
GPU bitstreams can be compared with oracle.decompose value by value.
"""
import numpy as np


def unpack_packed(buf: bytes, n: int, w: int) -> np.ndarray:
    """AR_LAYOUT_PACKED: LSB-first bitstream, row i at bits [i*w, i*w+w) of little-endian uint32 words."""
    if w == 0:
        return np.zeros(n, dtype=np.uint64)
    words = np.frombuffer(buf, dtype="<u4").astype(np.uint64)
    bits = np.arange(n, dtype=np.uint64) * np.uint64(w)
    wi = (bits >> np.uint64(5)).astype(np.int64)
    sh = bits & np.uint64(31)
    lo = words[wi]
    hi = words[np.minimum(wi + 1, words.size - 1)]
    v = ((lo | (hi << np.uint64(32))) >> sh) & np.uint64((1 << w) - 1)
    return v


def unpack_sliced(buf: bytes, n: int, w: int) -> np.ndarray:
    """AR_LAYOUT_SLICED: block b of 32 rows = w words, word j = bit j of rows 32b..32b+31 (bit l = row 32b+l)."""
    if w == 0:
        return np.zeros(n, dtype=np.uint64)
    words = np.frombuffer(buf, dtype="<u4").astype(np.uint64)
    rows = np.arange(n, dtype=np.int64)
    b, l = rows // 32, (rows % 32).astype(np.uint64)
    v = np.zeros(n, dtype=np.uint64)
    for j in range(w):
        v |= ((words[b * w + j] >> l) & np.uint64(1)) << np.uint64(j)
    return v


def unpack_split(buf: bytes, n: int, k: int, h: int) -> np.ndarray:
    """Split SLICED residual (ar_column_desc.residual_split = h): per 8192-row super-group of 256 blocks,
    first the h high planes of its blocks (h words per block: planes k-h .. k-1), then the k-h low planes
    (k-h words per block: planes 0 .. k-h-1); within a word bit l = row 32b+l of block b."""
    words = np.frombuffer(buf, dtype="<u4").astype(np.uint64)
    rows = np.arange(n, dtype=np.int64)
    b, l = rows // 32, (rows % 32).astype(np.uint64)
    sg, bb = (b // 256) * (256 * k), b % 256
    v = np.zeros(n, dtype=np.uint64)
    for j in range(k):
        if j >= k - h:
            idx = sg + bb * h + (j - (k - h))
        else:
            idx = sg + 256 * h + bb * (k - h) + j
        v |= ((words[idx] >> l) & np.uint64(1)) << np.uint64(j)
    return v
