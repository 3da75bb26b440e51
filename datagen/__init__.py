"""Seeded synthetic inputs shared by the oracle and the CUDA path.

This module holds none of the method's arithmetic (no decomposition,
relaxation, predicate or aggregate); it only generates the columns of the
paper's workloads.  The fast
generator is plain C (`datagen.c`, compiled on demand with gcc); `*_np`
functions are a line-by-line numpy mirror used by tests to check the C code.

Workload configs (BASELINE.json `configs`):
  C1  1M-row uniform u32 column, one 1 % range predicate
  C2  TPC-H SF10-shaped Q6 columns (60 M rows)
  C3  1 G-row u32 column (uniform, or a keyed bijection of [0, N))
  C4  SF100 Q6 row-sharded over G GPUs
  C5  SF1000 Q6, residuals in pinned host memory
  C6  spatial range count of Table I on GPS-fix-shaped int32 lon/lat
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "datagen.c")
_LIB = os.path.join(_HERE, "libdatagen.so")
_lock = threading.Lock()
_lib = None

GAMMA = 0x9E3779B97F4A7C15
ROWS_PER_SF = 6_000_000          # N = 6,000,000 x SF
PARTS_PER_SF = 200_000           # TPC-H part table cardinality [ext]

# Q6 predicates (TPC-H Q6 [ext]); shipdate is days since 1992-01-01
Q6_SHIPDATE = (731, 1095)        # [1994-01-01, 1995-01-01)
Q6_DISCOUNT = (5, 7)             # BETWEEN 0.05 AND 0.07, hundredths
Q6_QUANTITY = (0, 23)            # < 24

# config C6: Table I, degrees scaled 1e5 (decimal(8,5) / decimal(7,5))
SPATIAL_ROWS = 250_000_000        # "around 250 million tuples"
SPATIAL_LON = (268288, 270228)    # lon BETWEEN 2.68288 AND 2.70228
SPATIAL_LAT = (5042220, 5044850)  # lat BETWEEN 50.4222 AND 50.4485
SPATIAL_BOX = ((-1262427, 2964975), (2709371, 7013643))   # data range

# config C1
C1_N = 1_000_000
C1_LO = 0x5A5A5A37
C1_HI = C1_LO + int(0.01 * 2**32) - 1


def build(force: bool = False) -> str:
    """Compile libdatagen.so in-tree (gcc, -O2, pthreads)."""
    with _lock:
        if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
            tmp = _LIB + f".tmp{os.getpid()}"
            subprocess.check_call(["gcc", "-O2", "-fPIC", "-shared", "-pthread", "-o", tmp, _SRC])
            os.replace(tmp, _LIB)
    return _LIB


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        u64, u32, i64, i32, p = (ctypes.c_uint64, ctypes.c_uint32, ctypes.c_int64,
                                 ctypes.c_int, ctypes.c_void_p)
        lib.dg_key.argtypes = [u64, u32]
        lib.dg_key.restype = u64
        lib.dg_uniform_u32.argtypes = [u64, u32, u64, i64, u32, u32, p, i32]
        lib.dg_bijection_u32.argtypes = [u64, u32, u64, u64, i64, p, i32]
        lib.dg_q6.argtypes = [u64, u64, u64, i64, p, p, p, p, i32]
        lib.dg_spatial.argtypes = [u64, u64, i64, p, p, i32]
        lib.dg_threads_default.restype = i32
        _lib = lib
    return _lib


def _ptr(a):
    return None if a is None else a.ctypes.data_as(ctypes.c_void_p)


def _out(n, out):
    if out is None:
        return np.empty(n, dtype=np.uint32)
    assert out.dtype == np.uint32 and out.flags.c_contiguous and out.size >= n
    return out


def uniform_u32(seed, n, lo=0, hi=2**32 - 1, row0=0, stream=0, out=None, threads=0):
    out = _out(n, out)
    _load().dg_uniform_u32(seed, stream, row0, n, lo, hi, _ptr(out), threads)
    return out


def bijection_u32(seed, N, n=None, row0=0, stream=0, out=None, threads=0):
    n = N - row0 if n is None else n
    out = _out(n, out)
    _load().dg_bijection_u32(seed, stream, N, row0, n, _ptr(out), threads)
    return out


def q6_columns(seed, sf, n=None, row0=0, threads=0, which=("shipdate", "discount", "quantity", "extprice")):
    """TPC-H-lineitem-shaped Q6 columns for table rows [row0, row0+n) at scale factor sf."""
    if n is None:
        n = int(round(sf * ROWS_PER_SF)) - row0
    n_parts = max(1, int(round(sf * PARTS_PER_SF)))
    cols = {name: (np.empty(n, dtype=np.uint32) if name in which else None)
            for name in ("shipdate", "discount", "quantity", "extprice")}
    _load().dg_q6(seed, n_parts, row0, n, _ptr(cols["shipdate"]), _ptr(cols["discount"]),
                  _ptr(cols["quantity"]), _ptr(cols["extprice"]), threads)
    return {k: v for k, v in cols.items() if v is not None}


def spatial_columns(seed, n, row0=0, threads=0):
    """GPS-fix (lon, lat) int32 columns in 1e-5 degrees for rows [row0, row0+n) (config C6)."""
    lon = np.empty(n, dtype=np.int32)
    lat = np.empty(n, dtype=np.int32)
    _load().dg_spatial(seed, row0, n, _ptr(lon), _ptr(lat), threads)
    return {"lon": lon, "lat": lat}


def default_threads() -> int:
    return int(_load().dg_threads_default())


# --------------------------------------------------------------------------
# numpy mirror of datagen.c (tests only: checks the C generator)
# --------------------------------------------------------------------------
_M = np.uint64(0xFFFFFFFFFFFFFFFF)


def _mix64_np(z):
    z = np.asarray(z, dtype=np.uint64)
    with np.errstate(over="ignore"):
        z = (z ^ (z >> np.uint64(30))) * np.uint64(0xBF58476D1CE4E5B9)
        z = (z ^ (z >> np.uint64(27))) * np.uint64(0x94D049BB133111EB)
    return z ^ (z >> np.uint64(31))


def key_np(seed, stream):
    with np.errstate(over="ignore"):
        z = (np.uint64(seed) * np.uint64(GAMMA) + np.uint64(stream) * np.uint64(0xD1B54A32D192ED03)
             + np.uint64(1))
    return _mix64_np(z)


def _draw_np(key, rows):
    with np.errstate(over="ignore"):
        return _mix64_np(np.uint64(key) + (rows.astype(np.uint64) + np.uint64(1)) * np.uint64(GAMMA))


def _span_np(r, span):
    return (((r >> np.uint64(32)) * np.uint64(span)) >> np.uint64(32)).astype(np.uint64)


def uniform_u32_np(seed, n, lo=0, hi=2**32 - 1, row0=0, stream=0):
    rows = np.arange(row0, row0 + n, dtype=np.uint64)
    r = _draw_np(key_np(seed, stream), rows)
    return (np.uint64(lo) + _span_np(r, hi - lo + 1)).astype(np.uint32)


def q6_columns_np(seed, sf, n, row0=0):
    n_parts = max(1, int(round(sf * PARTS_PER_SF)))
    rows = np.arange(row0, row0 + n, dtype=np.uint64)
    od = _span_np(_draw_np(key_np(seed, 0), rows), 2406)
    sd = np.uint64(1) + _span_np(_draw_np(key_np(seed, 1), rows), 121)
    q = np.uint64(1) + _span_np(_draw_np(key_np(seed, 2), rows), 50)
    d = _span_np(_draw_np(key_np(seed, 3), rows), 11)
    pk = np.uint64(1) + _span_np(_draw_np(key_np(seed, 4), rows), n_parts)
    retail = (np.uint64(90000) + (pk // np.uint64(10)) % np.uint64(20001)
              + np.uint64(100) * (pk % np.uint64(1000)))
    return {"shipdate": (od + sd).astype(np.uint32), "discount": d.astype(np.uint32),
            "quantity": q.astype(np.uint32), "extprice": (q * retail).astype(np.uint32)}


def spatial_columns_np(seed, n, row0=0):
    rows = np.arange(row0, row0 + n, dtype=np.uint64)
    trip, j = rows // np.uint64(128), (rows % np.uint64(128)).astype(np.int64)

    def uni(stream, r, lo, hi):
        return lo + _span_np(_draw_np(key_np(seed, stream), r), hi - lo + 1).astype(np.int64)

    u = _span_np(_draw_np(key_np(seed, 12), trip), 1 << 16)
    with np.errstate(over="ignore"):
        city = (np.uint64(32) * u * u) >> np.uint64(32)
    (lon_lo, lon_hi), (lat_lo, lat_hi) = SPATIAL_BOX
    clon = np.where(city == 0, 269258, uni(10, city, lon_lo, lon_hi))
    clat = np.where(city == 0, 5043535, uni(11, city, lat_lo, lat_hi))
    slon = clon + uni(13, trip, -10000, 10000) + uni(19, trip, -10000, 10000)
    slat = clat + uni(14, trip, -10000, 10000) + uni(20, trip, -10000, 10000)
    lon = slon + j * uni(15, trip, -30, 30) + uni(17, rows, -3, 3)
    lat = slat + j * uni(16, trip, -30, 30) + uni(18, rows, -3, 3)
    return {"lon": np.clip(lon, lon_lo, lon_hi).astype(np.int32), "lat": np.clip(lat, lat_lo, lat_hi).astype(np.int32)}
