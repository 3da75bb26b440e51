"""CPU oracle for A&R over BWD columns -- TEST INFRASTRUCTURE ONLY.

Plain, slow, obviously correct definitions of what the hot path computes,
written from the paper (PAPER.md = H. Pirk, S. Manegold, M. Kersten, "Waste
Not... Efficient Co-Processing of Relational Data", ICDE 2014).  The arithmetic
lives in plain C (`oracle.c`, compiled with gcc on demand); this module only
marshals numpy arrays.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline and
`--impl reference` legs may import this package.  The product package
(paper_conf_icde_pirkmk14_b200) never imports it, and the two share no code.

Pins (tests/test_oracle_*.py):
  decompose       Fig. 2 worked value, round trip, non-redundancy
  bucket_flags    Fig. 4, Fig. 6, brute-force
                  exists/forall over residuals, printed f(x) superset
  select_sum      brute force on tiny tables, closed-form sums, thread-count invariance
  sum_at          closed forms
  sum_bounds      brute force over every residual of tiny tables, k = 0 collapse to the
                  exact answer, closed forms, containment of the exact answer
  select_minmax   pure-Python brute force on tiny tables, closed forms
  select_group_sum  Fig. 4's grouped count, pure-Python brute force, closed forms
  select_group_sum_keys  pure-Python dict grouping on tiny tables, the dense-key special case equals
                  select_group_sum, one constant key equals select_sum, closed forms
  minmax_ar       Fig. 6 (the false positive holds the single minimal
                  approximation, the propagated set still holds the true minimum), refined
                  answer == select_minmax, bounds contain it, k = 0 collapse, brute force
No function is "parity unpinned".
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None

OPS = {"==": 0, ">": 1, ">=": 2, "<": 3, "<=": 4}


def build(force: bool = False) -> str:
    """Compile liboracle.so in-tree with gcc (plain C, pthreads)."""
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
        p, i64, i32, u32 = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int, ctypes.c_uint32
        lib.or_decompose.argtypes = [p, i64, i32, u32, p, p]
        lib.or_decompose.restype = i32
        lib.or_bucket_flags.argtypes = [p, i64, i32, u32, u32, u32, p, p]
        lib.or_paper_f_flags.argtypes = [p, i64, i32, i32, u32, p]
        lib.or_select_sum.argtypes = [i64, i32, p, p, p, p, i32, p, p, p, p, i32]
        lib.or_select_sum.restype = i32
        lib.or_sum_at.argtypes = [p, i64, i32, p, p]
        lib.or_sum_at.restype = i32
        lib.or_sum_bounds.argtypes = [i64, i32, p, p, p, p, p, p, i32, p, p, p, p]
        lib.or_sum_bounds.restype = i32
        lib.or_select_minmax.argtypes = [i64, i32, p, p, p, p, p, i32, i32, p]
        lib.or_minmax_ar.argtypes = [i64, i32, p, p, p, p, p, p, p, i32, u32, i32, i32, p, p]
        lib.or_select_group_sum.argtypes = [i64, i32, p, p, p, p, i32, i32, p, p, p]
        lib.or_select_group_sum.restype = i32
        lib.or_select_group_sum_keys.argtypes = [i64, i32, p, p, p, p, p, i32, p, i64, p, p, p, p]
        lib.or_select_group_sum_keys.restype = i32
        lib.or_threads_default.restype = i32
        _lib = lib
    return _lib


def _u32(a):
    a = np.ascontiguousarray(a, dtype=np.uint32)
    return a


def _ptr(a):
    return a.ctypes.data_as(ctypes.c_void_p)


def _ptr_array(arrs):
    arr = (ctypes.c_void_p * max(1, len(arrs)))(*[a.ctypes.data for a in arrs])
    return arr


def _signed_preds(pred_cols, los, his, signed):
    """int32 predicate columns / bounds as their uint32 bit patterns, plus the per-predicate flags
    (None when every predicate is unsigned)."""
    if signed is None:
        return [_u32(c) for c in pred_cols], list(los), list(his), None
    sg = np.asarray([1 if x else 0 for x in signed], dtype=np.int32)
    cols = [np.ascontiguousarray(c).view(np.uint32) if np.asarray(c).dtype == np.int32 else _u32(c)
            for c in pred_cols]
    return cols, [int(x) & 0xFFFFFFFF for x in los], [int(x) & 0xFFFFFFFF for x in his], sg


def default_threads() -> int:
    return int(_load().or_threads_default())


def decompose(v, k: int, base: int = 0):
    """(major, residual, w_M) of the BWD split with k residual bits (Fig. 2)."""
    v = _u32(v)
    major = np.empty_like(v)
    residual = np.empty_like(v)
    w = _load().or_decompose(_ptr(v), v.size, k, base, _ptr(major), _ptr(residual))
    return major, residual, int(w)


def bucket_flags(major, k: int, lo: int, hi: int, base: int = 0):
    """(cand, def) bool flags of lo <= v <= hi on the approximation."""
    major = _u32(major)
    cand = np.empty(major.size, dtype=np.uint8)
    dfn = np.empty(major.size, dtype=np.uint8)
    _load().or_bucket_flags(_ptr(major), major.size, k, base, lo, hi, _ptr(cand), _ptr(dfn))
    return cand.astype(bool), dfn.astype(bool)


def paper_f_flags(v, k: int, op: str, x: int):
    """Candidate flags under the printed relaxation f(x)."""
    v = _u32(v)
    flag = np.empty(v.size, dtype=np.uint8)
    _load().or_paper_f_flags(_ptr(v), v.size, k, OPS[op], x, _ptr(flag))
    return flag.astype(bool)


def approx_select(values, ks, los, his, base=None, signed=None):
    """Reference intermediates of the approximate selection (conjunction of predicates):
    returns (cand_positions int64, definite flags at those positions).  Each predicate
    column is decomposed with its own k; cand/def of a row are the ANDs over predicates.
    signed[c] true: column c is int32 and its bounds are signed; it is decomposed in the
    order-preserving key domain d = v ^ 2^31 (DESIGN R8), base[c] in that domain."""
    n = len(values[0])
    cand = np.ones(n, dtype=bool)
    dfn = np.ones(n, dtype=bool)
    for c, v in enumerate(values):
        b = 0 if base is None else base[c]
        lo, hi = int(los[c]), int(his[c])
        v = np.asarray(v)
        if signed is not None and signed[c]:
            v = np.ascontiguousarray(v).view(np.uint32) ^ np.uint32(0x80000000)
            lo, hi = (lo & 0xFFFFFFFF) ^ 0x80000000, (hi & 0xFFFFFFFF) ^ 0x80000000
        major, _, _ = decompose(v, ks[c], b)
        cf, df = bucket_flags(major, ks[c], lo, hi, b)
        cand &= cf
        dfn &= df
    pos = np.nonzero(cand)[0].astype(np.int64)
    return pos, dfn[pos]


def select_sum(pred_cols, los, his, agg_cols=(), threads: int = 1, positions: bool = True, signed=None):
    """Exact select + product SUM (the plain definition): returns (positions|None, count, sum).
    signed[p] true: predicate p's column (int32 array) and bounds compare as int32."""
    sg = None
    if signed is not None:
        sg = np.asarray([1 if x else 0 for x in signed], dtype=np.int32)
        pred_cols = [np.ascontiguousarray(c).view(np.uint32) if np.asarray(c).dtype == np.int32 else c
                     for c in pred_cols]
        los = [int(x) & 0xFFFFFFFF for x in los]
        his = [int(x) & 0xFFFFFFFF for x in his]
    pred_cols = [_u32(c) for c in pred_cols]
    agg_cols = [_u32(c) for c in agg_cols]
    n = pred_cols[0].size if pred_cols else (agg_cols[0].size if agg_cols else 0)
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    out = np.empty(n if positions else 1, dtype=np.int64)
    cnt = ctypes.c_int64(0)
    s = ctypes.c_int64(0)
    pc, ac = _ptr_array(pred_cols), _ptr_array(agg_cols)
    ovf = _load().or_select_sum(n, len(pred_cols), ctypes.cast(pc, ctypes.c_void_p), _ptr(lo), _ptr(hi),
                                _ptr(sg) if sg is not None else None, len(agg_cols), ctypes.cast(ac, ctypes.c_void_p),
                                _ptr(out) if positions else None, ctypes.byref(cnt), ctypes.byref(s),
                                threads)
    if ovf:
        raise OverflowError("exact SUM does not fit in int64")
    return (out[: cnt.value] if positions else None), int(cnt.value), int(s.value)


def sum_at(pos, agg_cols):
    """Exact product SUM at given positions (SUM(refine), Fig. 3 / Fig. 7)."""
    pos = np.ascontiguousarray(pos, dtype=np.int64)
    agg_cols = [_u32(c) for c in agg_cols]
    s = ctypes.c_int64(0)
    ac = _ptr_array(agg_cols)
    if _load().or_sum_at(_ptr(pos), pos.size, len(agg_cols), ctypes.cast(ac, ctypes.c_void_p), ctypes.byref(s)):
        raise OverflowError("exact SUM does not fit in int64")
    return int(s.value)


def sum_bounds(pred_cols, pred_ks, los, his, agg_cols=(), agg_ks=(), pred_bases=None, agg_bases=None,
               pred_signed=None):
    """bwd.sumapproximate (Fig. 7; bounds PAPER.md:375-382):
    (sum_lo, sum_hi, count_lo, count_hi) from the approximation alone.  pred_signed[p]: predicate p's
    column is int32 (bounds signed, base in the key domain v ^ 2^31)."""
    pred_cols, los, his, sg = _signed_preds(pred_cols, los, his, pred_signed)
    agg_cols = [_u32(c) for c in agg_cols]
    n = pred_cols[0].size
    npred, nagg = len(pred_cols), len(agg_cols)
    pks = np.asarray(pred_ks, dtype=np.int32)
    aks = np.asarray(list(agg_ks) or [0], dtype=np.int32)
    pb = np.asarray(pred_bases if pred_bases is not None else [0] * npred, dtype=np.uint32)
    ab = np.asarray(agg_bases if agg_bases is not None else [0] * max(nagg, 1), dtype=np.uint32)
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    out = np.zeros(4, dtype=np.int64)
    pc, ac = _ptr_array(pred_cols), _ptr_array(agg_cols)
    if _load().or_sum_bounds(n, npred, ctypes.cast(pc, ctypes.c_void_p), _ptr(pks), _ptr(pb), _ptr(lo), _ptr(hi),
                             _ptr(sg) if sg is not None else None, nagg, ctypes.cast(ac, ctypes.c_void_p), _ptr(aks), _ptr(ab), _ptr(out)):
        raise OverflowError("SUM bound does not fit in int64")
    return tuple(int(x) for x in out)


def select_minmax(pred_cols, los, his, ycol, mode: str = "min", signed=None, y_signed: bool = False):
    """Exact select min(Y) / max(Y) over the conjunction (the plain definition):
    (value, |R|); value is 0 when R is empty."""
    sg = None
    if signed is not None:
        sg = np.asarray([1 if x else 0 for x in signed], dtype=np.int32)
        pred_cols = [np.ascontiguousarray(c).view(np.uint32) if np.asarray(c).dtype == np.int32 else c
                     for c in pred_cols]
        los = [int(x) & 0xFFFFFFFF for x in los]
        his = [int(x) & 0xFFFFFFFF for x in his]
    pred_cols = [_u32(c) for c in pred_cols]
    y = np.ascontiguousarray(ycol).view(np.uint32) if np.asarray(ycol).dtype == np.int32 else _u32(ycol)
    n = y.size
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    out = np.zeros(2, dtype=np.int64)
    pc = _ptr_array(pred_cols)
    _load().or_select_minmax(n, len(pred_cols), ctypes.cast(pc, ctypes.c_void_p), _ptr(lo), _ptr(hi),
                             _ptr(sg) if sg is not None else None, _ptr(y), 1 if y_signed else 0,
                             0 if mode == "min" else 1, _ptr(out))
    return int(out[0]), int(out[1])


def minmax_ar(pred_cols, pred_ks, los, his, ycol, y_k: int, mode: str = "min", pred_bases=None,
              y_base: int = 0, y_signed: bool = False, flags: bool = False, pred_signed=None):
    """A&R MIN / MAX of s IV-F: dict with the refined answer and survivors,
    the approximate bounds (lo, hi), |refined|, |D|, |C|, and (flags=True) the refined-row mask.
    pred_signed[p]: predicate p's column is int32 (bounds signed, base in the key domain)."""
    pred_cols, los, his, sg = _signed_preds(pred_cols, los, his, pred_signed)
    y = np.ascontiguousarray(ycol).view(np.uint32) if np.asarray(ycol).dtype == np.int32 else _u32(ycol)
    n = y.size
    npred = len(pred_cols)
    pks = np.asarray(pred_ks, dtype=np.int32)
    pb = np.asarray(pred_bases if pred_bases is not None else [0] * npred, dtype=np.uint32)
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    out = np.zeros(7, dtype=np.int64)
    fl = np.zeros(max(n, 1), dtype=np.uint8)
    pc = _ptr_array(pred_cols)
    _load().or_minmax_ar(n, npred, ctypes.cast(pc, ctypes.c_void_p), _ptr(pks), _ptr(pb), _ptr(lo), _ptr(hi),
                         _ptr(sg) if sg is not None else None, _ptr(y), y_k, y_base & 0xFFFFFFFF, 1 if y_signed else 0, 0 if mode == "min" else 1,
                         _ptr(out), _ptr(fl) if flags else None)
    r = {"value": int(out[0]), "survivors": int(out[1]), "lo": int(out[2]), "hi": int(out[3]),
         "refined": int(out[4]), "definite": int(out[5]), "candidates": int(out[6])}
    if flags:
        r["refine_flags"] = fl[:n].astype(bool)
    return r


def select_group_sum(pred_cols, los, his, key, ngroups: int, agg_cols=()):
    """Exact grouped COUNT / product SUM over the selection (s IV-E; Fig. 4 "select count(*) from R where
    A<5 groupby B"): (sums int64[ngroups], counts int64[ngroups]), group id = key value."""
    pred_cols = [_u32(c) for c in pred_cols]
    agg_cols = [_u32(c) for c in agg_cols]
    key = _u32(key)
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    sums = np.zeros(max(ngroups, 1), dtype=np.int64)
    cnts = np.zeros(max(ngroups, 1), dtype=np.int64)
    pc, ac = _ptr_array(pred_cols), _ptr_array(agg_cols)
    rc = _load().or_select_group_sum(key.size, len(pred_cols), ctypes.cast(pc, ctypes.c_void_p), _ptr(lo), _ptr(hi),
                                     _ptr(key), ngroups, len(agg_cols), ctypes.cast(ac, ctypes.c_void_p),
                                     _ptr(sums), _ptr(cnts))
    if rc == 1:
        raise OverflowError("a group SUM does not fit in int64")
    if rc == 2:
        raise ValueError("a qualifying row has key >= ngroups")
    return sums[:ngroups], cnts[:ngroups]


def select_group_sum_keys(pred_cols, los, his, key, agg_cols=(), signed=None, max_groups=1 << 20):
    """Exact grouped COUNT / product SUM over the selection for arbitrary uint32 keys (s IV-E, the plain
    definition): (keys ascending, counts, sums) of the groups among the qualifying rows."""
    pred_cols, los, his, sg = _signed_preds(pred_cols, los, his, signed)
    agg_cols = [_u32(c) for c in agg_cols]
    key = np.ascontiguousarray(key).view(np.uint32) if np.asarray(key).dtype == np.int32 else _u32(key)
    lo = np.asarray(los, dtype=np.uint32)
    hi = np.asarray(his, dtype=np.uint32)
    cap = max(1, int(max_groups))
    keys = np.zeros(cap, dtype=np.uint32)
    cnts = np.zeros(cap, dtype=np.int64)
    sums = np.zeros(cap, dtype=np.int64)
    ng = ctypes.c_int64(0)
    pc, ac = _ptr_array(pred_cols), _ptr_array(agg_cols)
    rc = _load().or_select_group_sum_keys(key.size, len(pred_cols), ctypes.cast(pc, ctypes.c_void_p), _ptr(lo),
                                          _ptr(hi), _ptr(sg) if sg is not None else None, _ptr(key),
                                          len(agg_cols), ctypes.cast(ac, ctypes.c_void_p), cap, _ptr(keys),
                                          _ptr(cnts), _ptr(sums), ctypes.byref(ng))
    if rc == 1:
        raise OverflowError("a group SUM does not fit in int64")
    if rc == 2:
        raise ValueError("more groups than max_groups")
    g = int(ng.value)
    return keys[:g], cnts[:g], sums[:g]
