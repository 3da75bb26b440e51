"""ctypes binding of include/ar.h (argument marshalling only).

Every function here has the name and argument order of the C entry point and
raises ARError when the call returns a status other than AR_OK.  All compute
happens in libar_b200.so (sm_100a kernels); there is no Python or CPU
fallback: if the library cannot be built or loaded, import fails loudly.
"""
from __future__ import annotations

import ctypes
import os

from . import build as _build

AR_OK, AR_ERR_INVALID, AR_ERR_RANGE, AR_ERR_CUDA, AR_ERR_NCCL, AR_ERR_UNSUPPORTED = range(6)
AR_LOC_DEVICE, AR_LOC_HOST_PINNED = 0, 1
AR_LAYOUT_SLICED, AR_LAYOUT_PACKED = 0, 1
AR_MAX_PRED, AR_MAX_AGG, AR_MAX_PLANES = 8, 2, 64
AR_SELECT_CARRY_APPR = 1
AR_DECOMPOSE_SIGNED, AR_DECOMPOSE_BASE_MIN = 1, 2


def AR_DECOMPOSE_SPLIT(h: int) -> int:
    return (h & 31) << 8
AR_AUX_DEFINITE = 0x80000000
AR_PROJECT_APPROX, AR_PROJECT_EXACT = 0, 1
AR_MIN, AR_MAX = 0, 1
AR_SRS_PDL, AR_SRS_PDL_EARLY_READ = 1, 2
AR_GROUP_APPROX, AR_GROUP_EXACT = 0, 1
AR_MAX_GROUPS = 4096


class ARError(RuntimeError):
    def __init__(self, status: int, func: str, detail: str):
        super().__init__(f"{func}: {STATUS_NAMES.get(status, status)}: {detail}")
        self.status = status


STATUS_NAMES = {0: "AR_OK", 1: "AR_ERR_INVALID", 2: "AR_ERR_RANGE", 3: "AR_ERR_CUDA", 4: "AR_ERR_NCCL",
                5: "AR_ERR_UNSUPPORTED"}


class ColumnDesc(ctypes.Structure):
    _fields_ = [("n", ctypes.c_int64), ("major_bits", ctypes.c_int32), ("k", ctypes.c_int32),
                ("w_major", ctypes.c_int32), ("major_layout", ctypes.c_int32), ("residual_loc", ctypes.c_int32),
                ("base", ctypes.c_uint32), ("major_bytes", ctypes.c_uint64), ("residual_bytes", ctypes.c_uint64),
                ("major_loc", ctypes.c_int32), ("residual_layout", ctypes.c_int32),
                ("value_signed", ctypes.c_int32), ("residual_split", ctypes.c_int32)]


class Pred(ctypes.Structure):
    _fields_ = [("col", ctypes.c_void_p), ("lo", ctypes.c_uint32), ("hi", ctypes.c_uint32)]


class Cands(ctypes.Structure):
    _fields_ = [("pos", ctypes.c_void_p), ("aux", ctypes.c_void_p), ("count", ctypes.c_void_p),
                ("capacity", ctypes.c_int64), ("appr_bits", ctypes.c_int32), ("reserved", ctypes.c_int32)]


class Positions(ctypes.Structure):
    _fields_ = [("pos", ctypes.c_void_p), ("count", ctypes.c_void_p), ("capacity", ctypes.c_int64)]


# name -> (restype, argtypes); restype c_int means ar_status
_P, _I64, _I32, _U32, _U64, _SZ = (ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32, ctypes.c_uint32,
                                   ctypes.c_uint64, ctypes.c_size_t)
SIGNATURES = {
    "ar_status_str": (ctypes.c_char_p, [ctypes.c_int]),
    "ar_last_error": (ctypes.c_char_p, []),
    "ar_version": (ctypes.c_char_p, []),
    "ar_last_scan_kernel": (ctypes.c_char_p, []),
    "ar_decompose_ws_bytes": (_SZ, []),
    "ar_decompose_plan": (ctypes.c_int, [_P, _I64, _I32, _I32, _I32, _U32, _I32, _P, _SZ, ctypes.POINTER(ColumnDesc),
                                         _P]),
    "ar_decompose": (ctypes.c_int, [_P, ctypes.POINTER(ColumnDesc), _P, _U64, _P, _U64, _P, ctypes.POINTER(_P)]),
    "ar_column_wrap": (ctypes.c_int, [ctypes.POINTER(ColumnDesc), _P, _P, ctypes.POINTER(_P)]),
    "ar_column_get_desc": (ctypes.c_int, [_P, ctypes.POINTER(ColumnDesc)]),
    "ar_column_free": (None, [_P]),
    "ar_select_ws_bytes": (_SZ, [_I64]),
    "ar_approx_select": (ctypes.c_int, [ctypes.POINTER(Pred), _I32, _I32, ctypes.POINTER(Cands), _P, _SZ, _P]),
    "ar_refine_ws_bytes": (_SZ, [_I64]),
    "ar_refine": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(Pred), _I32, ctypes.POINTER(Positions), _P,
                                 _SZ, _P]),
    "ar_sum": (ctypes.c_int, [ctypes.POINTER(Positions), ctypes.POINTER(_P), _I32, _P, _P]),
    "ar_sum_approximate": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(_P), _I32, _P, _P]),
    "ar_project": (ctypes.c_int, [ctypes.POINTER(Positions), _P, _I32, _P, _P]),
    "ar_minmax_ws_bytes": (_SZ, [_I64]),
    "ar_refine_group_sum": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(Pred), _I32, _P, ctypes.POINTER(_P),
                                           _I32, _I32, _P, _P]),
    "ar_minmax": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(Pred), _I32, _P, _I32, _P, _P, _SZ, _P]),
    "ar_refine_sum": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(Pred), _I32, ctypes.POINTER(_P), _I32,
                                     _P, _P, _P]),
    "ar_select_refine_sum": (ctypes.c_int, [ctypes.POINTER(Pred), _I32, ctypes.POINTER(_P), _I32, _P, _P]),
    "ar_select_refine_sum_ws_bytes": (_SZ, []),
    "ar_select_refine_sum_ws": (ctypes.c_int, [ctypes.POINTER(Pred), _I32, ctypes.POINTER(_P), _I32, _I32, _P, _P,
                                               _SZ, _P]),
    "ar_dist_unique_id_bytes": (_SZ, []),
    "ar_dist_get_unique_id": (ctypes.c_int, [_P]),
    "ar_dist_init": (ctypes.c_int, [ctypes.POINTER(_P), _P, _I32, _I32]),
    "ar_dist_offsets": (ctypes.c_int, [_P, _P, _P, _P, _P]),
    "ar_dist_sum": (ctypes.c_int, [_P, _P, _I32, _P]),
    "ar_dist_free": (None, [_P]),
    "ar_dist_shard_range": (ctypes.c_int, [_I64, _I32, _I32, ctypes.POINTER(_I64), ctypes.POINTER(_I64)]),
    "ar_dist_exclusive_offsets": (ctypes.c_int, [_P, _I32, _I32, _P, _P, _P]),
    "ar_dist_concat_positions": (ctypes.c_int, [ctypes.POINTER(Positions), _I64, _P, _P, _I64, _P, _P]),
    "ar_decompose_set_width": (ctypes.c_int, [ctypes.POINTER(ColumnDesc), _I32]),
    "ar_group_table_bytes": (_SZ, [_I64]),
    "ar_group_ids": (ctypes.c_int, [ctypes.POINTER(Positions), _P, _I32, _P, _I64, _I32, _P, _P, _P, _P, _P]),
    "ar_refine_group_sum_ids": (ctypes.c_int, [ctypes.POINTER(Cands), ctypes.POINTER(Pred), _I32, _P, _I32,
                                               ctypes.POINTER(_P), _I32, _P, _P]),
}

_lib = None


def lib_path() -> str:
    return _build.OUT


def load():
    """Load libar_b200.so (building it in-tree with nvcc if it is missing or stale)."""
    global _lib
    if _lib is None:
        path = _build.build()
        if not os.path.exists(path):
            raise ImportError(f"libar_b200.so not found at {path}")
        lib = ctypes.CDLL(path)
        for name, (res, args) in SIGNATURES.items():
            f = getattr(lib, name)
            f.restype = res
            f.argtypes = args
        _lib = lib
    return _lib


def _check(status: int, func: str):
    if status != AR_OK:
        detail = load().ar_last_error()
        raise ARError(status, func, detail.decode() if detail else "")


def _call(name, *args):
    st = getattr(load(), name)(*args)
    _check(st, name)
    return st


def ar_version() -> str:
    return load().ar_version().decode()


def ar_last_scan_kernel() -> str:
    return load().ar_last_scan_kernel().decode()


def ar_decompose_ws_bytes() -> int:
    return int(load().ar_decompose_ws_bytes())


def ar_decompose_plan(col, n, major_bits, major_layout, residual_loc, base, flags, ws, ws_bytes,
                      stream) -> ColumnDesc:
    desc = ColumnDesc()
    _call("ar_decompose_plan", col, n, major_bits, major_layout, residual_loc, base, flags, ws, ws_bytes,
          ctypes.byref(desc), stream)
    return desc


def ar_decompose(col, desc, major_buf, major_buf_bytes, residual_buf, residual_buf_bytes, stream) -> int:
    out = ctypes.c_void_p()
    _call("ar_decompose", col, ctypes.byref(desc), major_buf, major_buf_bytes, residual_buf, residual_buf_bytes,
          stream, ctypes.byref(out))
    return out.value


def ar_column_wrap(desc, major_buf, residual_buf) -> int:
    out = ctypes.c_void_p()
    _call("ar_column_wrap", ctypes.byref(desc), major_buf, residual_buf, ctypes.byref(out))
    return out.value


def ar_column_get_desc(col) -> ColumnDesc:
    desc = ColumnDesc()
    _call("ar_column_get_desc", col, ctypes.byref(desc))
    return desc


def ar_column_free(col):
    load().ar_column_free(col)


def ar_select_ws_bytes(n) -> int:
    return int(load().ar_select_ws_bytes(n))


def ar_refine_ws_bytes(capacity) -> int:
    return int(load().ar_refine_ws_bytes(capacity))


def _preds(preds):
    """preds: sequence of (column_handle, lo, hi)."""
    arr = (Pred * max(1, len(preds)))()
    for i, (c, lo, hi) in enumerate(preds):
        arr[i].col, arr[i].lo, arr[i].hi = c, lo, hi
    return arr


def _handles(cols):
    return (ctypes.c_void_p * max(1, len(cols)))(*cols)


def ar_approx_select(preds, flags, cands: Cands, ws, ws_bytes, stream):
    _call("ar_approx_select", _preds(preds), len(preds), flags, ctypes.byref(cands), ws, ws_bytes, stream)


def ar_refine(cands: Cands, preds, out: Positions, ws, ws_bytes, stream):
    _call("ar_refine", ctypes.byref(cands), _preds(preds), len(preds), ctypes.byref(out), ws, ws_bytes, stream)


def ar_sum(pos: Positions, cols, out_sum_dev, stream):
    _call("ar_sum", ctypes.byref(pos), _handles(cols), len(cols), out_sum_dev, stream)


def ar_sum_approximate(cands: Cands, cols, out4_dev, stream):
    _call("ar_sum_approximate", ctypes.byref(cands), _handles(cols), len(cols), out4_dev, stream)


def ar_project(pos: Positions, col, mode, out_values_dev, stream):
    _call("ar_project", ctypes.byref(pos), col, mode, out_values_dev, stream)


def ar_minmax_ws_bytes(capacity: int) -> int:
    return int(load().ar_minmax_ws_bytes(capacity))


def ar_minmax(cands: Cands, preds, col, mode, out7_dev, ws, ws_bytes, stream):
    _call("ar_minmax", ctypes.byref(cands), _preds(preds), len(preds), col, mode, out7_dev, ws, ws_bytes, stream)


def ar_refine_group_sum(cands: Cands, preds, key, cols, ngroups, out_dev, stream):
    _call("ar_refine_group_sum", ctypes.byref(cands), _preds(preds), len(preds), key, _handles(cols), len(cols),
          ngroups, out_dev, stream)


def ar_refine_sum(cands: Cands, preds, cols, out_sum_dev, out_count_dev, stream):
    _call("ar_refine_sum", ctypes.byref(cands), _preds(preds), len(preds), _handles(cols), len(cols), out_sum_dev,
          out_count_dev, stream)


def ar_select_refine_sum(preds, cols, out_dev, stream):
    _call("ar_select_refine_sum", _preds(preds), len(preds), _handles(cols), len(cols), out_dev, stream)


def ar_select_refine_sum_ws_bytes() -> int:
    return int(load().ar_select_refine_sum_ws_bytes())


def ar_select_refine_sum_ws(preds, cols, flags, out_dev, ws, ws_bytes, stream):
    _call("ar_select_refine_sum_ws", _preds(preds), len(preds), _handles(cols), len(cols), flags, out_dev, ws,
          ws_bytes, stream)


def ar_dist_unique_id_bytes() -> int:
    return int(load().ar_dist_unique_id_bytes())


def ar_dist_get_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(ar_dist_unique_id_bytes())
    _call("ar_dist_get_unique_id", ctypes.cast(buf, ctypes.c_void_p))
    return buf.raw


def ar_dist_init(unique_id: bytes, rank: int, world: int) -> int:
    out = ctypes.c_void_p()
    buf = ctypes.create_string_buffer(unique_id, len(unique_id))
    _call("ar_dist_init", ctypes.byref(out), ctypes.cast(buf, ctypes.c_void_p), rank, world)
    return out.value


def ar_dist_offsets(d, local_count_dev, all_counts_dev, global_offset_dev, stream):
    _call("ar_dist_offsets", d, local_count_dev, all_counts_dev, global_offset_dev, stream)


def ar_dist_sum(d, values_dev, n, stream):
    _call("ar_dist_sum", d, values_dev, n, stream)


def ar_dist_free(d):
    load().ar_dist_free(d)


def ar_dist_shard_range(n: int, world: int, rank: int):
    """(row0, rows) of rank's shard (host only)."""
    row0, rows = ctypes.c_int64(0), ctypes.c_int64(0)
    _call("ar_dist_shard_range", n, world, rank, ctypes.byref(row0), ctypes.byref(rows))
    return int(row0.value), int(rows.value)


def ar_dist_exclusive_offsets(all_counts_dev, world, rank, global_offset_dev, total_dev, stream):
    _call("ar_dist_exclusive_offsets", all_counts_dev, world, rank, global_offset_dev, total_dev, stream)


def ar_dist_concat_positions(local: Positions, row0, global_offset_dev, out_global, out_capacity, overflow_dev,
                             stream):
    _call("ar_dist_concat_positions", ctypes.byref(local), row0, global_offset_dev, out_global, out_capacity,
          overflow_dev, stream)


def ar_decompose_set_width(desc: ColumnDesc, w_major: int):
    _call("ar_decompose_set_width", ctypes.byref(desc), w_major)


def ar_group_table_bytes(slots: int) -> int:
    return int(load().ar_group_table_bytes(slots))


def ar_group_ids(rows: Positions, key, mode, table, table_slots, max_groups, gids_out, group_keys_out, ngroups_dev,
                 overflow_dev, stream):
    _call("ar_group_ids", ctypes.byref(rows), key, mode, table, table_slots, max_groups, gids_out, group_keys_out,
          ngroups_dev, overflow_dev, stream)


def ar_refine_group_sum_ids(cands: Cands, preds, gids, ngroups, cols, out_dev, stream):
    _call("ar_refine_group_sum_ids", ctypes.byref(cands), _preds(preds), len(preds), gids, ngroups, _handles(cols),
          len(cols), out_dev, stream)
