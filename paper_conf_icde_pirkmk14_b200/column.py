"""Torch plumbing around the C ABI: device / pinned buffers, streams, handles.

PyTorch only supplies memory and streams here; every step of the A&R path
runs in libar_b200.so.  Names follow the paper: a column is decomposed
(bwdecompose) into an approximation (major bits) and a
residual (minor bits); the approximate selection yields a candidate relation
(PAPER.md:368-374), the refinement the exact positions and
SUM(refine) the aggregate (Fig. 7).
"""
from __future__ import annotations

import numpy as np
import torch

from . import _ar
from ._ar import (AR_LAYOUT_PACKED, AR_LAYOUT_SLICED, AR_LOC_DEVICE, AR_LOC_HOST_PINNED,  # noqa: F401
                  AR_SELECT_CARRY_APPR, Cands, Positions)


def _stream(stream=None) -> int:
    s = stream if stream is not None else torch.cuda.current_stream()
    return s.cuda_stream


def _nbytes_tensor(nbytes: int, device, pinned: bool = False) -> torch.Tensor:
    nbytes = max(int(nbytes), 16)
    if pinned:
        return torch.empty(nbytes, dtype=torch.uint8, pin_memory=True)
    return torch.empty(nbytes, dtype=torch.uint8, device=device)


def as_u32_device(values, device="cuda") -> torch.Tensor:
    """uint32 / int32 numpy array or int32 tensor -> contiguous int32 CUDA tensor holding the same bits."""
    if isinstance(values, np.ndarray):
        if values.dtype == np.int32:
            values = values.view(np.uint32)
        values = torch.from_numpy(np.ascontiguousarray(values, dtype=np.uint32).view(np.int32))
    return values.to(device=device, dtype=torch.int32).contiguous()


class BWDColumn:
    """A bitwise-decomposed column (major part in HBM, residual in HBM or pinned host memory).

    signed=True decomposes int32 values in the order-preserving key domain v ^ 0x80000000 (predicate
    bounds are then int32 values); base="min" is the frame-of-reference prefix base min(key).
    width_agree: for a row shard of a larger table, a callable mapping this shard's planned stored
    width w_M to the table's (e.g. an allreduce-MAX over ranks); the descriptor is widened to it
    (ar_decompose_set_width) so every shard shares one bucket geometry.
    split=h: the residual in the split layout, its h high planes stored apart (AR_DECOMPOSE_SPLIT)."""

    def __init__(self, values, major_bits: int, layout: int = AR_LAYOUT_SLICED,
                 residual_loc: int = AR_LOC_DEVICE, base=0, signed: bool = False, device="cuda", stream=None,
                 width_agree=None, split: int = 0, _wrap=None):
        self.device = torch.device(device)
        if _wrap is not None:
            self.desc, self.major, self.residual = _wrap
            self.handle = _ar.ar_column_wrap(self.desc, self.major.data_ptr(),
                                             self.residual.data_ptr() if self.desc.residual_bytes else None)
            return
        col = as_u32_device(values, self.device)
        s = _stream(stream)
        ws = torch.empty(_ar.ar_decompose_ws_bytes(), dtype=torch.uint8, device=self.device)
        n = col.numel()
        flags = (_ar.AR_DECOMPOSE_SIGNED if signed else 0) | (_ar.AR_DECOMPOSE_BASE_MIN if base == "min" else 0) \
            | _ar.AR_DECOMPOSE_SPLIT(split)
        self.desc = _ar.ar_decompose_plan(col.data_ptr() if n else None, n, major_bits, layout, residual_loc,
                                          0 if base == "min" else int(base), flags, ws.data_ptr(), ws.numel(), s)
        if width_agree is not None:
            w = int(width_agree(int(self.desc.w_major)))
            if w != self.desc.w_major:
                _ar.ar_decompose_set_width(self.desc, w)
        self.major = _nbytes_tensor(self.desc.major_bytes, self.device)
        self.residual = _nbytes_tensor(self.desc.residual_bytes, self.device,
                                       pinned=(residual_loc == AR_LOC_HOST_PINNED))
        self.handle = _ar.ar_decompose(col.data_ptr() if n else None, self.desc, self.major.data_ptr(),
                                       self.major.numel(), self.residual.data_ptr(), self.residual.numel(), s)
        torch.cuda.current_stream(self.device).synchronize() if stream is None else stream.synchronize()
        del col

    # -- metadata (decomposition + compression base)
    @property
    def n(self) -> int:
        return int(self.desc.n)

    @property
    def k(self) -> int:
        return int(self.desc.k)

    @property
    def w_major(self) -> int:
        return int(self.desc.w_major)

    def nbytes(self) -> dict:
        return {"major": int(self.desc.major_bytes), "residual": int(self.desc.residual_bytes)}

    def copy(self, major_loc=None, residual_loc=None) -> "BWDColumn":
        """A second handle over copies of the buffers, optionally moved between HBM and pinned host
        memory (used to rotate inputs past L2, and for host-resident parts)."""
        def place(t, loc):
            if loc == AR_LOC_HOST_PINNED:
                return t.cpu().pin_memory()
            return t.to(self.device).clone() if t.device.type == "cuda" else t.to(self.device)
        mloc = self.desc.major_loc if major_loc is None else major_loc
        rloc = self.desc.residual_loc if residual_loc is None else residual_loc
        desc = _ar.ColumnDesc.from_buffer_copy(self.desc)
        desc.major_loc, desc.residual_loc = mloc, rloc
        return BWDColumn(None, 0, _wrap=(desc, place(self.major, mloc), place(self.residual, rloc)), device=self.device)

    def free(self):
        if getattr(self, "handle", None):
            _ar.ar_column_free(self.handle)
            self.handle = None

    def __del__(self):
        try:
            self.free()
        except Exception:
            pass


class CandidateList:
    """Device buffers of an ar_cands (positions, aux words, count)."""

    def __init__(self, capacity: int, device="cuda"):
        cap = max(int(capacity), 1)
        self.pos = torch.empty(cap + 8, dtype=torch.int32, device=device)
        self.aux = torch.empty(cap + 8, dtype=torch.int32, device=device)
        self.count_t = torch.zeros(1, dtype=torch.int64, device=device)
        self.c = Cands(self.pos.data_ptr(), self.aux.data_ptr(), self.count_t.data_ptr(), int(capacity), 0, 0)

    def count(self) -> int:
        return int(self.count_t.item())

    def positions(self) -> np.ndarray:
        n = self.count()
        return self.pos[:n].cpu().numpy().view(np.uint32).astype(np.int64)

    def aux_words(self) -> np.ndarray:
        n = self.count()
        return self.aux[:n].cpu().numpy().view(np.uint32)

    def definite(self) -> np.ndarray:
        return (self.aux_words() & _ar.AR_AUX_DEFINITE) != 0


class PositionList:
    def __init__(self, capacity: int, device="cuda"):
        cap = max(int(capacity), 1)
        self.pos = torch.empty(cap + 8, dtype=torch.int32, device=device)
        self.count_t = torch.zeros(1, dtype=torch.int64, device=device)
        self.p = Positions(self.pos.data_ptr(), self.count_t.data_ptr(), int(capacity))

    def count(self) -> int:
        return int(self.count_t.item())

    def positions(self) -> np.ndarray:
        n = self.count()
        return self.pos[:n].cpu().numpy().view(np.uint32).astype(np.int64)


def _pred_tuples(preds):
    return [(c.handle, int(lo), int(hi)) for c, lo, hi in preds]


class Workspace:
    """Caller-owned device workspace (the library never allocates device memory)."""

    def __init__(self, nbytes: int, device="cuda"):
        self.t = torch.empty(max(int(nbytes), 16), dtype=torch.uint8, device=device)

    @property
    def ptr(self):
        return self.t.data_ptr()

    @property
    def nbytes(self):
        return self.t.numel()


def approx_select(preds, cands: CandidateList, ws: Workspace, carry: bool = True, stream=None):
    """Steps a2+a3: preds = [(BWDColumn, lo, hi), ...] -> candidate relation in `cands`."""
    _ar.ar_approx_select(_pred_tuples(preds), AR_SELECT_CARRY_APPR if carry else 0, cands.c, ws.ptr, ws.nbytes,
                         _stream(stream))


def refine(cands: CandidateList, preds, out: PositionList, ws: Workspace, stream=None):
    """Step a5 (Algorithm 2): candidate relation -> exact ascending positions."""
    _ar.ar_refine(cands.c, _pred_tuples(preds), out.p, ws.ptr, ws.nbytes, _stream(stream))


def sum_at(pos: PositionList, cols, out: torch.Tensor, stream=None):
    """Step a6: out[0] = SUM over pos of prod(cols)."""
    _ar.ar_sum(pos.p, [c.handle for c in cols], out.data_ptr(), _stream(stream))


def sum_approximate(cands: CandidateList, cols, out4: torch.Tensor, stream=None):
    """bwd.sumapproximate (Fig. 7): out4 = [SUM lower bound, SUM upper bound, |definite|, |candidates|]
    from the candidate relation and the majors of `cols` only (no residual is read)."""
    _ar.ar_sum_approximate(cands.c, [c.handle for c in cols], out4.data_ptr(), _stream(stream))


def project(pos, col: BWDColumn, exact: bool = True, stream=None) -> torch.Tensor:
    """bwd.leftjoinrefine (exact values) / bwd.leftjoinapproximate (bucket minima) of `col` at the rows of
    a PositionList or CandidateList; returns a device int32 tensor (uint32 bits) of its capacity."""
    if isinstance(pos, CandidateList):
        p = Positions(pos.pos.data_ptr(), pos.count_t.data_ptr(), pos.c.capacity)
    else:
        p = pos.p
    out = torch.empty(max(int(p.capacity), 1), dtype=torch.int32, device=col.device)
    _ar.ar_project(p, col.handle, _ar.AR_PROJECT_EXACT if exact else _ar.AR_PROJECT_APPROX, out.data_ptr(),
                   _stream(stream))
    return out


def minmax(cands: CandidateList, preds, col: BWDColumn, mode: str, out7: torch.Tensor, ws: "Workspace" = None,
           stream=None):
    """MIN / MAX of `col` over the refined rows (s IV-F, Fig. 6): out7 = [answer, survivors, approx lower,
    approx upper, candidates refined, |definite|, |candidates|]."""
    ws = ws if ws is not None else Workspace(_ar.ar_minmax_ws_bytes(cands.c.capacity), col.device)
    _ar.ar_minmax(cands.c, _pred_tuples(preds), col.handle, _ar.AR_MIN if mode == "min" else _ar.AR_MAX,
                  out7.data_ptr(), ws.ptr, ws.nbytes, _stream(stream))


def refine_group_sum(cands: CandidateList, preds, key: BWDColumn, cols, ngroups: int, stream=None) -> torch.Tensor:
    """Grouped COUNT / SUM over the refined rows (s IV-E/F): returns a device int64 tensor [2, ngroups]
    (row 0: SUM(prod(cols)) per key value, row 1: COUNT)."""
    out = torch.empty(2 * ngroups, dtype=torch.int64, device=key.device)
    _ar.ar_refine_group_sum(cands.c, _pred_tuples(preds), key.handle, [c.handle for c in cols], ngroups,
                            out.data_ptr(), _stream(stream))
    return out.view(2, ngroups)


def refine_sum(cands: CandidateList, preds, cols, out_sum: torch.Tensor, out_count: torch.Tensor = None,
               stream=None):
    """Steps a5+a6 fused: out_sum[0] = SUM(prod(cols)) over the refined rows, out_count[0] = their number."""
    _ar.ar_refine_sum(cands.c, _pred_tuples(preds), [c.handle for c in cols], out_sum.data_ptr(),
                      out_count.data_ptr() if out_count is not None else None, _stream(stream))


def select_refine_sum(preds, cols, out4: torch.Tensor, stream=None, ws: "Workspace" = None, flags: int = 0):
    """Steps a3+a5+a6 in one pass: out4 = [SUM, |result|, |candidates|, |definite|].  With a workspace
    (SrsWorkspace) the call is one kernel launch, optionally a programmatic dependent one (flags)."""
    if ws is None:
        _ar.ar_select_refine_sum(_pred_tuples(preds), [c.handle for c in cols], out4.data_ptr(), _stream(stream))
    else:
        _ar.ar_select_refine_sum_ws(_pred_tuples(preds), [c.handle for c in cols], flags, out4.data_ptr(), ws.ptr,
                                    ws.nbytes, _stream(stream))


def SrsWorkspace(device="cuda") -> "Workspace":
    """Workspace of ar_select_refine_sum_ws: zeroed once here (the ticket word), left zero by every call."""
    w = Workspace(_ar.ar_select_refine_sum_ws_bytes(), device)
    w.t.zero_()
    return w


class Grouping:
    """Output of the approximation group operator (ar_group_ids, s IV-E): per-row group ids aligned with
    a position list, the grouping value of every id, the number of groups and the overflow flags."""

    def __init__(self, capacity: int, max_groups: int, device="cuda"):
        slots = 1
        while slots < 2 * max_groups:
            slots <<= 1
        self.max_groups, self.slots = int(max_groups), slots
        self.table = torch.empty(max(_ar.ar_group_table_bytes(slots), 16), dtype=torch.uint8, device=device)
        self.gids = torch.empty(max(int(capacity), 1) + 8, dtype=torch.int32, device=device)
        self.keys = torch.empty(max_groups, dtype=torch.int32, device=device)
        self.ngroups_t = torch.zeros(1, dtype=torch.int64, device=device)
        self.overflow_t = torch.zeros(1, dtype=torch.int32, device=device)

    def ngroups(self) -> int:
        return int(self.ngroups_t.item())

    def overflow(self) -> int:
        return int(self.overflow_t.item())

    def group_keys(self) -> np.ndarray:
        g = min(self.ngroups(), self.max_groups)
        return self.keys[:g].cpu().numpy().view(np.uint32)


def group_ids(rows, key: BWDColumn, grouping: Grouping, exact: bool = False, stream=None) -> Grouping:
    """The approximation group operator over the rows of a CandidateList or PositionList: hash-assigned
    dense group ids of the key's approximate (bucket minimum) or exact values, aligned with the rows."""
    if isinstance(rows, CandidateList):
        p = Positions(rows.pos.data_ptr(), rows.count_t.data_ptr(), rows.c.capacity)
    else:
        p = rows.p
    _ar.ar_group_ids(p, key.handle, _ar.AR_GROUP_EXACT if exact else _ar.AR_GROUP_APPROX, grouping.table.data_ptr(),
                     grouping.slots, grouping.max_groups, grouping.gids.data_ptr(), grouping.keys.data_ptr(),
                     grouping.ngroups_t.data_ptr(), grouping.overflow_t.data_ptr(), _stream(stream))
    return grouping


def refine_group_sum_ids(cands: CandidateList, preds, grouping: Grouping, cols, stream=None) -> torch.Tensor:
    """Grouped COUNT / SUM over the refined rows by the ids of `grouping` (aligned with `cands`): returns a
    device int64 tensor [2, max_groups] (row 0: SUM(prod(cols)) per id, row 1: COUNT)."""
    G = grouping.max_groups
    out = torch.empty(2 * G, dtype=torch.int64, device=grouping.gids.device)
    _ar.ar_refine_group_sum_ids(cands.c, _pred_tuples(preds), grouping.gids.data_ptr(), G, [c.handle for c in cols],
                                out.data_ptr(), _stream(stream))
    return out.view(2, G)
