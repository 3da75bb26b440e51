#!/usr/bin/env python
"""bench.py -- A&R select+refine rows/s (Q6-shaped) on B200, one process per GPU.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference] [--variant staged|fused]
    torchrun --nproc-per-node N --master-addr 127.0.0.1 bench.py --gpus N ...

Workload (BASELINE.json configs[1], "C2"): TPC-H SF10-shaped lineitem Q6 per GPU,
60 M rows: l_shipdate decomposed 24 GPU / 8 residual bits,
l_discount, l_quantity bit-packed with k = 0, l_extendedprice packed for the
gather; predicates shipdate in [731,1095], discount in [5,7], quantity <= 23;
SUM(l_extendedprice * l_discount).  With N GPUs each rank holds its own
60 M-row range of an SF(10 N) table (weak scaling) and the step adds the count
allgather (a4) and the int64 SUM allreduce over NCCL.

One step = one pass of the whole hot path over the batch.  Headline
(`--variant fused`, default): ar_select_refine_sum, the one-pass kernel that
runs a2+a3 (approximate select, candidate relation compacted per warp in shared
memory), a5 (refine) and a6 (SUM), then (N > 1) the SUM allreduce.  The staged
pipeline is timed in the same run and reported under "variants": a2+a3
ar_approx_select with the ordered candidate list in HBM, a4 count allgather
(N > 1), a5+a6 ar_refine_sum.
Inputs are resident in HBM; R copies of the decomposed columns are rotated so
consecutive steps never re-read L2-resident data (R x 345 MB > 126 MB L2).
The K timed steps are one CUDA-graph replay bracketed by CUDA events on the
launching stream.  The fused step is one kernel launch (ar_select_refine_sum_ws,
a programmatic dependent of the previous step's kernel), so at N = 1 its
per-launch duration is the step time; per-kernel durations of the staged
pipeline come from a second replay with CUDA events between the calls.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
if ROOT not in sys.path:
    sys.path.insert(0, ROOT)

import datagen  # noqa: E402

METRIC = "A&R select+refine rows/s (Q6-shaped) at 1/2/4/8 B200; % of HBM roofline"
UNIT = "rows/s"
SF_PER_GPU = 10
SEED = 2
PREDS = [datagen.Q6_SHIPDATE, datagen.Q6_DISCOUNT, datagen.Q6_QUANTITY]
SECTOR = 32


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=1000)
    ap.add_argument("--warmup", type=int, default=10)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--variant", choices=["staged", "fused"], default="fused",
                    help="headline variant (the other one is timed too and reported under 'variants')")
    ap.add_argument("--only", action="store_true", help="time the headline variant only")
    ap.add_argument("--sf", type=float, default=SF_PER_GPU, help="scale factor per GPU")
    ap.add_argument("--copies", type=int, default=3, help="rotated input copies (L2 defeat)")
    ap.add_argument("--e2e-steps", type=int, default=10)
    ap.add_argument("--cpu-seconds", type=float, default=10.0)
    ap.add_argument("--no-cpu", action="store_true")
    return ap.parse_args()


def dist_env():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


def workload(args, world, rank):
    rows = int(round(args.sf * datagen.ROWS_PER_SF))
    table_sf = args.sf * world
    cols = datagen.q6_columns(SEED, table_sf, n=rows, row0=rank * rows)
    return rows, table_sf, cols


def config_dict(args, world, rows, extra=None):
    d = {"workload": f"C2: TPC-H SF{args.sf:g}-shaped lineitem Q6 per GPU ({rows} rows; table SF{args.sf * world:g}"
                     f" row-sharded over {world} GPU(s))",
         "rows_per_gpu": rows, "rows_total": rows * world,
         "decomposition": "l_shipdate 24 GPU/8 residual bits; l_discount, l_quantity, l_extendedprice k=0",
         "predicates": "shipdate in [731,1095], discount in [5,7], quantity in [0,23]; SUM(extendedprice*discount)",
         "parallelism": f"rowshard{world}"}
    if extra:
        d.update(extra)
    return d


# ----------------------------------------------------------------- CPU oracle leg

def run_oracle(cols, rows, seconds, threads=0):
    import oracle
    values = [cols["shipdate"], cols["discount"], cols["quantity"]]
    los = [p[0] for p in PREDS]
    his = [p[1] for p in PREDS]
    aggs = [cols["extprice"], cols["discount"]]
    t0 = time.perf_counter()
    _, cnt, s = oracle.select_sum(values, los, his, aggs, threads=threads, positions=True)
    t1 = time.perf_counter() - t0
    reps = max(1, min(200, int(math.ceil(seconds / max(t1, 1e-6)))))
    times = [t1]
    for _ in range(reps - 1):
        t0 = time.perf_counter()
        oracle.select_sum(values, los, his, aggs, threads=threads, positions=True)
        times.append(time.perf_counter() - t0)
    med = statistics.median(times)
    used = threads if threads > 0 else oracle.default_threads()
    return {"value": rows / med, "unit": UNIT, "cores": used, "kind": "oracle",
            "sample": f"full per-GPU table ({rows} rows), exact select + SUM with positions, median of {len(times)}"
                      f" runs ({sum(times):.1f} s)", "count": cnt, "sum": s}


def reference_arm(args):
    world, rank, _ = dist_env()
    if rank != 0:
        return
    rows, table_sf, cols = workload(args, 1, 0)
    # each step = one oracle pass over the workload; K steps after W warm-ups, bounded by time
    import oracle
    values = [cols["shipdate"], cols["discount"], cols["quantity"]]
    los, his = [p[0] for p in PREDS], [p[1] for p in PREDS]
    aggs = [cols["extprice"], cols["discount"]]
    steps, warm = max(1, min(args.steps, 20)), max(0, min(args.warmup, 3))
    for _ in range(warm):
        oracle.select_sum(values, los, his, aggs, threads=0)
    t0 = time.perf_counter()
    for _ in range(steps):
        oracle.select_sum(values, los, his, aggs, threads=0)
    dt = time.perf_counter() - t0
    val = rows * steps / dt
    line = {"impl": "reference", "metric": METRIC, "value": val, "unit": UNIT, "n_gpus": args.gpus,
            "steps": steps, "warmup": warm, "ms_per_step": dt / steps * 1e3, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "u32", "data": "synthetic",
            "config": config_dict(args, 1, rows),
            "cpu_baseline": {"value": val, "unit": UNIT, "cores": oracle.default_threads(), "kind": "oracle",
                             "sample": f"{steps} oracle passes over the per-GPU table ({rows} rows)"},
            "e2e": {"value": val, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ------------------------------------------------------------------ clocks (NVML)

class ClockSampler:
    """Samples SM clock and throttle reasons through NVML (the library nvidia-smi reads) every ~2 ms."""

    def __init__(self, index):
        self.samples, self.reasons, self.stop_flag = [], set(), False
        self.ok = False
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            nv = pynvml
            # built here, not in the sampling thread, so the first sample is taken at once
            self.names = {getattr(nv, k): k.replace("nvmlClocksEventReason", "").replace("nvmlClocksThrottleReason", "")
                          for k in dir(nv)
                          if (k.startswith("nvmlClocksEventReason") or k.startswith("nvmlClocksThrottleReason"))
                          and isinstance(getattr(nv, k), int)
                          and k not in ("nvmlClocksEventReasonAll", "nvmlClocksThrottleReasonAll")}
            nv.nvmlDeviceGetClockInfo(self.h, nv.NVML_CLOCK_SM)
            nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
            self.ok = True
        except Exception as e:  # pragma: no cover
            self.err = str(e)

    def _run(self):
        nv, names = self.nv, self.names
        while not self.stop_flag:
            try:
                self.samples.append(nv.nvmlDeviceGetClockInfo(self.h, nv.NVML_CLOCK_SM))
                r = nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
                for bit, name in names.items():
                    if bit and (r & bit) == bit and name not in ("None", "GpuIdle"):
                        self.reasons.add(_snake(name))
            except Exception:
                pass
            time.sleep(0.002)

    def __enter__(self):
        if self.ok:
            self.t = threading.Thread(target=self._run, daemon=True)
            self.t.start()
        return self

    def __exit__(self, *a):
        self.stop_flag = True
        if self.ok:
            self.t.join()

    def result(self):
        if not self.ok or not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": getattr(self, "max_mhz", None), "reasons": [],
                    "samples": 0, "source": "nvml"}
        return {"sm_mhz": statistics.median(self.samples), "sm_max_mhz": self.max_mhz,
                "reasons": sorted(self.reasons), "samples": len(self.samples), "source": "nvml"}


def _snake(s):
    out = ""
    for ch in s:
        out += ("_" + ch.lower()) if ch.isupper() and out else ch.lower()
    return out


# -------------------------------------------------------------- algorithmic bytes

def algorithmic_bytes(cols, rows, k_ship=8):
    """Bytes the method must move per query: packed scans + sector-granular gathers + output."""
    sd, dc, qt, ep = cols["shipdate"], cols["discount"], cols["quantity"], cols["extprice"]
    w_sd = int((int(sd.max()) >> k_ship)).bit_length()
    w_dc, w_qt, w_ep = int(dc.max()).bit_length(), int(qt.max()).bit_length(), int(ep.max()).bit_length()
    scan = rows * (w_sd + w_dc + w_qt) / 8.0
    major = sd >> k_ship
    lo, hi = PREDS[0]
    cand_sd = (major >= (lo >> k_ship)) & (major <= (hi >> k_ship))
    def_sd = (major >= ((lo + 255) >> 8)) & (major <= (((hi + 1) >> 8) - 1))
    other = (dc >= PREDS[1][0]) & (dc <= PREDS[1][1]) & (qt >= PREDS[2][0]) & (qt <= PREDS[2][1])
    cand = cand_sd & other
    nondef = cand & ~def_sd
    result = other & (sd >= lo) & (sd <= hi)
    idx_nd = np.nonzero(nondef)[0].astype(np.int64)
    idx_res = np.nonzero(result)[0].astype(np.int64)
    res_sectors = np.unique((idx_nd * k_ship) // (SECTOR * 8)).size
    # a 24-bit packed value may straddle two sectors
    b0 = idx_res * w_ep
    ep_sectors = np.unique(np.concatenate([b0 // (SECTOR * 8), (b0 + w_ep - 1) // (SECTOR * 8)])).size
    gathered = min(rows * k_ship / 8.0, SECTOR * res_sectors) + min(rows * w_ep / 8.0, SECTOR * ep_sectors)
    ncand = int(cand.sum())
    res64 = np.unique((idx_nd * k_ship) // (64 * 8)).size
    ep64 = np.unique(np.concatenate([b0 // (64 * 8), (b0 + w_ep - 1) // (64 * 8)])).size
    return {"scan": scan, "gather": gathered, "zero_copy_64": 64.0 * (res64 + ep64), "residual_sectors": int(res_sectors), "ep_sectors": int(ep_sectors),
            "total": scan + gathered + 8.0, "n_cand": ncand, "n_def": int((cand & def_sd).sum()),
            "n_result": int(result.sum()), "cand_list_bytes": 8.0 * ncand,
            "widths": {"shipdate_major": w_sd, "discount": w_dc, "quantity": w_qt, "extprice": w_ep}}


# ----------------------------------------------------------------------- our arm

def ours(args):
    import torch
    from paper_conf_icde_pirkmk14_b200 import _ar, column as cu
    from cuda.bindings import driver as drv

    world, rank, local = dist_env()
    if world != args.gpus and world > 1:
        raise SystemExit(f"--gpus {args.gpus} but WORLD_SIZE {world}")
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    pg = None
    dist_h = None
    if world > 1:
        import torch.distributed as tdist
        tdist.init_process_group("nccl", device_id=dev)
        pg = tdist
        uid = _ar.ar_dist_get_unique_id() if rank == 0 else b""
        obj = [uid]
        tdist.broadcast_object_list(obj, src=0)
        dist_h = _ar.ar_dist_init(obj[0], rank, world)

    rows, table_sf, cols = workload(args, world, rank)
    # decompose once (untimed): bwdecompose(l_shipdate, 24); the rest are bit-packed whole (k = 0)
    base = [cu.BWDColumn(cols["shipdate"], 24), cu.BWDColumn(cols["discount"], 32),
            cu.BWDColumn(cols["quantity"], 32), cu.BWDColumn(cols["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)]
    copies = [base] + [[c.copy() for c in base] for _ in range(max(0, args.copies - 1))]
    bytes_per_copy = sum(c.nbytes()["major"] + c.nbytes()["residual"] for c in base)
    torch.cuda.synchronize()

    stream = torch.cuda.Stream(device=dev)
    s_ptr = stream.cuda_stream
    cands = cu.CandidateList(rows, device=dev)
    ws_sel = cu.Workspace(_ar.ar_select_ws_bytes(rows), device=dev)
    out = torch.zeros(4, dtype=torch.int64, device=dev)        # SUM, |result|, (fused: |cand|, |def|)
    # one-pass query stream: the workspace call is a single launch per step (out written, not
    # accumulated) and a programmatic dependent of the previous step's kernel; the columns are
    # immutable, so its tile loads may start while that kernel drains (AR_SRS_PDL_EARLY_READ)
    srs_ws = cu.SrsWorkspace(device=dev)
    srs_flags = _ar.AR_SRS_PDL_EARLY_READ
    counts = torch.zeros(world, dtype=torch.int64, device=dev)
    goff = torch.zeros(1, dtype=torch.int64, device=dev)

    def preds_of(cs):
        return [(cs[0].handle, *PREDS[0]), (cs[1].handle, *PREDS[1]), (cs[2].handle, *PREDS[2])]

    pred_sets = [preds_of(cs) for cs in copies]
    agg_sets = [[cs[3].handle, cs[1].handle] for cs in copies]

    def new_event():
        err, e = drv.cuEventCreate(drv.CUevent_flags.CU_EVENT_DEFAULT)
        assert err == drv.CUresult.CUDA_SUCCESS, err
        return e

    def rec(e):
        err, = drv.cuEventRecordWithFlags(e, s_ptr, drv.CUevent_record_flags.CU_EVENT_RECORD_EXTERNAL)
        assert err == drv.CUresult.CUDA_SUCCESS, err

    def elapsed(a, b):
        err, ms = drv.cuEventElapsedTime(a, b)
        assert err == drv.CUresult.CUDA_SUCCESS, err
        return ms

    def step(variant, i, ev=None):
        """One pass of the hot path on copy i % R; ev = events recorded around each kernel."""
        r = i % len(copies)
        if variant == "staged":
            if ev is not None:
                rec(ev[0])
            _ar.ar_approx_select(pred_sets[r], _ar.AR_SELECT_CARRY_APPR, cands.c, ws_sel.ptr, ws_sel.nbytes, s_ptr)
            if ev is not None:
                rec(ev[1])
            if dist_h:
                _ar.ar_dist_offsets(dist_h, cands.count_t.data_ptr(), counts.data_ptr(), goff.data_ptr(), s_ptr)
            if ev is not None:
                rec(ev[2])
            _ar.ar_refine_sum(cands.c, pred_sets[r], agg_sets[r], out.data_ptr(), out.data_ptr() + 8, s_ptr)
            if ev is not None:
                rec(ev[3])
            if dist_h:
                _ar.ar_dist_sum(dist_h, out.data_ptr(), 2, s_ptr)
        else:
            if ev is not None:
                rec(ev[0])
            _ar.ar_select_refine_sum_ws(pred_sets[r], agg_sets[r], srs_flags, out.data_ptr(), srs_ws.ptr,
                                        srs_ws.nbytes, s_ptr)
            if ev is not None:
                rec(ev[1])
            if dist_h:
                _ar.ar_dist_sum(dist_h, out.data_ptr(), 4, s_ptr)

    # the one-pass call launches the result-ring kernel where it applies (fused.cu), else the
    # general one (select.cu); ask the library which one ran
    with torch.cuda.stream(stream):
        step("fused", 0)
    stream.synchronize()
    fused_name = _ar.ar_last_scan_kernel() or "fused_kernel"
    with torch.cuda.stream(stream):
        step("staged", 0)
    stream.synchronize()
    ref_name = _ar.ar_last_scan_kernel() or "refine_sum_kernel"   # the specialised or the general refine+SUM
    SEL = "select_tile_kernel+compact_kernel"   # ar_approx_select: two launches (+ memsets)
    KERNELS = {"staged": ["select_tile_kernel", "compact_kernel", ref_name]
               + (["exclusive_offset_kernel"] if dist_h else []),
               "fused": [fused_name]}
    K = args.steps

    def time_variant(variant, sampler=None):
        # eager warm-up (also primes the library's attribute / occupancy caches before capture)
        with torch.cuda.stream(stream):
            for i in range(max(3, args.warmup)):
                step(variant, i)
        stream.synchronize()
        n_ev = 4 if variant == "staged" else 2
        evs = [[new_event() for _ in range(n_ev)] for _ in range(K)]
        # the headline graph has no event nodes between steps (they would serialise the
        # programmatic dependent launches); a second graph with events gives per-kernel durations
        g_warm, g_timed, g_ev = torch.cuda.CUDAGraph(), torch.cuda.CUDAGraph(), torch.cuda.CUDAGraph()
        with torch.cuda.graph(g_warm, stream=stream, capture_error_mode="relaxed"):
            for i in range(args.warmup):
                step(variant, i)
        with torch.cuda.graph(g_timed, stream=stream, capture_error_mode="relaxed"):
            for i in range(K):
                step(variant, i + args.warmup)
        with torch.cuda.graph(g_ev, stream=stream, capture_error_mode="relaxed"):
            for i in range(K):
                step(variant, i + args.warmup, evs[i])
        torch.cuda.synchronize()
        t0, t1 = new_event(), new_event()
        with torch.cuda.stream(stream):
            g_warm.replay()
            stream.synchronize()
            if pg:
                pg.barrier()
            torch.cuda.synchronize()
            ctx = sampler if sampler is not None else _Null()
            with ctx:
                drv.cuEventRecord(t0, s_ptr)
                g_timed.replay()
                drv.cuEventRecord(t1, s_ptr)
                stream.synchronize()
        torch.cuda.synchronize()
        with torch.cuda.stream(stream):
            g_ev.replay()
            stream.synchronize()
        torch.cuda.synchronize()
        if pg:
            pg.barrier()
        ms_total = elapsed(t0, t1)
        if pg:
            t = torch.tensor([ms_total], dtype=torch.float64, device=dev)
            pg.all_reduce(t, op=pg.ReduceOp.MAX)
            ms_total = float(t.item())
        if variant == "staged":
            kern = {SEL: [elapsed(e[0], e[1]) for e in evs],
                    ref_name: [elapsed(e[2], e[3]) for e in evs]}
        else:
            kern = {fused_name: [elapsed(e[0], e[1]) for e in evs]}
        res = out.cpu().tolist()
        del g_warm, g_timed, g_ev
        kern_ms = {k: statistics.mean(v) for k, v in kern.items()}
        if variant == "fused" and world == 1:
            # the step is exactly one kernel launch: its steady-state duration is the step time
            # (the evented graph's isolated launch time is kept alongside)
            kern_ms = {fused_name: ms_total / K, fused_name + " (isolated launch)": kern_ms[fused_name]}
        return ms_total, kern_ms, res

    ab = algorithmic_bytes(cols, rows)
    peaks = {}
    try:
        peaks = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))
    except Exception:
        pass
    hbm_peak = peaks.get("hbm_gbs")
    peak_src = "measured (MEASURED_PEAKS.json hbm_gbs)" if hbm_peak else "fallback (B200_PROFILING.md 6.65 TB/s)"
    hbm_peak = hbm_peak or 6650.0
    per_kernel_bytes = {
        fused_name: ab["total"],                                            # majors + touched residual/ep sectors
        SEL: ab["scan"] + ab["cand_list_bytes"],                            # majors read + (pos, aux) written
        ref_name: ab["cand_list_bytes"] + ab["gather"] + 16.0,   # cands read + sector gathers + out
    }

    variants = [args.variant] + [v for v in ("fused", "staged") if v != args.variant and not args.only]
    results = {}
    sampler = ClockSampler(torch.cuda.current_device() if "CUDA_VISIBLE_DEVICES" not in os.environ else local)
    for v in variants:
        ms_total, kern_ms, res = time_variant(v, sampler if v == args.variant else None)
        ms_step = ms_total / K
        dom = max((k for k in kern_ms if k in per_kernel_bytes), key=lambda k: kern_ms[k])
        achieved = per_kernel_bytes[dom] / (kern_ms[dom] / 1e3) / 1e9
        results[v] = {
            "value": rows * world * K / (ms_total / 1e3), "ms_per_step": ms_step, "result": res,
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": hbm_peak, "unit": "GB/s",
                         "frac": achieved / hbm_peak, "traffic": None, "kernel": dom,
                         "algorithmic_bytes_per_launch": per_kernel_bytes[dom], "kernel_ms": kern_ms[dom],
                         "peak_source": peak_src,
                         "per_kernel": {k: {"ms": kern_ms[k], "bytes": per_kernel_bytes[k.split(" (")[0]],
                                            "gbs": per_kernel_bytes[k.split(" (")[0]] / (kern_ms[k] / 1e3) / 1e9}
                                        for k in kern_ms},
                         "step_bytes": ab["total"],
                         "step_frac": ab["total"] / (ms_step / 1e3) / 1e9 / hbm_peak},
            "gpu_launches": len(KERNELS[v]) * K, "gpu_kernels": KERNELS[v]}
    head = results[args.variant]
    traffic_file = os.path.join(ROOT, "profiles", "traffic.json")
    if os.path.exists(traffic_file):
        try:
            tr = json.load(open(traffic_file))
            for v in results:
                results[v]["roofline"]["traffic"] = tr.get(v, {}).get(results[v]["roofline"]["kernel"])
        except Exception:
            pass

    # e2e: the decomposed table at rest in pinned host memory.  Every step copies the
    # scanned major parts H2D (they are read in full), while the A&R refine and SUM read
    # only the residual sectors and l_extendedprice sectors they touch, zero-copy over the
    # host link (ar_column with host-resident parts); then the (SUM, count) result D2H.
    e2e = None
    if args.e2e_steps > 0:
        sd_e = base[0].copy(residual_loc=_ar.AR_LOC_HOST_PINNED)       # major in HBM, residual on host
        dc_e, qt_e = base[1].copy(), base[2].copy()
        ep_e = base[3].copy(major_loc=_ar.AR_LOC_HOST_PINNED)          # gathered column stays on host
        host_src = [(base[0].major.cpu().pin_memory(), sd_e.major), (base[1].major.cpu().pin_memory(), dc_e.major),
                    (base[2].major.cpu().pin_memory(), qt_e.major)]
        e_preds = [(sd_e.handle, *PREDS[0]), (dc_e.handle, *PREDS[1]), (qt_e.handle, *PREDS[2])]
        e_aggs = [ep_e.handle, dc_e.handle]
        res_host = torch.zeros(4, dtype=torch.int64).pin_memory()
        copied = sum(h.numel() for h, _ in host_src)
        zero_copy = ab["zero_copy_64"]
        for i in range(2):                                              # warm-up
            _ar.ar_select_refine_sum(e_preds, e_aggs, out.data_ptr(), s_ptr)
        with torch.cuda.stream(stream):
            if pg:
                pg.barrier()
            torch.cuda.synchronize()
            e0, e1 = new_event(), new_event()
            drv.cuEventRecord(e0, s_ptr)
            for i in range(args.e2e_steps):
                for h, d in host_src:
                    d.copy_(h, non_blocking=True)
                _ar.ar_select_refine_sum(e_preds, e_aggs, out.data_ptr(), s_ptr)
                if dist_h:
                    _ar.ar_dist_sum(dist_h, out.data_ptr(), 4, s_ptr)
                res_host.copy_(out, non_blocking=True)
            drv.cuEventRecord(e1, s_ptr)
            stream.synchronize()
        ms_e2e = elapsed(e0, e1)
        if pg:
            t = torch.tensor([ms_e2e], dtype=torch.float64, device=dev)
            pg.all_reduce(t, op=pg.ReduceOp.MAX)
            ms_e2e = float(t.item())
        e2e_ok = res_host.tolist()[:2] == head["result"][:2]
        e2e = {"value": rows * world * args.e2e_steps / (ms_e2e / 1e3), "unit": UNIT,
               "h2d_bytes_per_step": int(copied + zero_copy), "d2h_bytes_per_step": 32,
               "h2d_copied_bytes": int(copied), "h2d_zero_copy_bytes_64B": int(zero_copy),
               "ms_per_step": ms_e2e / args.e2e_steps, "result_matches_device_run": e2e_ok,
               "path": "decomposed table in pinned host memory; per step: cudaMemcpyAsync H2D of the scanned "
                       "majors (105 MB), ar_select_refine_sum reading the shipdate residual and l_extendedprice "
                       "zero-copy over the host link (only touched 64-B granules), D2H of (SUM, count)"}

    cpu = cpu1 = None
    if rank == 0 and world == 1 and not args.no_cpu:
        cpu = run_oracle(cols, rows, args.cpu_seconds)
        # and single-threaded (the paper's MonetDB baseline ran one thread)
        cpu1 = run_oracle(cols, rows, 0.0, threads=1)
        cpu1 = {k: v for k, v in cpu1.items() if k not in ("sum", "count")}

    if dist_h:
        _ar.ar_dist_free(dist_h)
    if rank != 0:
        if pg:
            pg.destroy_process_group()
        return
    parity = None
    if cpu is not None:
        parity = {"oracle_sum": cpu["sum"], "oracle_count": cpu["count"],
                  "gpu": {v: {"sum": results[v]["result"][0], "count": results[v]["result"][1]} for v in results},
                  "match": all(results[v]["result"][0] == cpu["sum"] and results[v]["result"][1] == cpu["count"]
                               for v in results)}
        cpu = {k: v for k, v in cpu.items() if k not in ("sum", "count")}
    other = {v: {k: results[v][k] for k in ("value", "ms_per_step", "roofline", "gpu_launches", "gpu_kernels")}
             for v in results if v != args.variant}
    line = {"metric": METRIC, "value": head["value"], "unit": UNIT, "n_gpus": world, "steps": K,
            "warmup": args.warmup, "ms_per_step": head["ms_per_step"], "higher_is_better": True, "scaling": "weak",
            "vs_baseline": None, "dtype": "u32", "data": "synthetic",
            "config": config_dict(args, world, rows, {
                "variant": args.variant,
                "variant_desc": VARIANT_DESC[args.variant],
                "l2": f"inputs rotated over {len(copies)} copies of the decomposed columns "
                      f"({len(copies)} x {bytes_per_copy / 1e6:.0f} MB > 126 MB L2)",
                "timing": "K steps = one CUDA-graph replay; CUDA events on the launching stream; max over ranks; "
                          "fused step = 1 launch of ar_select_refine_sum_ws (PDL, early input reads)"}),
            "roofline": head["roofline"], "cpu_baseline": cpu, "cpu_baseline_single_thread": cpu1, "e2e": e2e,
            "gpu_launches": head["gpu_launches"], "gpu_kernels": head["gpu_kernels"],
            "clocks": sampler.result(),
            "counts": {"candidates": ab["n_cand"], "definite": ab["n_def"], "result": ab["n_result"],
                       "gpu_result_count": head["result"][1], "gpu_sum": head["result"][0]},
            "parity": parity,
            "variants": other,
            "hbm_roofline_rows_per_s": hbm_peak * 1e9 / (ab["total"] / rows)}
    print(json.dumps(line), flush=True)
    if pg:
        pg.destroy_process_group()


class _Null:
    def __enter__(self):
        return self

    def __exit__(self, *a):
        return False


VARIANT_DESC = {
    "fused": "one pass: a3 approximate select (candidate relation compacted per warp in shared memory) + a5 refine "
             "+ a6 SUM in one kernel (ar_select_refine_sum)",
    "staged": "ar_approx_select (ordered candidate list in HBM) -> [a4 count allgather] -> ar_refine_sum",
}


def main():
    args = parse()
    if args.impl == "reference":
        reference_arm(args)
        return
    ours(args)


if __name__ == "__main__":
    main()
