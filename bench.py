#!/usr/bin/env python
"""bench.py -- A&R select+refine rows/s (Q6-shaped) on B200, one process per GPU.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
                    [--workload c4|c2] [--variant fused|staged] [--scaling strong|weak]
    torchrun --nproc-per-node N --master-addr 127.0.0.1 bench.py --gpus N ...

Headline workload (BASELINE.json configs[3], "C4", the metric's "at 1/2/4/8
B200" series): TPC-H SF100-shaped lineitem Q6, N = 600,000,000 rows, row-range
sharded over the ranks by the library (ar_dist_shard_range: ceil(N / G) rows
per rank rounded to 128-row multiples); every shard is decomposed with the
table's global stored width (allreduce-MAX of the planned w_M).
Columns: l_shipdate decomposed 24 GPU / 8 residual bits,
l_discount, l_quantity bit-packed with k = 0, l_extendedprice bit-packed for
the gather; predicates shipdate in [731,1095], discount in [5,7], quantity <=
23; SUM(l_extendedprice * l_discount).  `--scaling weak` instead gives every
rank its own SF100 (600 M-row) range of an SF(100 G) table.

One step = one pass of the whole hot path over the batch.  Headline
(`--variant fused`): ar_select_refine_sum_ws, the one-pass kernel running a2+a3
(approximate select), a5 (refine) and a6 (SUM) -- one launch per query, a
programmatic dependent of the previous query's kernel -- then, with G > 1, the
int64 SUM allreduce (ar_dist_sum) on a side stream that overlaps the next
query.  `staged`: ar_approx_select (ordered candidate relation in HBM) ->
ar_refine_sum, with the candidate-count allgather (ar_dist_offsets) on the side
stream overlapping the refine, then the SUM allreduce.  Both are timed every
run (the other under "variants"), plus:
  * latency: single-query time of isolated launches (no overlap), median / min / p90;
  * c2: BASELINE configs[1] (SF10, 60 M rows per GPU) one-pass throughput;
  * c5: BASELINE configs[4]'s per-GPU share (SF1000 / 8 = 750 M rows) with the
    l_shipdate residual in pinned host memory on the GPU's NUMA node, against
    the host-link roofline measured in the same run;
  * e2e: the decomposed table at rest in pinned host memory, every step copying
    what it scans host->device and reading residual / l_extendedprice sectors
    over the host link, result copied back;
  * cpu_baseline: the CPU oracle (test infrastructure) on a bounded sample;
  * parity: every rank's GPU result against the oracle on its shard, and on
    rank 0 the global SUM / count / offsets against the whole-table oracle.
Inputs are resident in HBM and larger than L2 (C4: 3.45 GB of decomposed
columns per rank at G = 1), so consecutive steps never hit in L2.  K steps are
one CUDA-graph replay bracketed by barrier + synchronize and CUDA events on the
launching stream; the max over ranks is reported.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import platform
import statistics
import subprocess
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
PREDS = [datagen.Q6_SHIPDATE, datagen.Q6_DISCOUNT, datagen.Q6_QUANTITY]
SECTOR = 32
K_SHIP = 8                                   # bwdecompose(l_shipdate, 24): 8 residual bits
WORKLOADS = {
    # name: (seed, scale factor of the table, description)
    "c4": (4, 100.0, "C4: TPC-H SF100-shaped lineitem Q6 (600 M rows), row-sharded"),
    "c2": (2, 10.0, "C2: TPC-H SF10-shaped lineitem Q6 (60 M rows) per GPU"),
    "c5": (5, 1000.0, "C5: per-GPU share (1/8) of TPC-H SF1000-shaped Q6, l_shipdate residual in pinned host memory"),
}


def parse(argv=None):
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=200)
    ap.add_argument("--warmup", type=int, default=10)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--workload", choices=["c4", "c2", "c5"], default="c4",
                    help="headline workload (c5: print only the C5 host-link measurement, for tools)")
    ap.add_argument("--variant", choices=["staged", "fused"], default="fused",
                    help="headline variant (the other one is timed too and reported under 'variants')")
    ap.add_argument("--scaling", choices=["strong", "weak"], default="strong",
                    help="c4: strong = one SF100 table split over the ranks; weak = SF100 per rank")
    ap.add_argument("--only", action="store_true", help="time the headline variant only (no latency/c2/c5)")
    ap.add_argument("--no-c2", action="store_true")
    ap.add_argument("--no-c5", action="store_true")
    ap.add_argument("--split", type=int, default=0,
                    help="c4 / c2: the l_shipdate residual in the split layout with this many high planes apart")
    ap.add_argument("--c5-split", type=int, default=4,
                    help="c5: store the l_shipdate residual in the split layout with this many high planes apart")
    ap.add_argument("--latency-reps", type=int, default=30)
    ap.add_argument("--replays", type=int, default=5, help="extra timed replays for the median / min / p90")
    ap.add_argument("--e2e-steps", type=int, default=5)
    ap.add_argument("--cpu-seconds", type=float, default=10.0)
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--no-parity", action="store_true")
    return ap.parse_args(argv)


def dist_env():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


# ------------------------------------------------------------------ workloads

def shard_of(workload, world, rank, scaling="strong"):
    """(seed, table_sf, table_rows, row0, rows) of this rank's shard.  c4 strong: the library's
    ar_dist_shard_range over the SF100 table; c4 weak / c2: one SF-sized range per rank; c5: the
    per-GPU 1/8 share of the SF1000 table (rank r takes share r; the 8-GPU run covers the table)."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    seed, sf, _ = WORKLOADS[workload]
    per = int(round(sf * datagen.ROWS_PER_SF))
    if workload == "c4" and scaling == "strong":
        row0, rows = _ar.ar_dist_shard_range(per, world, rank)
        return seed, sf, per, row0, rows
    if workload == "c5":
        row0, rows = _ar.ar_dist_shard_range(per, 8, rank % 8)
        return seed, sf, per, row0, rows
    return seed, sf * world, per * world, rank * per, per


def gen_columns(seed, table_sf, row0, rows):
    return datagen.q6_columns(seed, table_sf, n=rows, row0=row0)


def config_dict(workload, world, rows, table_rows, scaling, extra=None):
    d = {"workload": WORKLOADS[workload][2] + (f" over {world} GPU(s)" if workload == "c4" else ""),
         "table_rows": table_rows, "rows_per_gpu": rows, "rows_total": rows * world if workload != "c4" or
         scaling == "weak" else table_rows,
         "decomposition": "l_shipdate 24 GPU/8 residual bits; l_discount, l_quantity, l_extendedprice k=0",
         "predicates": "shipdate in [731,1095], discount in [5,7], quantity in [0,23]; SUM(extendedprice*discount)",
         "parallelism": f"rowshard{world}"}
    if extra:
        d.update(extra)
    return d


# ----------------------------------------------------------------- CPU oracle leg

def cpu_info():
    info = {"model": platform.processor() or None, "sockets": None, "logical_cpus": os.cpu_count()}
    try:
        out = subprocess.run(["lscpu"], capture_output=True, text=True, timeout=10).stdout
        for line in out.splitlines():
            k, _, v = line.partition(":")
            v = v.strip()
            if k.strip() == "Model name":
                info["model"] = v
            elif k.strip() == "Socket(s)":
                info["sockets"] = int(v) if v.isdigit() else v
            elif k.strip() == "Core(s) per socket":
                info["cores_per_socket"] = int(v) if v.isdigit() else v
            elif k.strip() == "Thread(s) per core":
                info["threads_per_core"] = int(v) if v.isdigit() else v
    except Exception:
        pass
    return info


def run_oracle(cols, seconds, threads=0):
    """The oracle as it stands (exact select + SUM with positions) over `cols`, repeated for ~seconds."""
    import oracle
    rows = cols["shipdate"].size
    values = [cols["shipdate"], cols["discount"], cols["quantity"]]
    los = [p[0] for p in PREDS]
    his = [p[1] for p in PREDS]
    aggs = [cols["extprice"], cols["discount"]]
    times = []
    t_end = time.perf_counter() + seconds
    while True:
        t0 = time.perf_counter()
        _, cnt, s = oracle.select_sum(values, los, his, aggs, threads=threads, positions=True)
        times.append(time.perf_counter() - t0)
        if time.perf_counter() >= t_end or len(times) >= 200:
            break
    med = statistics.median(times)
    used = threads if threads > 0 else oracle.default_threads()
    return {"value": rows / med, "unit": UNIT, "cores": used, "kind": "oracle",
            "sample": f"{rows} rows of the workload, exact select + SUM with positions, median of {len(times)} "
                      f"runs ({sum(times):.1f} s)", "count": cnt, "sum": s}


def oracle_counts(cols):
    """Oracle per-shard (|candidates|, |definite|, |R|, SUM) -- the parity reference."""
    import oracle
    values = [cols["shipdate"], cols["discount"], cols["quantity"]]
    los, his = [p[0] for p in PREDS], [p[1] for p in PREDS]
    _, cnt, s = oracle.select_sum(values, los, his, [cols["extprice"], cols["discount"]], threads=0,
                                  positions=False)
    cpos, cdef = oracle.approx_select(values, [K_SHIP, 0, 0], los, his)
    return {"cand": int(cpos.size), "def": int(cdef.sum()), "count": int(cnt), "sum": int(s)}


def oracle_sum_count(cols):
    import oracle
    values = [cols["shipdate"], cols["discount"], cols["quantity"]]
    _, cnt, s = oracle.select_sum(values, [p[0] for p in PREDS], [p[1] for p in PREDS],
                                  [cols["extprice"], cols["discount"]], threads=0, positions=False)
    return int(s), int(cnt)


def reference_arm(args):
    """--impl reference: the CPU oracle, as it stands, on the headline workload's rows (bounded)."""
    world, rank, _ = dist_env()
    if rank != 0:
        return
    seed, table_sf, table_rows, row0, rows = shard_of(args.workload, 1, 0, args.scaling)
    # each step: one oracle pass over a bounded 60 M-row sample of the workload (~0.1 s at 16 cores)
    sample = min(rows, 60_000_000)
    cols = gen_columns(seed, table_sf, row0, sample)
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
    val = sample * steps / dt
    cpu = cpu_info()
    line = {"impl": "reference", "metric": METRIC, "value": val, "unit": UNIT, "n_gpus": args.gpus,
            "steps": steps, "warmup": warm, "ms_per_step": dt / steps * 1e3, "higher_is_better": True,
            "scaling": args.scaling if args.workload == "c4" else "weak", "vs_baseline": None, "dtype": "u32",
            "data": "synthetic",
            "config": config_dict(args.workload, 1, rows, table_rows, args.scaling),
            "cpu_baseline": {"value": val, "unit": UNIT, "cores": oracle.default_threads(), "kind": "oracle",
                             "sample": f"{steps} oracle passes over the first {sample} rows of the workload",
                             "cpu": cpu},
            "e2e": {"value": val, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ------------------------------------------------------------------ clocks (NVML)

class ClockSampler:
    """Samples SM clock and throttle reasons through NVML (the library nvidia-smi reads) every ~2 ms."""

    def __init__(self, index):
        self.samples, self.reasons, self.stop_flag = [], set(), False
        self.mem, self.power = [], []
        self.index = index
        self.ok = False
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            nv = pynvml
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
                self.mem.append(nv.nvmlDeviceGetClockInfo(self.h, nv.NVML_CLOCK_MEM))
                self.power.append(nv.nvmlDeviceGetPowerUsage(self.h) / 1000.0)
                r = nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
                for bit, name in names.items():
                    if bit and (r & bit) == bit and name not in ("None", "GpuIdle"):
                        self.reasons.add(_snake(name))
            except Exception:
                pass
            time.sleep(0.002)

    def __enter__(self):
        if self.ok:
            self.stop_flag = False
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
                "mem_mhz": statistics.median(self.mem) if self.mem else None,
                "power_w_median": statistics.median(self.power) if self.power else None,
                "reasons": sorted(self.reasons), "samples": len(self.samples), "source": "nvml"}


def _snake(s):
    out = ""
    for ch in s:
        out += ("_" + ch.lower()) if ch.isupper() and out else ch.lower()
    return out


# -------------------------------------------------------------- algorithmic bytes

def split_lo_byte(blk, h):
    """Byte offset of the low residual planes of 32-row block `blk` in the split layout (ar.h
    ar_column_desc.residual_split: super-groups of 256 blocks, h high planes then k - h low planes)."""
    return 4 * ((blk // 256) * (256 * K_SHIP) + 256 * h + (blk % 256) * (K_SHIP - h))


def split_hi_byte(blk, h):
    return 4 * ((blk // 256) * (256 * K_SHIP) + (blk % 256) * h)


def _sectors(start, nbytes, gran=SECTOR):
    """Distinct `gran`-byte units touched by the byte ranges [start, start + nbytes)."""
    if start.size == 0:
        return 0
    return np.unique(np.concatenate([start // gran, (start + nbytes - 1) // gran])).size


def algorithmic_bytes(cols, w_sd=None, split=0, high_streamed=True):
    """Bytes the method must move per query: packed scans + sector-granular gathers + output.
    Per column: scanned majors N w / 8; the l_shipdate residual: 32 B per distinct residual sector that holds
    a non-definite candidate; l_extendedprice: 32 B per distinct sector that holds (part of) a result row;
    each gathered column capped at its size; + 8 B of output.  Computed from the data, not the GPU.
    split = h > 0 (the split residual layout, DESIGN s6.3d): with high_streamed (HBM residual, one-pass
    kernel) the h high planes are a scanned part (N h / 8) and the k - h low planes are gathered for the rows
    the high planes leave undecided (candidate, not definite at granularity 2^(k-h)); otherwise (residual
    over the host link) the high planes of every block with a non-definite candidate are gathered too."""
    sd, dc, qt, ep = cols["shipdate"], cols["discount"], cols["quantity"], cols["extprice"]
    rows = sd.size
    if w_sd is None:
        w_sd = int((int(sd.max()) >> K_SHIP)).bit_length()
    w_dc, w_qt, w_ep = int(dc.max()).bit_length(), int(qt.max()).bit_length(), int(ep.max()).bit_length()
    scan = rows * (w_sd + w_dc + w_qt) / 8.0
    lo, hi = PREDS[0]

    def cand_def(kk):   # candidate / definite buckets of l_shipdate at granularity 2^kk
        m = sd >> kk
        c = (m >= (lo >> kk)) & (m <= (hi >> kk))
        d = (m >= ((lo + (1 << kk) - 1) >> kk)) & (m <= (((hi + 1) >> kk) - 1))
        return c, d

    cand_sd, def_sd = cand_def(K_SHIP)
    other = (dc >= PREDS[1][0]) & (dc <= PREDS[1][1]) & (qt >= PREDS[2][0]) & (qt <= PREDS[2][1])
    cand = cand_sd & other
    nondef = cand & ~def_sd
    result = other & (sd >= lo) & (sd <= hi)
    idx_nd = np.nonzero(nondef)[0].astype(np.int64)
    idx_res = np.nonzero(result)[0].astype(np.int64)
    blk_nd = np.unique(idx_nd // 32)
    if split:
        kl = K_SHIP - split
        cf, df = cand_def(kl)
        blk_und = np.unique(np.nonzero(cf & ~df & other)[0].astype(np.int64) // 32)
        lo_start = split_lo_byte(blk_und, split)
        res_sectors = _sectors(lo_start, 4 * kl)
        res64 = _sectors(lo_start, 4 * kl, 64)
        if high_streamed:
            scan += rows * split / 8.0
        else:
            hi_start = split_hi_byte(blk_nd, split)
            res_sectors += _sectors(hi_start, 4 * split)
            res64 += _sectors(hi_start, 4 * split, 64)
    else:
        # SLICED residual: a 32-row block's k planes are k * 4 B (one 32-B sector at k = 8)
        res_sectors = np.unique(blk_nd * (K_SHIP * 4) // SECTOR).size
        res64 = np.unique(blk_nd * (K_SHIP * 4) // 64).size
    b0 = idx_res * w_ep                                   # a packed 24-bit value may straddle two sectors
    ep_sectors = np.unique(np.concatenate([b0 // (SECTOR * 8), (b0 + w_ep - 1) // (SECTOR * 8)])).size
    gathered = min(rows * K_SHIP / 8.0, SECTOR * res_sectors) + min(rows * w_ep / 8.0, SECTOR * ep_sectors)
    ncand = int(cand.sum())
    ep64 = np.unique(np.concatenate([b0 // (64 * 8), (b0 + w_ep - 1) // (64 * 8)])).size
    return {"scan": scan, "gather": gathered, "residual_gather": SECTOR * res_sectors,
            "ep_gather": SECTOR * ep_sectors, "zero_copy_64": 64.0 * (res64 + ep64),
            "residual_granules_64": 64.0 * res64, "residual_sectors": int(res_sectors), "ep_sectors": int(ep_sectors),
            "total": scan + gathered + 8.0, "n_cand": ncand, "n_def": int((cand & def_sd).sum()),
            "n_result": int(result.sum()), "cand_list_bytes": 8.0 * ncand, "residual_split": split,
            "widths": {"shipdate_major": w_sd, "discount": w_dc, "quantity": w_qt, "extprice": w_ep}}


def load_peaks():
    peaks = {}
    try:
        peaks = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))
    except Exception:
        pass
    hbm = peaks.get("hbm_gbs")
    src = "measured (MEASURED_PEAKS.json hbm_gbs, copy kernel)" if hbm else "fallback (B200_PROFILING.md 6.65 TB/s)"
    return (hbm or 6650.0), src


def load_traffic():
    """dram__bytes_read.sum + dram__bytes_write.sum per launch from the committed `ncu --set full` capture
    (tools/ncu_traffic.py writes profiles/traffic.json with the commit and config it was taken at)."""
    try:
        return json.load(open(os.path.join(ROOT, "profiles", "traffic.json")))
    except Exception:
        return {}


def pct(xs, q):
    xs = sorted(xs)
    if not xs:
        return None
    i = min(len(xs) - 1, max(0, int(math.ceil(q / 100.0 * len(xs))) - 1))
    return xs[i]


def dist_stats(xs):
    return {"median": statistics.median(xs), "min": min(xs), "p90": pct(xs, 90), "n": len(xs)} if xs else None


# ----------------------------------------------------------------------- our arm

class Ctx:
    """Per-rank runtime: device, streams, process group, the library's NCCL communicator, CUDA events."""

    def __init__(self, args):
        import torch
        from cuda.bindings import driver as drv
        from paper_conf_icde_pirkmk14_b200 import _ar
        self.torch, self.drv, self._ar = torch, drv, _ar
        self.world, self.rank, self.local = dist_env()
        if self.world != args.gpus and self.world > 1:
            raise SystemExit(f"--gpus {args.gpus} but WORLD_SIZE {self.world}")
        torch.cuda.set_device(self.local)
        self.dev = torch.device("cuda", self.local)
        self.pg = None
        self.dist_h = None
        if self.world > 1:
            import torch.distributed as tdist
            tdist.init_process_group("nccl", device_id=self.dev)
            self.pg = tdist
            uid = _ar.ar_dist_get_unique_id() if self.rank == 0 else b""
            obj = [uid]
            tdist.broadcast_object_list(obj, src=0)
            self.dist_h = _ar.ar_dist_init(obj[0], self.rank, self.world)
        self.stream = torch.cuda.Stream(device=self.dev)
        self.side = torch.cuda.Stream(device=self.dev)          # collectives overlapping the next query
        self.s_ptr = self.stream.cuda_stream
        self.side_ptr = self.side.cuda_stream

    def event(self, flags=None):
        drv = self.drv
        err, e = drv.cuEventCreate(drv.CUevent_flags.CU_EVENT_DEFAULT if flags is None else flags)
        assert err == drv.CUresult.CUDA_SUCCESS, err
        return e

    def rec(self, e, stream_ptr=None, external=False):
        drv = self.drv
        s = self.s_ptr if stream_ptr is None else stream_ptr
        if external:
            err, = drv.cuEventRecordWithFlags(e, s, drv.CUevent_record_flags.CU_EVENT_RECORD_EXTERNAL)
        else:
            err, = drv.cuEventRecord(e, s)
        assert err == drv.CUresult.CUDA_SUCCESS, err

    def wait(self, stream_ptr, e):
        err, = self.drv.cuStreamWaitEvent(stream_ptr, e, 0)
        assert err == self.drv.CUresult.CUDA_SUCCESS, err

    def elapsed(self, a, b):
        err, ms = self.drv.cuEventElapsedTime(a, b)
        assert err == self.drv.CUresult.CUDA_SUCCESS, err
        return ms

    def barrier(self):
        if self.pg:
            self.pg.barrier()
        self.torch.cuda.synchronize()

    def max_over_ranks(self, x):
        if not self.pg:
            return x
        t = self.torch.tensor([x], dtype=self.torch.float64, device=self.dev)
        self.pg.all_reduce(t, op=self.pg.ReduceOp.MAX)
        return float(t.item())

    def allreduce_max_int(self, x):
        if not self.pg:
            return x
        t = self.torch.tensor([x], dtype=self.torch.int64, device=self.dev)
        self.pg.all_reduce(t, op=self.pg.ReduceOp.MAX)
        return int(t.item())

    def gather_obj(self, obj):
        if not self.pg:
            return [obj]
        out = [None] * self.world
        self.pg.all_gather_object(out, obj)
        return out


class Q6:
    """One rank's decomposed Q6 columns and the query's predicate / aggregate handles."""

    def __init__(self, ctx, cols, residual_loc=0, split=0):
        from paper_conf_icde_pirkmk14_b200 import _ar, column as cu
        agree = ctx.allreduce_max_int          # the table's global w_M per column (allreduce-MAX)
        self.sd = cu.BWDColumn(cols["shipdate"], 32 - K_SHIP, residual_loc=residual_loc, device=ctx.dev,
                               width_agree=agree, split=split)
        self.dc = cu.BWDColumn(cols["discount"], 32, device=ctx.dev, width_agree=agree)
        self.qt = cu.BWDColumn(cols["quantity"], 32, device=ctx.dev, width_agree=agree)
        self.ep = cu.BWDColumn(cols["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED, device=ctx.dev, width_agree=agree)
        self.rows = self.sd.n
        self.preds = [(self.sd.handle, *PREDS[0]), (self.dc.handle, *PREDS[1]), (self.qt.handle, *PREDS[2])]
        self.aggs = [self.ep.handle, self.dc.handle]
        self.cols = [self.sd, self.dc, self.qt, self.ep]

    def device_bytes(self):
        return sum(c.nbytes()["major"] + (c.nbytes()["residual"] if c.desc.residual_loc == 0 else 0)
                   for c in self.cols)

    def free(self):
        for c in self.cols:
            c.free()
        self.cols = []


class Runner:
    """Times the fused and staged query streams on one rank."""

    def __init__(self, ctx, q, K):
        import torch
        from paper_conf_icde_pirkmk14_b200 import _ar, column as cu
        self.ctx, self.q, self.K, self._ar = ctx, q, K, _ar
        dev = ctx.dev
        self.cands = cu.CandidateList(q.rows, device=dev)
        self.ws_sel = cu.Workspace(_ar.ar_select_ws_bytes(q.rows), device=dev)
        self.srs_ws = cu.SrsWorkspace(device=dev)
        self.srs_flags = _ar.AR_SRS_PDL_EARLY_READ
        # one output slot per step: the side stream's allreduce of query i never races query i + 1
        self.out = torch.zeros((K + 64, 4), dtype=torch.int64, device=dev)
        self.counts = torch.zeros((K + 64, max(ctx.world, 1)), dtype=torch.int64, device=dev)
        self.goff = torch.zeros((K + 64,), dtype=torch.int64, device=dev)
        self.kern_names = {}

    def slot(self, i):
        return self.out[i % self.out.shape[0]]

    def step(self, variant, i, ev=None, fork=None, pdl=True):
        """One query on the main stream; with G > 1 its collectives go to the side stream, which waits on
        `fork[i]` (recorded after the query's last kernel) -- nothing on the main stream waits for them."""
        ctx, q, _ar = self.ctx, self.q, self._ar
        o = self.slot(i)
        if variant == "fused":
            if ev is not None:
                ctx.rec(ev[0], external=True)
            _ar.ar_select_refine_sum_ws(q.preds, q.aggs, self.srs_flags if pdl else 0, o.data_ptr(),
                                        self.srs_ws.ptr, self.srs_ws.nbytes, ctx.s_ptr)
            if ev is not None:
                ctx.rec(ev[1], external=True)
            if ctx.dist_h:
                ctx.rec(fork[i])
                ctx.wait(ctx.side_ptr, fork[i])
                _ar.ar_dist_sum(ctx.dist_h, o.data_ptr(), 4, ctx.side_ptr)
        else:
            if ev is not None:
                ctx.rec(ev[0], external=True)
            _ar.ar_approx_select(q.preds, _ar.AR_SELECT_CARRY_APPR, self.cands.c, self.ws_sel.ptr,
                                 self.ws_sel.nbytes, ctx.s_ptr)
            self.select_kernel = _ar.ar_last_scan_kernel()
            if ev is not None:
                ctx.rec(ev[1], external=True)
            if ctx.dist_h:       # candidate-count allgather + prefix (a4), overlapping the refine
                j = i % self.counts.shape[0]
                o2 = o[2:3]
                o2.copy_(self.cands.count_t)                      # |candidates| of this query into its slot
                ctx.rec(fork[i][0])
                ctx.wait(ctx.side_ptr, fork[i][0])
                _ar.ar_dist_offsets(ctx.dist_h, o2.data_ptr(), self.counts[j].data_ptr(),
                                    self.goff[j:j + 1].data_ptr(), ctx.side_ptr)
            if ev is not None:
                ctx.rec(ev[2], external=True)
            _ar.ar_refine_sum(self.cands.c, q.preds, q.aggs, o.data_ptr(), o.data_ptr() + 8, ctx.s_ptr)
            if ev is not None:
                ctx.rec(ev[3], external=True)
            if ctx.dist_h:
                ctx.rec(fork[i][1])
                ctx.wait(ctx.side_ptr, fork[i][1])
                _ar.ar_dist_sum(ctx.dist_h, o.data_ptr(), 2, ctx.side_ptr)

    def join(self, ev):
        """Main stream waits for the side stream (the last collectives) -- the end of the timed region."""
        if self.ctx.dist_h:
            self.ctx.rec(ev, self.ctx.side_ptr)
            self.ctx.wait(self.ctx.s_ptr, ev)

    def forks(self, variant, n):
        ctx = self.ctx
        if not ctx.dist_h:
            return None
        if variant == "fused":
            return [ctx.event() for _ in range(n)]
        return [(ctx.event(), ctx.event()) for _ in range(n)]

    def kernel_names(self, variant):
        torch = self.ctx.torch
        with torch.cuda.stream(self.ctx.stream):
            self.step(variant, 0, fork=self.forks(variant, 1))
            jn = self.ctx.event()
            self.join(jn)
        self.ctx.stream.synchronize()
        self.ctx.side.synchronize()
        return self._ar.ar_last_scan_kernel() or ""

    def time_variant(self, variant, W, replays, sampler=None):
        ctx, torch, K = self.ctx, self.ctx.torch, self.K
        with torch.cuda.stream(ctx.stream):                 # eager warm-up (primes the library's caches)
            fk = self.forks(variant, max(3, W))
            for i in range(max(3, W)):
                self.step(variant, i, fork=fk)
            jn = ctx.event()
            self.join(jn)
        torch.cuda.synchronize()
        n_ev = 4 if variant == "staged" else 2
        evs = [[ctx.event() for _ in range(n_ev)] for _ in range(K)]
        f_w, f_t, f_e = self.forks(variant, W), self.forks(variant, K), self.forks(variant, K)
        j_w, j_t, j_e = ctx.event(), ctx.event(), ctx.event()
        # the headline graph has no event nodes between steps (they would serialise the programmatic
        # dependent launches); a second graph with external events gives per-kernel durations
        g_warm, g_timed, g_ev = torch.cuda.CUDAGraph(), torch.cuda.CUDAGraph(), torch.cuda.CUDAGraph()
        with torch.cuda.graph(g_warm, stream=ctx.stream, capture_error_mode="relaxed"):
            for i in range(W):
                self.step(variant, i, fork=f_w)
            self.join(j_w)
        with torch.cuda.graph(g_timed, stream=ctx.stream, capture_error_mode="relaxed"):
            for i in range(K):
                self.step(variant, i, fork=f_t)
            self.join(j_t)
        with torch.cuda.graph(g_ev, stream=ctx.stream, capture_error_mode="relaxed"):
            for i in range(K):
                self.step(variant, i, evs[i], fork=f_e)
            self.join(j_e)
        torch.cuda.synchronize()
        t0, t1 = ctx.event(), ctx.event()
        runs = []
        for r in range(1 + replays):
            with torch.cuda.stream(ctx.stream):
                g_warm.replay()
                ctx.stream.synchronize()
                ctx.barrier()
                # run 0 is the headline (its clocks are the line's); the replays get their own sampler
                if sampler is not None and r == 0:
                    cm = sampler
                elif sampler is not None:
                    if getattr(sampler, "replay_sampler", None) is None:
                        sampler.replay_sampler = ClockSampler(sampler.index)
                    cm = sampler.replay_sampler
                else:
                    cm = _Null()
                with cm:
                    ctx.rec(t0)
                    g_timed.replay()
                    ctx.rec(t1)
                    ctx.stream.synchronize()
            torch.cuda.synchronize()
            runs.append(ctx.max_over_ranks(ctx.elapsed(t0, t1)))
        with torch.cuda.stream(ctx.stream):
            g_ev.replay()
            ctx.stream.synchronize()
        torch.cuda.synchronize()
        ctx.barrier()
        if variant == "staged":
            kern = {"select": [ctx.elapsed(e[0], e[1]) for e in evs], "refine_sum": [ctx.elapsed(e[2], e[3]) for e in evs]}
        else:
            kern = {"fused": [ctx.elapsed(e[0], e[1]) for e in evs]}
        res = self.slot(K - 1).cpu().tolist()
        allres = self.out[:K].cpu()
        consistent = bool((allres == allres[0]).all().item())
        del g_warm, g_timed, g_ev
        return runs, kern, res, consistent

    def latency(self, variant, reps):
        """Single-query latency: isolated launches (no PDL, stream synchronised between queries), CUDA events
        around each query on the launching stream (and its collectives when G > 1)."""
        ctx, torch = self.ctx, self.ctx.torch
        a, b = ctx.event(), ctx.event()
        out = []
        for i in range(reps + 3):
            ctx.barrier()
            with torch.cuda.stream(ctx.stream):
                ctx.rec(a)
                self.step(variant, i, fork=self.forks(variant, i + 1), pdl=False)
                jn = ctx.event()
                self.join(jn)
                ctx.rec(b)
                ctx.stream.synchronize()
            if i >= 3:
                out.append(ctx.max_over_ranks(ctx.elapsed(a, b)))
        return out


class _Null:
    def __enter__(self):
        return self

    def __exit__(self, *a):
        return False


def numa_node_of(ctx):
    """NUMA node of this rank's GPU (sysfs of its PCI device) and that node's CPUs, or (None, None)."""
    try:
        props = ctx.torch.cuda.get_device_properties(ctx.dev)
        bus = f"{props.pci_domain_id:04x}:{props.pci_bus_id:02x}:{props.pci_device_id:02x}.0"
        node = int(open(f"/sys/bus/pci/devices/{bus}/numa_node").read().strip())
        if node < 0:
            return None, None, bus
        cpus = open(f"/sys/devices/system/node/node{node}/cpulist").read().strip()
        cpuset = set()
        for part in cpus.split(","):
            lo, _, hi = part.partition("-")
            cpuset.update(range(int(lo), int(hi or lo) + 1))
        return node, cpuset, bus
    except Exception:
        return None, None, None


def measure_h2d(ctx, nbytes=1 << 30, reps=5):
    """Pinned host -> device copy bandwidth of this GPU's host link (GB/s, best of reps)."""
    torch = ctx.torch
    h = torch.empty(nbytes, dtype=torch.uint8).pin_memory()
    d = torch.empty(nbytes, dtype=torch.uint8, device=ctx.dev)
    a, b = ctx.event(), ctx.event()
    best = 0.0
    for _ in range(reps):
        with torch.cuda.stream(ctx.stream):
            ctx.rec(a)
            d.copy_(h, non_blocking=True)
            ctx.rec(b)
            ctx.stream.synchronize()
        best = max(best, nbytes / (ctx.elapsed(a, b) / 1e3) / 1e9)
    del h, d
    return best


def bench_c5(ctx, args):
    """BASELINE configs[4] per-GPU share: 750 M rows of the SF1000 table (rank r: share r of 8) with the
    l_shipdate residual in pinned host memory on this GPU's NUMA node; majors and l_extendedprice in HBM.
    The one-pass kernel reads the residual sectors it needs over the host link (zero copy)."""
    torch = ctx.torch
    seed, table_sf, table_rows, row0, rows = shard_of("c5", ctx.world, ctx.rank)
    node, cpus, bus = numa_node_of(ctx)
    old_aff = None
    if cpus:
        try:                                   # first touch of the pinned pages from the GPU's node
            old_aff = os.sched_getaffinity(0)
            os.sched_setaffinity(0, cpus)
        except Exception:
            old_aff = None
    cols = gen_columns(seed, table_sf, row0, rows)
    q = Q6(ctx, cols, residual_loc=1, split=args.c5_split)
    link = measure_h2d(ctx)
    if old_aff:
        os.sched_setaffinity(0, old_aff)
    ab = algorithmic_bytes(cols, q.sd.w_major, args.c5_split, high_streamed=False)
    r = Runner(ctx, q, max(3, min(args.steps, 10)))
    runs, kern, res, consistent = r.time_variant("fused", 2, 0)
    ms = runs[0] / r.K
    host_bytes = ab["residual_gather"]
    parity = None
    if not args.no_parity:
        oc = oracle_counts(cols)
        parity = {"gpu": res, "oracle": [oc["sum"], oc["count"], oc["cand"], oc["def"]],
                  "match": res == [oc["sum"], oc["count"], oc["cand"], oc["def"]] and consistent}
    hbm_bytes = ab["scan"] + ab["ep_gather"] + 8.0
    out = {"workload": WORKLOADS["c5"][2], "rows": rows, "table_rows": table_rows, "row0": row0,
           "value": rows / (ms / 1e3), "unit": UNIT, "ms_per_step": ms, "steps": r.K,
           "host_link": {"bound": "host_link", "achieved": host_bytes / (ms / 1e3) / 1e9, "peak": link,
                         "unit": "GB/s", "frac": host_bytes / (ms / 1e3) / 1e9 / link,
                         "peak_source": "pinned->device cudaMemcpyAsync of 1 GiB on this GPU, best of 5, same run",
                         "algorithmic_host_bytes": host_bytes, "host_bytes_64B_granules": ab["residual_granules_64"]},
           "hbm": {"bytes": hbm_bytes, "gbs": hbm_bytes / (ms / 1e3) / 1e9},
           "numa_node": node, "gpu_pci": bus, "pinned_on_node": bool(cpus), "residual_split": args.c5_split,
           "kernel": r.kernel_names("fused"), "parity": parity}
    del r
    q.free()
    torch.cuda.empty_cache()
    return out


def run_e2e(ctx, q, ab, steps, sd_host=None):
    """The same metric end to end through the C ABI with HOST buffers: the decomposed table at rest in
    pinned host memory; every step copies the scanned majors H2D, ar_select_refine_sum reads the shipdate
    residual and l_extendedprice zero-copy over the host link (only touched sectors), and the (SUM, count)
    result is copied D2H (after the SUM allreduce when G > 1).  Double-buffered: step i + 1's major copies
    (copy stream, device buffer set (i + 1) % 2) run while step i's query reads the host link, and wait for
    step i - 1's query (the previous user of that buffer set)."""
    torch, _ar = ctx.torch, ctx._ar
    from paper_conf_icde_pirkmk14_b200 import column as cu

    def twin(col):   # a second handle: its own device major buffer, the same (host) residual
        desc = _ar.ColumnDesc.from_buffer_copy(col.desc)
        res = col.residual if col.desc.k > 0 else None
        return cu.BWDColumn(None, 0, _wrap=(desc, torch.empty_like(col.major), res), device=ctx.dev)

    # sd_host: the l_shipdate column decomposed with its residual in pinned host memory (split layout)
    sd_e = sd_host if sd_host is not None else q.sd.copy(residual_loc=_ar.AR_LOC_HOST_PINNED)
    dc_e, qt_e = q.dc.copy(), q.qt.copy()
    ep_e = q.ep.copy(major_loc=_ar.AR_LOC_HOST_PINNED)
    sets = [(sd_e, dc_e, qt_e), (twin(sd_e), twin(dc_e), twin(qt_e))]
    srcs = [q.sd.major.cpu().pin_memory(), q.dc.major.cpu().pin_memory(), q.qt.major.cpu().pin_memory()]
    preds = [[(sd.handle, *PREDS[0]), (dc.handle, *PREDS[1]), (qt.handle, *PREDS[2])] for sd, dc, qt in sets]
    aggs = [[ep_e.handle, dc.handle] for _, dc, _ in sets]
    outs = [torch.zeros(4, dtype=torch.int64, device=ctx.dev) for _ in range(2)]
    res_host = [torch.zeros(4, dtype=torch.int64).pin_memory() for _ in range(2)]
    copied = sum(h.numel() for h in srcs)
    cs = torch.cuda.Stream(device=ctx.dev)

    def run(n, e0=None):
        ev_c = [torch.cuda.Event() for _ in range(n)]
        ev_d = [torch.cuda.Event() for _ in range(n)]
        start = torch.cuda.Event()
        start.record(ctx.stream)
        for i in range(n):
            b = i % 2
            with torch.cuda.stream(cs):
                cs.wait_event(start)
                if i >= 2:
                    cs.wait_event(ev_d[i - 2])      # step i - 2's query is done with buffer set b
                for h, col in zip(srcs, sets[b]):
                    col.major.copy_(h, non_blocking=True)
                ev_c[i].record(cs)
            ctx.stream.wait_event(ev_c[i])
            with torch.cuda.stream(ctx.stream):
                _ar.ar_select_refine_sum(preds[b], aggs[b], outs[b].data_ptr(), ctx.s_ptr)
                if ctx.dist_h:
                    _ar.ar_dist_sum(ctx.dist_h, outs[b].data_ptr(), 4, ctx.s_ptr)
                res_host[b].copy_(outs[b], non_blocking=True)
                ev_d[i].record(ctx.stream)

    run(2)
    torch.cuda.synchronize()
    ctx.barrier()
    e0, e1 = ctx.event(), ctx.event()
    ctx.rec(e0)
    run(steps)
    ctx.rec(e1)
    ctx.stream.synchronize()
    ms = ctx.max_over_ranks(ctx.elapsed(e0, e1))
    result = res_host[(steps - 1) % 2].tolist()
    for c in (sd_e, dc_e, qt_e, ep_e, *sets[1]):
        c.free()
    return {"ms_total": ms, "steps": steps, "h2d_copied": copied, "zero_copy_64": ab["zero_copy_64"], "result": result}


def ours(args):
    ctx = Ctx(args)
    torch, _ar = ctx.torch, ctx._ar
    if args.workload == "c5":
        out = bench_c5(ctx, args)
        if ctx.rank == 0:
            print(json.dumps(out), flush=True)
        return
    world, rank = ctx.world, ctx.rank
    seed, table_sf, table_rows, row0, rows = shard_of(args.workload, world, rank, args.scaling)
    cols = gen_columns(seed, table_sf, row0, rows)
    q = Q6(ctx, cols, split=args.split)
    torch.cuda.synchronize()
    K = args.steps
    hbm_peak, peak_src = load_peaks()
    ab = algorithmic_bytes(cols, q.sd.w_major, args.split)
    r = Runner(ctx, q, K)
    names = {"fused": r.kernel_names("fused"), "staged": None}
    names["staged"] = r.kernel_names("staged")
    sel_kernels = (["select_rr_kernel"] if getattr(r, "select_kernel", "") == "select_rr_kernel"
                   else ["select_tile_kernel", "compact_kernel"])
    KERNELS = {"staged": sel_kernels + [names["staged"] or "refine_sum_kernel"],
               "fused": [names["fused"] or "fused_kernel"]}
    per_kernel_bytes = {"fused": ab["total"], "select": ab["scan"] + ab["cand_list_bytes"],
                        "refine_sum": ab["cand_list_bytes"] + ab["gather"] + 16.0}
    kname = {"fused": KERNELS["fused"][0], "select": "+".join(sel_kernels), "refine_sum": KERNELS["staged"][-1]}

    variants = [args.variant] + [v for v in ("fused", "staged") if v != args.variant and not args.only]
    sampler = ClockSampler(torch.cuda.current_device() if "CUDA_VISIBLE_DEVICES" not in os.environ else ctx.local)
    results = {}
    traffic = load_traffic()
    for v in variants:
        runs, kern, res, consistent = r.time_variant(v, args.warmup, args.replays if v == args.variant else 0,
                                                     sampler if v == args.variant else None)
        ms_total = runs[0]
        ms_step = ms_total / K
        kern_ms = {k: statistics.mean(x) for k, x in kern.items()}
        if v == "fused" and world == 1:
            # one launch per step: the steady-state launch duration is the step time; the evented graph's
            # (serialised, isolated) launch time is kept alongside
            kern_ms = {"fused": ms_step, "fused (isolated launch)": kern_ms["fused"]}
        dom = max((k for k in kern_ms if k in per_kernel_bytes), key=lambda k: kern_ms[k])
        achieved = per_kernel_bytes[dom] / (kern_ms[dom] / 1e3) / 1e9
        tr = traffic.get(args.workload, {}).get(kname[dom])
        results[v] = {
            "value": rows * world * K / (ms_total / 1e3) if args.workload != "c4" or args.scaling == "weak"
            else table_rows * K / (ms_total / 1e3),
            "ms_per_step": ms_step, "result": res, "steps_consistent": consistent,
            "ms_per_step_replays": dict(dist_stats([x / K for x in runs]) or {},
                                        runs=[round(x / K, 5) for x in runs]),
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": hbm_peak, "unit": "GB/s",
                         "frac": achieved / hbm_peak, "traffic": (tr or {}).get("bytes_per_launch"),
                         "traffic_source": (tr or {}).get("source"),
                         "kernel": kname[dom], "algorithmic_bytes_per_launch": per_kernel_bytes[dom],
                         "kernel_ms": kern_ms[dom], "peak_source": peak_src,
                         "per_kernel": {kname.get(k.split(" (")[0], k) + (" (isolated launch)" if "(" in k else ""):
                                        {"ms": kern_ms[k], "bytes": per_kernel_bytes[k.split(" (")[0]],
                                         "gbs": per_kernel_bytes[k.split(" (")[0]] / (kern_ms[k] / 1e3) / 1e9}
                                        for k in kern_ms},
                         "step_bytes": ab["total"],
                         "step_frac": ab["total"] / (ms_step / 1e3) / 1e9 / hbm_peak},
            "gpu_launches": len(KERNELS[v]) * K, "gpu_kernels": KERNELS[v]}
    head = results[args.variant]

    latency = None
    if not args.only and args.latency_reps > 0:
        latency = {}
        for v in variants:
            lat = r.latency(v, args.latency_reps)
            st = dist_stats(lat)
            latency[v] = {"ms": st, "rows_per_s_median": (table_rows if args.workload == "c4" and
                                                          args.scaling == "strong" else rows * world)
                          / (st["median"] / 1e3),
                          "frac_median": ab["total"] / (st["median"] / 1e3) / 1e9 / hbm_peak}

    # parity (untimed): this rank's shard against the oracle; rank 0: global SUM / count / offsets against
    # the whole-table oracle
    parity = None
    if not args.no_parity:
        oc = oracle_counts(cols)
        local_ok = {}
        with torch.cuda.stream(ctx.stream):
            o = torch.zeros(4, dtype=torch.int64, device=ctx.dev)
            _ar.ar_select_refine_sum(q.preds, q.aggs, o.data_ptr(), ctx.s_ptr)
            _ar.ar_approx_select(q.preds, _ar.AR_SELECT_CARRY_APPR, r.cands.c, r.ws_sel.ptr, r.ws_sel.nbytes,
                                 ctx.s_ptr)
            o2 = torch.zeros(2, dtype=torch.int64, device=ctx.dev)
            _ar.ar_refine_sum(r.cands.c, q.preds, q.aggs, o2.data_ptr(), o2.data_ptr() + 8, ctx.s_ptr)
            ctx.stream.synchronize()
        local = o.cpu().tolist()
        local_ok["fused"] = local == [oc["sum"], oc["count"], oc["cand"], oc["def"]]
        local_ok["staged"] = o2.cpu().tolist() == [oc["sum"], oc["count"]] and r.cands.count() == oc["cand"]
        staged_ran = "staged" in results
        gathered = ctx.gather_obj({"rank": rank, "row0": row0, "rows": rows, "oracle": oc, "local_ok": local_ok,
                                   "goff": int(r.goff[(K - 1) % r.goff.shape[0]].item())
                                   if (ctx.dist_h and staged_ran) else None})
        if rank == 0:
            gathered.sort(key=lambda d: d["rank"])
            if world == 1 or args.workload != "c4" or args.scaling != "strong":
                whole = {"sum": sum(g["oracle"]["sum"] for g in gathered),
                         "count": sum(g["oracle"]["count"] for g in gathered), "source": "sum of shard oracles"}
            else:
                # regenerate the whole SF100 table in chunks and run the oracle over it on rank 0
                ws_sum = ws_cnt = 0
                step_rows = 50_000_000
                for c0 in range(0, table_rows, step_rows):
                    cc = gen_columns(seed, table_sf, c0, min(step_rows, table_rows - c0))
                    a_sum, a_cnt = oracle_sum_count(cc)
                    ws_sum += a_sum
                    ws_cnt += a_cnt
                whole = {"sum": ws_sum, "count": ws_cnt, "source": "oracle over the whole table (rank 0)"}
            cand_prefix = np.concatenate([[0], np.cumsum([g["oracle"]["cand"] for g in gathered])[:-1]]).tolist()
            glob = {v: results[v]["result"] for v in results}
            parity = {"whole_table_oracle": whole,
                      "gpu_global": {v: glob[v][:2] for v in glob},
                      "global_match": all(glob[v][0] == whole["sum"] and glob[v][1] == whole["count"]
                                          for v in glob),
                      "all_steps_identical": all(results[v]["steps_consistent"] for v in results),
                      "per_rank_match": [g["local_ok"] for g in gathered],
                      "candidate_offsets_gpu": [g["goff"] for g in gathered] if ctx.dist_h and staged_ran else None,
                      "candidate_offsets_oracle": cand_prefix,
                      "offsets_match": ([g["goff"] for g in gathered] == cand_prefix)
                      if ctx.dist_h and staged_ran else None}
            parity["match"] = bool(parity["global_match"] and parity["all_steps_identical"] and
                                   all(all(x.values()) for x in parity["per_rank_match"]) and
                                   parity["offsets_match"] in (None, True))

    e2e = None
    if args.e2e_steps > 0:
        # the e2e path reads the residual over the host link: there the split layout (--c5-split high
        # planes apart, as C5) is the faster one (DESIGN s6.3d)
        from paper_conf_icde_pirkmk14_b200 import column as cu
        hsplit = args.c5_split
        sd_host = cu.BWDColumn(cols["shipdate"], 32 - K_SHIP, residual_loc=_ar.AR_LOC_HOST_PINNED, device=ctx.dev,
                               width_agree=ctx.allreduce_max_int, split=hsplit)
        ab_e = algorithmic_bytes(cols, sd_host.w_major, hsplit, high_streamed=False)
        e = run_e2e(ctx, q, ab_e, args.e2e_steps, sd_host=sd_host)
        e2e = {"value": (table_rows if args.workload == "c4" and args.scaling == "strong" else rows * world)
               * e["steps"] / (e["ms_total"] / 1e3), "unit": UNIT,
               "h2d_bytes_per_step": int(e["h2d_copied"] + e["zero_copy_64"]), "d2h_bytes_per_step": 32,
               "h2d_copied_bytes": int(e["h2d_copied"]), "h2d_zero_copy_bytes_64B": int(e["zero_copy_64"]),
               "ms_per_step": e["ms_total"] / e["steps"], "result_matches_device_run": e["result"][:2] == head["result"][:2],
               "path": "decomposed table in pinned host memory; per step: cudaMemcpyAsync H2D of the scanned majors "
                       "(copy stream, double-buffered: overlaps the previous step's query), "
                       "ar_select_refine_sum reading the shipdate residual (split layout, "
                       f"{hsplit} high planes apart) and l_extendedprice zero-copy over the host "
                       "link (only touched 64-B granules), [SUM allreduce,] D2H of (SUM, count, |cand|, |def|)"}

    del r
    q.free()
    del cols
    torch.cuda.empty_cache()

    c2 = None
    if not args.only and not args.no_c2 and args.workload != "c2":
        seed2, sf2, trows2, r02, rows2 = shard_of("c2", world, rank)
        cols2 = gen_columns(seed2, sf2, r02, rows2)
        q2 = Q6(ctx, cols2, split=args.split)
        ab2 = algorithmic_bytes(cols2, q2.sd.w_major, args.split)
        # C2 (345 MB per copy) is rotated over 3 copies of the decomposed columns so no step hits in L2
        copies = [q2] + [_copy_q6(ctx, q2) for _ in range(2)]
        r2 = RotRunner(ctx, copies, max(args.steps, 200))
        runs, kern, res, consistent = r2.time_variant("fused", args.warmup, 0)
        ms = runs[0] / r2.K
        oc2 = oracle_counts(cols2) if not args.no_parity else None
        c2 = {"workload": WORKLOADS["c2"][2], "rows_per_gpu": rows2, "value": rows2 * world / (ms / 1e3),
              "ms_per_step": ms, "steps": r2.K, "kernel": r2.kernel_names("fused"),
              "isolated_launch_ms": statistics.mean(kern["fused"]),
              "frac": ab2["total"] / (ms / 1e3) / 1e9 / hbm_peak, "algorithmic_bytes": ab2["total"],
              "l2": "3 rotated copies (3 x 345 MB > 126 MB L2)",
              "parity": None if oc2 is None else {"gpu": res, "match": res == [oc2["sum"], oc2["count"], oc2["cand"],
                                                                                 oc2["def"]] and consistent}}
        del r2
        for qq in copies:
            qq.free()
        torch.cuda.empty_cache()

    c5 = None
    if not args.only and not args.no_c5:
        c5 = bench_c5(ctx, args)

    cpu = cpu1 = None
    if rank == 0 and not args.no_cpu:
        # bounded sample of the same workload: the first 60 M rows of this rank's shard
        sample = gen_columns(seed, table_sf, row0, min(rows, 60_000_000))
        cpu = run_oracle(sample, args.cpu_seconds)
        cpu1 = run_oracle(sample, 0.0, threads=1)   # single-threaded, like the paper's MonetDB baseline
        cpu = {k: v for k, v in cpu.items() if k not in ("sum", "count")}
        cpu1 = {k: v for k, v in cpu1.items() if k not in ("sum", "count")}
        cpu["cpu"] = cpu_info()
    ctx.barrier()
    if ctx.dist_h:
        _ar.ar_dist_free(ctx.dist_h)
    if rank != 0:
        if ctx.pg:
            ctx.pg.destroy_process_group()
        return
    other = {v: {k: results[v][k] for k in ("value", "ms_per_step", "roofline", "gpu_launches", "gpu_kernels")}
             for v in results if v != args.variant}
    strong = args.workload == "c4" and args.scaling == "strong"
    line = {"metric": METRIC, "value": head["value"], "unit": UNIT, "n_gpus": world, "steps": K,
            "warmup": args.warmup, "ms_per_step": head["ms_per_step"], "higher_is_better": True,
            "scaling": "strong" if strong else "weak", "vs_baseline": None, "dtype": "u32", "data": "synthetic",
            "config": config_dict(args.workload, world, rows, table_rows, args.scaling, {
                "variant": args.variant,
                "variant_desc": VARIANT_DESC[args.variant],
                "l2": f"inputs larger than L2: {q_bytes_str(ab, rows)} of decomposed columns per rank (> 126 MB L2)",
                "timing": "K steps = one CUDA-graph replay; CUDA events on the launching stream; barrier + "
                          "synchronize around it; max over ranks; fused step = 1 launch of ar_select_refine_sum_ws "
                          "(PDL, early input reads) [+ SUM allreduce on a side stream]"}),
            "roofline": head["roofline"], "cpu_baseline": cpu, "cpu_baseline_single_thread": cpu1, "e2e": e2e,
            "gpu_launches": head["gpu_launches"], "gpu_kernels": head["gpu_kernels"],
            "clocks": sampler.result(),
            "clocks_replays": sampler.replay_sampler.result() if getattr(sampler, "replay_sampler", None) else None,
            "ms_per_step_replays": head["ms_per_step_replays"],
            "latency": latency,
            "counts": {"candidates": ab["n_cand"], "definite": ab["n_def"], "result": ab["n_result"],
                       "rank0_rows": rows},
            "parity": parity,
            "variants": other, "c2": c2, "c5": c5,
            "hbm_roofline_rows_per_s": hbm_peak * 1e9 / (ab["total"] / rows) * world}
    print(json.dumps(line), flush=True)
    if ctx.pg:
        ctx.pg.destroy_process_group()


def q_bytes_str(ab, rows):
    b = ab["scan"] + rows * (K_SHIP + ab["widths"]["extprice"]) / 8.0
    return f"{b / 1e9:.2f} GB"


def _copy_q6(ctx, q):
    """A second set of handles over copies of q's decomposed buffers (L2 rotation)."""
    c = Q6.__new__(Q6)
    c.sd, c.dc, c.qt, c.ep = q.sd.copy(), q.dc.copy(), q.qt.copy(), q.ep.copy()
    c.rows = q.rows
    c.preds = [(c.sd.handle, *PREDS[0]), (c.dc.handle, *PREDS[1]), (c.qt.handle, *PREDS[2])]
    c.aggs = [c.ep.handle, c.dc.handle]
    c.cols = [c.sd, c.dc, c.qt, c.ep]
    return c


class RotRunner(Runner):
    """Runner over R rotated copies of the same columns (step i reads copy i % R)."""

    def __init__(self, ctx, copies, K):
        super().__init__(ctx, copies[0], K)
        self.copies = copies

    def step(self, variant, i, ev=None, fork=None, pdl=True):
        self.q = self.copies[i % len(self.copies)]
        super().step(variant, i, ev, fork, pdl)


VARIANT_DESC = {
    "fused": "one pass: a3 approximate select + a5 refine (exact predicate on the streamed residual planes) + "
             "a6 SUM with l_extendedprice gathered at result rows, one kernel (ar_select_refine_sum_ws)",
    "staged": "ar_approx_select (ordered candidate relation in HBM) -> [a4 count allgather on a side stream] "
              "-> ar_refine_sum",
}


def main():
    args = parse()
    if args.impl == "reference":
        reference_arm(args)
        return
    ours(args)


if __name__ == "__main__":
    main()
