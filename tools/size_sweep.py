"""Per-query time of the one-pass Q6 query (ar_select_refine_sum_ws, PDL early reads, K queries captured in one
CUDA graph, as bench.py) against the table size: t(N) = fixed + N / rate separates the per-query fixed cost
(launch, pipeline fill / drain, tail, finalize) from the streaming rate.

    python tools/size_sweep.py [sf ...]
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import datagen  # noqa: E402
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu  # noqa: E402


def main():
    sfs = [float(x) for x in sys.argv[1:]] or [2.5, 5, 10, 20, 40, 100]
    K = 100
    pts = []
    s = torch.cuda.Stream()
    for sf in sfs:
        c = datagen.q6_columns(4, sf)
        n = c["shipdate"].size
        # rotate over copies so the columns never sit in L2 across consecutive queries
        copies = max(1, int(np.ceil(400e6 / (n * 5.75))))
        qs = []
        for _ in range(copies):
            sd = cu.BWDColumn(c["shipdate"], 24)
            dc, qt = cu.BWDColumn(c["discount"], 32), cu.BWDColumn(c["quantity"], 32)
            ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
            qs.append(([(sd, *datagen.Q6_SHIPDATE), (dc, *datagen.Q6_DISCOUNT), (qt, *datagen.Q6_QUANTITY)],
                       [ep, dc], (sd, dc, qt, ep)))
        ws = cu.SrsWorkspace()
        out = torch.zeros((K, 4), dtype=torch.int64, device="cuda")
        with torch.cuda.stream(s):
            for i in range(5):
                p, a, _ = qs[i % copies]
                cu.select_refine_sum(p, a, out[i], ws=ws, flags=_ar.AR_SRS_PDL_EARLY_READ, stream=s)
        torch.cuda.synchronize()
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=s):
            for i in range(K):
                p, a, _ = qs[i % copies]
                cu.select_refine_sum(p, a, out[i], ws=ws, flags=_ar.AR_SRS_PDL_EARLY_READ, stream=s)
        torch.cuda.synchronize()
        g.replay()
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        with torch.cuda.stream(s):
            e0.record()
            g.replay()
            e1.record()
        torch.cuda.synchronize()
        us = e0.elapsed_time(e1) / K * 1e3
        pts.append((n, us))
        print({"sf": sf, "rows": n, "copies": copies, "us_per_query": round(us, 2), "kernel": _ar.ar_last_scan_kernel()},
              flush=True)
        del g, qs
        torch.cuda.empty_cache()
    x = np.array([p[0] for p in pts], dtype=np.float64)
    y = np.array([p[1] for p in pts], dtype=np.float64)
    b, a = np.polyfit(x, y, 1)
    print({"fixed_us": round(a, 2), "ns_per_Mrow": round(b * 1e6 * 1e3, 1), "rows_per_s_streaming": 1e6 / b})


if __name__ == "__main__":
    main()
