"""Read-bandwidth reference points on this GPU: torch reductions and copies over
buffers of the C2 scan size (165 MB) and of 2 GB, back-to-back, CUDA events.
Rotates 3 buffers so nothing is served from L2."""
import json
import torch

def bench(fn, reps=30):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record()
    for _ in range(reps):
        fn()
    b.record()
    torch.cuda.synchronize()
    return a.elapsed_time(b) / reps

for mb in (165, 330, 2048):
    n = mb * 1024 * 1024 // 4
    xs = [torch.ones(n, dtype=torch.int32, device="cuda") for _ in range(3)]
    ys = [torch.empty_like(x) for x in xs]
    i = [0]
    def red():
        i[0] += 1
        return xs[i[0] % 3].sum()
    def cp():
        i[0] += 1
        ys[i[0] % 3].copy_(xs[i[0] % 3])
    ms_r = bench(red)
    ms_c = bench(cp)
    print(json.dumps({"MB": mb, "sum_us": ms_r * 1e3, "sum_read_gbs": n * 4 / ms_r / 1e6,
                      "copy_us": ms_c * 1e3, "copy_rw_gbs": 2 * n * 4 / ms_c / 1e6}))
    del xs, ys
