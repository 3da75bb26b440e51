import sys, os
sys.path.insert(0, '.')
import torch, datagen
from paper_conf_icde_pirkmk14_b200 import column as cu
for mb in (24, 16, 8):
    v = datagen.uniform_u32(3, 10_000_000)
    col = cu.BWDColumn(v, mb)
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum([(col, 0x5A5A5A37, 0x5A5A5A37 + (1 << 32) // 100)], [], o4)
    torch.cuda.synchronize()
    print(mb, o4.tolist(), flush=True)
