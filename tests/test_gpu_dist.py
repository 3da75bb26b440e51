"""Row-sharded A&R on one GPU (logical shards, S s4 'distributed without a cluster')
and the NCCL exchange calls on a one-rank communicator."""
import os
import socket

import numpy as np
import pytest

import datagen
import oracle

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")

Q6_LO = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
Q6_HI = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


@pytest.mark.parametrize("world", [1, 2, 3, 4, 8])
def test_gpu_logical_shards_match_whole_table(cu, world):
    from paper_conf_icde_pirkmk14_b200 import _ar
    from paper_conf_icde_pirkmk14_b200.dist import exclusive_offsets, shard_range
    n = 1_000_003
    c = datagen.q6_columns(2, 0.2, n=n)
    pieces, counts, sums = [], [], 0
    for r in range(world):
        s, e = shard_range(n, r, world)
        if e == s:
            counts.append(0)
            pieces.append(np.zeros(0, dtype=np.int64))
            continue
        sd = cu.BWDColumn(c["shipdate"][s:e], 24)
        dc = cu.BWDColumn(c["discount"][s:e], 32)
        qt = cu.BWDColumn(c["quantity"][s:e], 32)
        ep = cu.BWDColumn(c["extprice"][s:e], 32, layout=_ar.AR_LAYOUT_PACKED)
        preds = [(sd, Q6_LO[0], Q6_HI[0]), (dc, Q6_LO[1], Q6_HI[1]), (qt, Q6_LO[2], Q6_HI[2])]
        cands = cu.CandidateList(e - s)
        cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(e - s)))
        pos = cu.PositionList(e - s)
        cu.refine(cands, preds, pos, cu.Workspace(_ar.ar_refine_ws_bytes(e - s)))
        o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
        cu.select_refine_sum(preds, [ep, dc], o4)
        torch.cuda.synchronize()
        local = pos.positions()
        counts.append(local.size)
        pieces.append(local + s)                      # global position = shard row base + local
        sums += int(o4[0].item())
        assert int(o4[1].item()) == local.size
    offs, total = exclusive_offsets(counts)
    glob = np.empty(total, dtype=np.int64)
    for off, p in zip(offs, pieces):
        glob[off:off + p.size] = p
    ref_pos, ref_cnt, ref_sum = oracle.select_sum([c["shipdate"], c["discount"], c["quantity"]], Q6_LO, Q6_HI,
                                                  [c["extprice"], c["discount"]])
    assert np.array_equal(glob, ref_pos) and total == ref_cnt and sums == ref_sum


def _free_port():
    with socket.socket() as so:
        so.bind(("127.0.0.1", 0))
        return so.getsockname()[1]


def test_gpu_nccl_exchange_single_rank(cu):
    import torch.distributed as dist
    from paper_conf_icde_pirkmk14_b200.dist import NcclComm
    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    os.environ["MASTER_PORT"] = str(_free_port())
    dist.init_process_group("gloo", rank=0, world_size=1)
    try:
        comm = NcclComm(0, 1)
        s = torch.cuda.current_stream().cuda_stream
        local = torch.tensor([12345], dtype=torch.int64, device="cuda")
        allc = torch.zeros(1, dtype=torch.int64, device="cuda")
        off = torch.full((1,), -1, dtype=torch.int64, device="cuda")
        comm.offsets(local.data_ptr(), allc.data_ptr(), off.data_ptr(), s)
        vals = torch.tensor([7, 11], dtype=torch.int64, device="cuda")
        comm.sum(vals.data_ptr(), 2, s)
        torch.cuda.synchronize()
        assert allc.tolist() == [12345] and off.tolist() == [0] and vals.tolist() == [7, 11]
        comm.close()
    finally:
        dist.destroy_process_group()
