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


def _shard_q6(cu, c, s, e):
    """Decompose rows [s, e) as one rank would and run approx_select -> refine and the one-pass query."""
    from paper_conf_icde_pirkmk14_b200 import _ar
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
    return cands, pos, o4


@pytest.mark.parametrize("world", [1, 2, 3, 4, 8])
def test_gpu_logical_shards_match_whole_table(cu, world):
    """Step a4 for every rank of a world-G split on one GPU: the library's shard geometry, the
    exclusive prefix kernel over the gathered counts (ar_dist_exclusive_offsets, rank > 0 included)
    and the placement of each slice (ar_dist_concat_positions) reproduce the whole-table oracle:
    offsets = prefix sums of the oracle's per-shard counts, concatenation = its positions."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    from paper_conf_icde_pirkmk14_b200.dist import shard_range
    n = 1_000_003
    c = datagen.q6_columns(2, 0.2, n=n)
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    ref_pos, ref_cnt, ref_sum = oracle.select_sum(vals, Q6_LO, Q6_HI, [c["extprice"], c["discount"]])
    ranges = [shard_range(n, r, world) for r in range(world)]
    shards = [(_shard_q6(cu, c, s, e) if e > s else None) for s, e in ranges]
    # the gathered count vectors (what ncclAllGather leaves on every rank): refined and candidate counts
    res_counts = torch.zeros(world, dtype=torch.int64, device="cuda")
    cand_counts = torch.zeros(world, dtype=torch.int64, device="cuda")
    for r, sh in enumerate(shards):
        if sh is not None:
            res_counts[r:r + 1].copy_(sh[1].count_t)
            cand_counts[r:r + 1].copy_(sh[0].count_t)
    total = torch.full((1,), -1, dtype=torch.int64, device="cuda")
    glob = torch.full((ref_cnt + 1,), -1, dtype=torch.int64, device="cuda")
    overflow = torch.zeros(1, dtype=torch.int32, device="cuda")
    offs, coffs = [], []
    s_ptr = torch.cuda.current_stream().cuda_stream
    oracle_counts, oracle_cands, sums = [], [], 0
    for r, ((s, e), sh) in enumerate(zip(ranges, shards)):
        off = torch.full((1,), -1, dtype=torch.int64, device="cuda")
        coff = torch.full((1,), -1, dtype=torch.int64, device="cuda")
        _ar.ar_dist_exclusive_offsets(res_counts.data_ptr(), world, r, off.data_ptr(), total.data_ptr(), s_ptr)
        _ar.ar_dist_exclusive_offsets(cand_counts.data_ptr(), world, r, coff.data_ptr(), 0, s_ptr)
        if sh is not None:
            _ar.ar_dist_concat_positions(sh[1].p, s, off.data_ptr(), glob.data_ptr(), ref_cnt, overflow.data_ptr(),
                                         s_ptr)
            sums += int(sh[2][0].item())
            assert int(sh[2][1].item()) == sh[1].count() and int(sh[2][2].item()) == sh[0].count()
        offs.append(off)
        coffs.append(coff)
        _, cnt, _ = oracle.select_sum([v[s:e] for v in vals], Q6_LO, Q6_HI, positions=False)
        cpos, _ = oracle.approx_select([v[s:e] for v in vals], [8, 0, 0], Q6_LO, Q6_HI)
        oracle_counts.append(cnt)
        oracle_cands.append(cpos.size)
    torch.cuda.synchronize()
    want = np.concatenate([[0], np.cumsum(oracle_counts)[:-1]]).tolist()
    cwant = np.concatenate([[0], np.cumsum(oracle_cands)[:-1]]).tolist()
    assert [int(o.item()) for o in offs] == want
    assert [int(o.item()) for o in coffs] == cwant
    if world > 1:
        assert any(w > 0 for w in want[1:])           # rank > 0 offsets really are non-zero
    assert int(total.item()) == ref_cnt and int(overflow.item()) == 0
    g = glob.cpu().numpy()
    assert np.array_equal(g[:ref_cnt], ref_pos) and g[ref_cnt] == -1 and sums == ref_sum


def test_gpu_concat_positions_overflow_flag(cu):
    from paper_conf_icde_pirkmk14_b200 import _ar
    pos = cu.PositionList(16)
    pos.pos[:4] = torch.tensor([1, 5, 9, 12], dtype=torch.int32, device="cuda")
    pos.count_t.fill_(4)
    off = torch.tensor([3], dtype=torch.int64, device="cuda")
    out = torch.full((6,), -1, dtype=torch.int64, device="cuda")
    ovf = torch.zeros(1, dtype=torch.int32, device="cuda")
    s_ptr = torch.cuda.current_stream().cuda_stream
    _ar.ar_dist_concat_positions(pos.p, 100, off.data_ptr(), out.data_ptr(), 6, ovf.data_ptr(), s_ptr)
    torch.cuda.synchronize()
    assert int(ovf.item()) == 1 and out.tolist() == [-1] * 6      # 3 + 4 > 6: nothing written
    out7 = torch.full((7,), -1, dtype=torch.int64, device="cuda")
    ovf.zero_()
    _ar.ar_dist_concat_positions(pos.p, 100, off.data_ptr(), out7.data_ptr(), 7, ovf.data_ptr(), s_ptr)
    torch.cuda.synchronize()
    assert int(ovf.item()) == 0 and out7.tolist() == [-1, -1, -1, 101, 105, 109, 112]


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


def _nccl_worker(rank, world, port, n, q):
    import torch
    import torch.distributed as dist
    from paper_conf_icde_pirkmk14_b200 import column as cu
    from paper_conf_icde_pirkmk14_b200.dist import NcclComm, shard_range
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    torch.cuda.set_device(rank)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    comm = NcclComm(rank, world)
    s, e = shard_range(n, rank, world)
    c = datagen.q6_columns(2, 0.2, n=e - s, row0=s)
    cands, pos, o4 = _shard_q6(cu, c, 0, e - s)
    st = torch.cuda.current_stream().cuda_stream
    allc = torch.zeros(world, dtype=torch.int64, device="cuda")
    off = torch.zeros(1, dtype=torch.int64, device="cuda")
    comm.offsets(pos.count_t.data_ptr(), allc.data_ptr(), off.data_ptr(), st)
    comm.sum(o4.data_ptr(), 2, st)
    torch.cuda.synchronize()
    q.put((rank, int(off.item()), allc.tolist(), (pos.positions().astype(np.int64) + s).tolist(), o4.tolist()[:2]))
    comm.close()
    dist.destroy_process_group()


def test_gpu_nccl_two_ranks():
    """The real exchange over NCCL between two GPUs (skipped on a one-GPU box)."""
    if torch.cuda.device_count() < 2:
        pytest.skip("needs 2 GPUs")
    import torch.multiprocessing as mp
    world, n = 2, 1_000_003
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_nccl_worker, args=(r, world, port, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    got = sorted(q.get(timeout=600) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    c = datagen.q6_columns(2, 0.2, n=n)
    ref_pos, ref_cnt, ref_sum = oracle.select_sum([c["shipdate"], c["discount"], c["quantity"]], Q6_LO, Q6_HI,
                                                  [c["extprice"], c["discount"]])
    glob = np.empty(ref_cnt, dtype=np.int64)
    for rank, off, allc, gpos, sc in got:
        assert sum(allc) == ref_cnt and sc == [ref_sum, ref_cnt]
        glob[off:off + len(gpos)] = gpos
    assert got[1][1] == got[0][2][0] > 0
    assert np.array_equal(glob, ref_pos)
