"""Row sharding (step a4) without a multi-GPU box: the library's shard geometry
(ar_dist_shard_range, a host-only entry point of libar_b200.so), and a
world_size-2 gloo run in which each rank takes its shard from the library,
evaluates it (oracle on CPU: no GPU here) and the ranks exchange counts / sums
as ar_dist_offsets / ar_dist_sum do; the concatenation must equal the
whole-table oracle."""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

import datagen
import oracle
from paper_conf_icde_pirkmk14_b200.dist import shard_range

Q6_LO = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
Q6_HI = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]


@pytest.mark.parametrize("n", [0, 1, 127, 128, 1000, 123457, 6_000_000])
@pytest.mark.parametrize("world", [1, 2, 3, 4, 8])
def test_shard_range_partitions(n, world):
    prev = 0
    for r in range(world):
        s, e = shard_range(n, r, world)
        assert s == prev and s <= e <= n
        assert s % 128 == 0 or s == n          # 16-B aligned bitstream starts
        prev = e
    assert prev == n


def exclusive_offsets(counts):
    """Offsets of each rank's slice in the concatenated result (test-side arithmetic)."""
    out, run = [], 0
    for c in counts:
        out.append(run)
        run += int(c)
    return out, run


def test_shard_range_matches_definition():
    # ceil(n / world) rounded up to 128 rows per shard; written out independently
    for n, world in [(600_000_000, 8), (600_000_000, 3), (1000, 8), (128 * 8 + 1, 8), (5, 4)]:
        per = -(-(-(-n // world)) // 128) * 128
        for r in range(world):
            assert shard_range(n, r, world) == (min(n, r * per), min(n, min(n, r * per) + per))


def test_shard_range_rejects_bad_rank():
    from paper_conf_icde_pirkmk14_b200 import _ar
    for n, r, w in [(10, 2, 2), (10, -1, 2), (-1, 0, 1), (10, 0, 0)]:
        with pytest.raises(_ar.ARError):
            shard_range(n, r, w)


def _shard_result(rank, world, n):
    s, e = shard_range(n, rank, world)
    c = datagen.q6_columns(2, 0.05, n=e - s, row0=s)
    values = [c["shipdate"], c["discount"], c["quantity"]]
    pos, cnt, sm = oracle.select_sum(values, Q6_LO, Q6_HI, [c["extprice"], c["discount"]])
    return s, pos, cnt, sm


def _worker(rank, world, port, n, q):
    import torch
    import torch.distributed as dist
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    s, pos, cnt, sm = _shard_result(rank, world, n)
    counts = [torch.zeros(1, dtype=torch.int64) for _ in range(world)]
    dist.all_gather(counts, torch.tensor([cnt], dtype=torch.int64))        # the count allgather (a4)
    offs, total = exclusive_offsets([int(c.item()) for c in counts])
    gsum = torch.tensor([sm, cnt], dtype=torch.int64)
    dist.all_reduce(gsum)                                                   # the SUM allreduce
    q.put((rank, offs[rank], total, (pos + s).tolist(), int(gsum[0]), int(gsum[1])))
    dist.destroy_process_group()


def _free_port():
    with socket.socket() as so:
        so.bind(("127.0.0.1", 0))
        return so.getsockname()[1]


@pytest.mark.parametrize("world", [2])
def test_gloo_row_sharded_q6_matches_whole_table(world):
    n = 300_001                                    # SF 0.05, ragged last shard
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    got = [q.get(timeout=300) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    got.sort()
    c = datagen.q6_columns(2, 0.05, n=n)
    values = [c["shipdate"], c["discount"], c["quantity"]]
    ref_pos, ref_cnt, ref_sum = oracle.select_sum(values, Q6_LO, Q6_HI, [c["extprice"], c["discount"]])
    # concatenating each rank's globally-offset slice reproduces the whole-table result
    glob = np.empty(got[0][2], dtype=np.int64)
    for rank, off, total, gpos, gs, gc in got:
        assert total == ref_cnt and gs == ref_sum and gc == ref_cnt
        glob[off:off + len(gpos)] = gpos
    assert np.array_equal(glob, ref_pos)
