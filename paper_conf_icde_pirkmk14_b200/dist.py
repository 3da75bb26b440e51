"""Row-sharded multi-GPU plumbing (step a4): shard geometry + communicator setup.

The table is split into contiguous row ranges, one per rank, with every shard
boundary on a 128-row multiple so each rank's packed bitstreams start 16-B
aligned.  Each rank decomposes and scans its own shard; the
only exchanges are the candidate / result counts (ncclAllGather -> exclusive
prefix = the rank's offset in the concatenated, globally ordered result) and
the int64 SUM (ncclAllReduce), both in libar_b200.so (`ar_dist_*`).
torch.distributed only provides the rendezvous that carries NCCL's unique id.
"""
from __future__ import annotations

from . import _ar


def shard_range(n: int, rank: int, world: int):
    """[start, end) of rank's rows (ar_dist_shard_range: ceil(n / world) rounded up to
    AR_SHARD_ALIGN_ROWS = 128 rows, last shard ragged, trailing shards may be empty)."""
    row0, rows = _ar.ar_dist_shard_range(n, world, rank)
    return row0, row0 + rows


class NcclComm:
    """The library's NCCL communicator for this rank (rendezvous through an initialised torch process group)."""

    def __init__(self, rank: int, world: int, group=None):
        import torch.distributed as dist

        uid = _ar.ar_dist_get_unique_id() if rank == 0 else b""
        obj = [uid]
        dist.broadcast_object_list(obj, src=0, group=group)
        self.handle = _ar.ar_dist_init(obj[0], rank, world)
        self.rank, self.world = rank, world

    def offsets(self, local_count_dev, all_counts_dev, global_offset_dev, stream):
        """ncclAllGather of the local count + the exclusive prefix (ar_dist_offsets)."""
        _ar.ar_dist_offsets(self.handle, local_count_dev, all_counts_dev, global_offset_dev, stream)

    def sum(self, values_dev, n, stream):
        _ar.ar_dist_sum(self.handle, values_dev, n, stream)

    def close(self):
        if self.handle:
            _ar.ar_dist_free(self.handle)
            self.handle = None
