"""Multi-GPU rotation sharding (production FTMap distributes rotations across nodes,
P:L960-962; the paper's future multi-GPU plan).

Every (probe, rotation) unit is scored and filtered independently (the filter is per rotation,
P:L168-170), so ranks take contiguous, equal blocks of the probe-major unit space and no data-path
exchange is needed until the very end, where ONE all-gather (NCCL over NVLink on GPUs, gloo in the
CPU tests) assembles the fixed-size pose blocks.

Data plane (``PoseGather``): the receive buffer of the all-gather ``[world * U][k][4]`` int32 is
allocated once; this rank's docking call writes its poses straight into its slot of that buffer
(``dock_probe_batch`` with device output is asynchronous), and one in-place
``all_gather_into_tensor`` -- enqueued behind the docking kernels, no host synchronisation --
assembles every rank's block.  No per-call allocation, copy or concatenation (uneven shards are
compacted by one preallocated index_select).
"""
from __future__ import annotations

from typing import Callable, Dict, Tuple

import torch
import torch.distributed as dist


def shard_range(n_units: int, rank: int, world: int) -> Tuple[int, int]:
    """Contiguous block of units owned by ``rank`` (sizes differ by at most one)."""
    if world < 1 or not 0 <= rank < world:
        raise ValueError("bad rank/world")
    return (n_units * rank) // world, (n_units * (rank + 1)) // world


def block_size(n_units: int, world: int) -> int:
    return -(-n_units // world)


class PoseGather:
    """Preallocated in-place all-gather of per-rank pose blocks ``[U_r][k][4]`` int32."""

    def __init__(self, n_units: int, k: int, device, group=None):
        self.group = group
        self.world = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.n_units, self.k = n_units, k
        self.begin, self.end = shard_range(n_units, self.rank, self.world)
        self.U = block_size(n_units, self.world)
        self.recv = torch.full((self.world * self.U, k, 4), -1, dtype=torch.int32, device=device)
        o = self.rank * self.U
        self.send = self.recv[o:o + self.U]                      # in-place: input = this rank's slot
        self.slot = self.recv[o:o + (self.end - self.begin)]     # what the docking kernels write
        if self.world * self.U == n_units:
            self.index = None
            self.out = self.recv
        else:   # uneven shards: drop each block's padding with one preallocated gather
            idx = [r * self.U + i for r in range(self.world)
                   for i in range(shard_range(n_units, r, self.world)[1] - shard_range(n_units, r, self.world)[0])]
            self.index = torch.tensor(idx, dtype=torch.long, device=device)
            self.out = torch.empty((n_units, k, 4), dtype=torch.int32, device=device)

    def gather(self) -> torch.Tensor:
        """One all_gather_into_tensor over the group -> ``[n_units][k][4]`` (every rank's poses)."""
        dist.all_gather_into_tensor(self.recv, self.send, group=self.group)
        if self.index is not None:
            torch.index_select(self.recv, 0, self.index, out=self.out)
        return self.out


_GATHERS: Dict[tuple, PoseGather] = {}


def pose_gather(n_units: int, k: int, device, group=None) -> PoseGather:
    """The cached PoseGather for this shape, device and group (allocated on first use)."""
    key = (n_units, k, str(torch.device(device)), id(group), dist.get_world_size(group), dist.get_rank(group))
    pg = _GATHERS.get(key)
    if pg is None:
        pg = _GATHERS[key] = PoseGather(n_units, k, device, group)
    return pg


def gather_poses(local: torch.Tensor, n_units: int, group=None) -> torch.Tensor:
    """All-gather per-rank pose blocks ``[U_r][k][4]`` int32 into ``[n_units][k][4]``.  When ``local``
    already is this rank's slot of the cached buffer (the docking call wrote there) nothing is copied."""
    pg = pose_gather(n_units, local.shape[1], local.device, group)
    if local.shape[0] != pg.end - pg.begin:
        raise ValueError("local block size does not match this rank's shard")
    if local.data_ptr() != pg.slot.data_ptr():
        pg.slot.copy_(local)
    return pg.gather()


def dock_sharded(dock_block: Callable[[int, int], torch.Tensor], n_units: int, group=None) -> torch.Tensor:
    """Run ``dock_block(begin, end) -> [end-begin][k][4] int32`` on this rank's shard and all-gather the
    result.  The CPU tests plug in the oracle; on GPUs ``dock_probe_sharded`` writes in place instead."""
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    b, e = shard_range(n_units, rank, world)
    return gather_poses(dock_block(b, e), n_units, group)


def dock_probe_sharded(ctx, probes, rot, k: int = 4, rho: int = 1, group=None, sync: bool = True) -> torch.Tensor:
    """Multi-GPU hot path: this rank docks its unit block with libdock directly into its slot of the
    all-gather buffer (asynchronous), then one NCCL all-gather assembles every rank's poses on every
    rank.  ``sync=False`` leaves the step fully asynchronous (call ``dock_sync`` later for errors)."""
    from .dock import dock_probe_batch, dock_sync
    n_units = len(probes) * int(rot.shape[0])
    pg = pose_gather(n_units, k, torch.device("cuda", ctx.device), group)
    if pg.end > pg.begin:
        dock_probe_batch(ctx, probes, rot, pg.begin, pg.end, k, rho, out=pg.slot)
    full = pg.gather()
    if sync:
        dock_sync(ctx)
    return full
