"""Multi-GPU rotation sharding (production FTMap distributes rotations across nodes,
P:L960-962; the paper's future multi-GPU plan).

Every (probe, rotation) unit is scored and filtered independently (the filter is per rotation,
P:L168-170), so no data-path exchange is needed until the very end, where ONE all-gather (NCCL over
NVLink on GPUs, gloo in the CPU tests) assembles the fixed-size pose blocks.  The product path shards
the ROTATIONS (``RotationGather``, ``dock_probe_sharded``): rank r docks every probe over its contiguous
rotation slice, so every rank gets the same probe mix -- with the occupancy schedule a unit's cost depends
on its probe's size, and contiguous blocks of the probe-major unit space (``shard_range`` over units,
``PoseGather``) would hand whole cheap or expensive probes to single ranks.

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


class RotationGather:
    """Preallocated all-gather for rotation shards.  Rank r docks all ``n_probes`` probes over rotations
    ``[r0, r1)`` (its units probe-major within the slice, rotation indices relative to the slice) straight into
    ``slot``; ``gather`` runs one in-place ``all_gather_into_tensor``, one preallocated ``index_select`` into the
    global probe-major unit order and one add that turns slice-relative rotation indices into global ones."""

    def __init__(self, n_probes: int, n_rot: int, k: int, device, group=None):
        self.group = group
        self.world = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        self.n_probes, self.n_rot, self.k = n_probes, n_rot, k
        self.r0, self.r1 = shard_range(n_rot, self.rank, self.world)
        self.U = n_probes * block_size(n_rot, self.world)
        self.recv = torch.full((self.world * self.U, k, 4), -1, dtype=torch.int32, device=device)
        o = self.rank * self.U
        self.send = self.recv[o:o + self.U]
        self.slot = self.recv[o:o + n_probes * (self.r1 - self.r0)]
        idx, off = [], []
        spans = [shard_range(n_rot, q, self.world) for q in range(self.world)]
        owner = [q for q, (a, b) in enumerate(spans) for _ in range(a, b)]
        for p in range(n_probes):
            for r in range(n_rot):
                q = owner[r]
                a, b = spans[q]
                idx.append(q * self.U + p * (b - a) + (r - a))
                off.append(a)
        self.index = torch.tensor(idx, dtype=torch.long, device=device)
        self.rot_off = torch.tensor(off, dtype=torch.int32, device=device).view(-1, 1)
        self.out = torch.empty((n_probes * n_rot, k, 4), dtype=torch.int32, device=device)

    def gather(self) -> torch.Tensor:
        """-> ``[n_probes * n_rot][k][4]`` in the global probe-major unit order, global rotation indices."""
        dist.all_gather_into_tensor(self.recv, self.send, group=self.group)
        torch.index_select(self.recv, 0, self.index, out=self.out)
        self.out[:, :, 0] += self.rot_off
        return self.out


_GATHERS: Dict[tuple, PoseGather] = {}
_RGATHERS: Dict[tuple, RotationGather] = {}


def rotation_gather(n_probes: int, n_rot: int, k: int, device, group=None) -> RotationGather:
    """The cached RotationGather for this shape, device and group (allocated on first use)."""
    key = (n_probes, n_rot, k, str(torch.device(device)), id(group), dist.get_world_size(group),
           dist.get_rank(group))
    rg = _RGATHERS.get(key)
    if rg is None:
        rg = _RGATHERS[key] = RotationGather(n_probes, n_rot, k, device, group)
    return rg


def dock_sharded_rotations(dock_slice: Callable[[int, int], torch.Tensor], n_probes: int, n_rot: int, k: int,
                           group=None, device="cpu") -> torch.Tensor:
    """Run ``dock_slice(r0, r1) -> [n_probes * (r1 - r0)][k][4] int32`` (every probe over rotations [r0, r1),
    rotation indices relative to r0) on this rank's rotation shard and all-gather the result into the global
    probe-major order.  The CPU tests plug in the oracle; on GPUs ``dock_probe_sharded`` writes in place."""
    rg = rotation_gather(n_probes, n_rot, k, device, group)
    local = dock_slice(rg.r0, rg.r1)
    if local.shape[0] != rg.slot.shape[0]:
        raise ValueError("local block size does not match this rank's rotation shard")
    rg.slot.copy_(local)
    return rg.gather()


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


class BlockShardBuffer:
    """Full-size pose buffer ``[n_units][k][4]`` int32 for block sharding (DOCK_TUNE_SHARD): every rank clusters
    the whole unit range the same way and docks the blocks rank, rank + world, ...; it writes only its units'
    rows, the rest keep the INT32_MIN fill, and one elementwise-MAX all-reduce combines the ranks (every field
    of a written row is > INT32_MIN except the bits of a -0.0 score, which MAX keeps)."""

    def __init__(self, n_units: int, k: int, device, group=None):
        self.group = group
        self.buf = torch.empty((n_units, k, 4), dtype=torch.int32, device=device)

    def reset(self) -> torch.Tensor:
        self.buf.fill_(-2 ** 31)
        return self.buf

    def gather(self) -> torch.Tensor:
        dist.all_reduce(self.buf, op=dist.ReduceOp.MAX, group=self.group)
        return self.buf


_BSHARDS: Dict[tuple, BlockShardBuffer] = {}


def block_shard_buffer(n_units: int, k: int, device, group=None) -> BlockShardBuffer:
    key = (n_units, k, str(torch.device(device)), id(group))
    b = _BSHARDS.get(key)
    if b is None:
        b = _BSHARDS[key] = BlockShardBuffer(n_units, k, device, group)
    return b


def dock_probe_sharded_blocks(ctx, probes, rot, k: int = 4, rho: int = 1, group=None, sync: bool = True):
    """Multi-GPU hot path with block sharding (tcgen05 variant-1 engine): this rank docks its blocks of the
    clustered block order into the full-size buffer (asynchronous), one NCCL all-reduce (MAX) combines the ranks.
    Raises DockError (DOCK_E_UNSUPPORTED) when the call would not run on variant 1."""
    from .dock import dock_probe_batch, dock_set_tuning, dock_sync
    from ._native import DOCK_TUNE_SHARD
    world, rank = dist.get_world_size(group), dist.get_rank(group)
    n_units = len(probes) * int(rot.shape[0])
    bb = block_shard_buffer(n_units, k, torch.device("cuda", ctx.device), group)
    dock_set_tuning(ctx, DOCK_TUNE_SHARD, (world << 16) | rank)
    try:
        dock_probe_batch(ctx, probes, rot, 0, n_units, k, rho, out=bb.reset())
    finally:
        dock_set_tuning(ctx, DOCK_TUNE_SHARD, 1 << 16)
    full = bb.gather()
    if sync:
        dock_sync(ctx)
    return full


def dock_probe_sharded(ctx, probes, rot, k: int = 4, rho: int = 1, group=None, sync: bool = True) -> torch.Tensor:
    """Multi-GPU hot path: this rank docks every probe over its rotation shard with libdock directly into its
    slot of the all-gather buffer (asynchronous), then one NCCL all-gather assembles every rank's poses on every
    rank (global probe-major unit order, global rotation indices).  ``rot`` is ``[n_rot][9]`` (a device tensor
    keeps the slice a view).  ``sync=False`` leaves the step fully asynchronous (``dock_sync`` later)."""
    from .dock import dock_probe_batch, dock_sync
    n_rot = int(rot.shape[0])
    rg = rotation_gather(len(probes), n_rot, k, torch.device("cuda", ctx.device), group)
    if rg.r1 > rg.r0:
        dock_probe_batch(ctx, probes, rot[rg.r0:rg.r1], 0, len(probes) * (rg.r1 - rg.r0), k, rho, out=rg.slot)
    full = rg.gather()
    if sync:
        dock_sync(ctx)
    return full
