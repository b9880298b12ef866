"""Multi-rank host logic on CPU: rotation sharding + the single all-gather (gloo, world 2),
with the FP64 oracle as the per-rank "kernel".  Sharded results must equal 1-rank results."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import dockgen as g


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _oracle_block(R, w, probes, rot, k, rho, b, e):
    import oracle
    t, s, st = oracle.dock(R, w, g.SPACING, probes, rot, k, rho, unit_begin=b, unit_end=e, n_threads=1)
    out = np.zeros((e - b, k, 4), dtype=np.int32)
    out[..., 0] = (np.arange(b, e) % len(rot))[:, None]
    out[..., 1] = t
    out[..., 2] = s.astype(np.float32).view(np.int32)
    return torch.from_numpy(out)


def _worker(rank, world, port, n_units_cfg, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ipps_sukhwanih10_b200 import parallel
        R = g.receptor_ftmap_like((16, 16, 16), 2)
        w = g.weights(2)
        probes = g.probes(2, 3, 2)
        rot = g.rotations(n_units_cfg)
        n_units = len(probes) * len(rot)
        full = parallel.dock_sharded(lambda b, e: _oracle_block(R, w, probes, rot, 3, 1, b, e), n_units)
        q.put((rank, full.numpy()))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,n_rot", [(2, 5), (2, 4), (3, 1)])
def test_sharded_equals_single_rank(orc, world, n_rot):
    """(3, 1): 2 units over 3 ranks -- one rank's shard is empty and still joins the all-gather."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n_rot, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    R = g.receptor_ftmap_like((16, 16, 16), 2)
    probes = g.probes(2, 3, 2)
    rot = g.rotations(n_rot)
    ref = _oracle_block(R, g.weights(2), probes, rot, 3, 1, 0, len(probes) * n_rot).numpy()
    assert all(np.array_equal(res[r], ref) for r in range(world))


def _worker_rot(rank, world, port, n_rot, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_ipps_sukhwanih10_b200 import parallel
        R = g.receptor_ftmap_like((16, 16, 16), 2)
        w = g.weights(2)
        probes = g.probes(3, 3, 2)
        rot = g.rotations(n_rot)
        full = parallel.dock_sharded_rotations(
            lambda r0, r1: _oracle_block(R, w, probes, rot[r0:r1], 3, 1, 0, len(probes) * (r1 - r0)),
            len(probes), n_rot, 3)
        q.put((rank, full.numpy()))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world,n_rot", [(2, 5), (3, 7), (3, 2)])
def test_rotation_sharded_equals_single_rank(orc, world, n_rot):
    """The product path's rotation sharding (every rank docks every probe over its rotation slice, the
    all-gather reorders into the global probe-major order and globalises the rotation indices) equals the
    single-rank result; (3, 2): one rank owns no rotation and still joins the all-gather."""
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker_rot, args=(r, world, port, n_rot, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    R = g.receptor_ftmap_like((16, 16, 16), 2)
    probes = g.probes(3, 3, 2)
    rot = g.rotations(n_rot)
    ref = _oracle_block(R, g.weights(2), probes, rot, 3, 1, 0, len(probes) * n_rot).numpy()
    assert all(np.array_equal(res[r], ref) for r in range(world))


def test_shard_ranges_cover_exactly():
    from paper_conf_ipps_sukhwanih10_b200 import parallel
    for n in (1, 7, 8000, 70000):
        for world in (1, 2, 3, 8):
            spans = [parallel.shard_range(n, r, world) for r in range(world)]
            assert spans[0][0] == 0 and spans[-1][1] == n
            assert all(spans[i][1] == spans[i + 1][0] for i in range(world - 1))
            sizes = [e - b for b, e in spans]
            assert max(sizes) - min(sizes) <= 1 and max(sizes) <= parallel.block_size(n, world)
