"""GPU parity: the CUDA path (through the C ABI) against the FP64 oracle.

Bars: voxel indices bit-exact; score grids |S_gpu - S_orc| <= 1e-4 * A;
integer-valued inputs bitwise; poses validated tie-aware (tests/validator.py); results
invariant (bitwise) to batch position, batch size, launch configuration and shard range.
"""
import concurrent.futures as cf

import numpy as np
import pytest

import dockgen as g
from validator import validate_unit

pytestmark = pytest.mark.gpu
H = g.SPACING


@pytest.fixture(scope="module")
def D():
    import torch
    assert torch.cuda.is_available(), "GPU tests need a CUDA device"
    from paper_conf_ipps_sukhwanih10_b200 import build
    build.build_native()
    import paper_conf_ipps_sukhwanih10_b200 as D
    return D


# engine ids used by the tests: 1 = FP32 FFMA; 2 = tcgen05 variant 1 (one channel group, resident receptor
# boxes, 128 translations x 4 rows); 3 = tcgen05 variant 2 (receptor streamed per (channel group, z-plane),
# any P, 64 / 128 / 160 translations per row); 4 = sparse ligand (FP32 gathers of per-atom channel grids at
# the occupied voxels, NEXT-3).  A tcgen05 variant that cannot run a case runs the other one.
ENGINES = [1, 2, 3, 4]


def _ctx(D, R, w, m_max, engine=0):
    ctx = D.dock_init(R, w, H, m_max=m_max)
    ctx.test_engine = engine
    if engine:
        D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, {1: 1, 2: 2, 3: 2, 4: 4}[engine])
        if engine in (2, 3):
            D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_VARIANT, engine - 1)
    return ctx


def _engine_id(info):
    e = info["engine_last"]
    return {1: 1, 4: 4}.get(e, 1 + info["tc_variant_last"])


def _oracle_SA(orc, R, w, pr, q):
    L = orc.voxelize(pr.xyz, pr.coef, pr.m, q, H)
    return orc.score_grid(R, L, w)


def _oracle_units(orc, R, w, probes, rot, units, threads=8):
    def one(u):
        pr, r = probes[u // len(rot)], u % len(rot)
        return _oracle_SA(orc, R, w, pr, rot[r])
    with cf.ThreadPoolExecutor(threads) as ex:
        return list(ex.map(one, units))


# ----------------------------------------------------------------------------- voxelize


@pytest.mark.parametrize("m", [1, 2, 3, 4, 5, 8])
def test_voxelize_matches_oracle(D, orc, m):
    P = 3
    R = g.receptor_uniform((16, 16, 16), P)
    ctx = D.dock_init(R, g.weights(P), H, m_max=8)
    rot = g.rotations(40, with_cube_group=True)
    for i in range(3):
        pr = g.probe(i, m, P) if m > 1 else g.Probe(np.zeros((1, 3)), np.ones((1, P), np.float32), 1)
        Lg = D.dock_voxelize(ctx, pr, rot)
        for r in range(rot.shape[0]):
            Lo = orc.voxelize(pr.xyz, pr.coef, m, rot[r], H)
            assert np.array_equal(Lg[r] != 0, Lo != 0)
            assert np.allclose(Lg[r], Lo, rtol=1e-6, atol=1e-6)
    ctx.close()


def _golden_voxel_cases():
    import os
    path = os.path.join(os.path.dirname(__file__), "golden", "voxelize_cases.txt")
    for line in open(path):
        if line.startswith("#") or not line.strip():
            continue
        m, x, v = line.split()
        yield int(m), float(x), int(v)


def test_voxelize_golden_cases_on_gpu(D):
    """tests/golden/voxelize_cases.txt (reading Q3) replayed through the C ABI on
    all three axes: dock_voxelize must put the atom on the hand-derived voxel, and both dock_voxelize
    and the hot path (dock_probe) must return DOCK_E_PROBE_OUTSIDE_GRID for the rows marked -1."""
    ctx = D.dock_init(g.receptor_uniform((16, 16, 16), 1), np.ones(1, np.float32), H, m_max=4)
    for m, x, v in _golden_voxel_cases():
        for axis in range(3):
            xyz = np.zeros((1, 3))
            xyz[0, axis] = x
            pr = g.Probe(xyz, np.ones((1, 1), np.float32), m)
            eye = np.eye(3).reshape(1, 9)
            if v < 0:
                with pytest.raises(D.DockError) as e:
                    D.dock_voxelize(ctx, pr, eye)
                assert e.value.status == -3, (m, x, axis)
                with pytest.raises(D.DockError) as e:
                    D.dock_probe(ctx, pr, eye, k=1, rho=0)
                assert e.value.status == -3, (m, x, axis)
                continue
            L = D.dock_voxelize(ctx, pr, eye)
            c = int(np.floor((m - 1) / 2.0 + 0.5))
            want = [c, c, c]
            want[axis] = v
            assert np.argwhere(L[0, 0] != 0).tolist() == [[want[2], want[1], want[0]]], (m, x, axis)
    ctx.close()


@pytest.mark.parametrize("m", [2, 3, 4, 5, 8])
def test_voxelize_half_voxel_boundaries_bitwise(D, orc, m):
    """Atoms placed so that Q x / h lands within 1e-9 A of a rounding boundary (k + 1/2 - c) under random
    rotations: the GPU's voxel indices equal the FP64 oracle's bit for bit (reading Q18).  An FP32 copy of
    h (0.8f = 0.800000011920929) would move g by ~2e-8 and flip these cases."""
    rng = np.random.default_rng(1800 + m)
    P = 1
    ctx = D.dock_init(g.receptor_uniform((16, 16, 16), P), np.ones(P, np.float32), H, m_max=8)
    rot = g.rotations(24, seed=77)
    c = (m - 1) / 2.0
    n_checked = 0
    for r in range(len(rot)):
        Q = rot[r].reshape(3, 3)
        atoms = []
        for a in range(8):
            y = (rng.integers(0, m, 3) - c) * H              # voxel centres ...
            axis = int(rng.integers(0, 3))
            kk = int(rng.integers(0, m - 1))
            eps = float(rng.choice([-1e-9, 0.0, 1e-9]))
            y[axis] = (kk + 0.5 - c) * H + eps               # ... with one coordinate on a boundary
            atoms.append(Q.T @ y)                            # so that Q x = y up to rounding
        xyz = np.array(atoms)
        coef = (2.0 ** np.arange(len(atoms))).astype(np.float32).reshape(-1, 1)   # exact sums identify atoms
        pr = g.Probe(xyz, coef, m)
        try:
            Lo = orc.voxelize(xyz, coef, m, rot[r], H)
        except orc.OracleError:
            with pytest.raises(D.DockError) as e:
                D.dock_voxelize(ctx, pr, rot[r:r + 1])
            assert e.value.status == -3
            continue
        Lg = D.dock_voxelize(ctx, pr, rot[r:r + 1])[0]
        assert np.array_equal(Lg.astype(np.float64), Lo), f"rotation {r}"
        n_checked += 1
    assert n_checked >= len(rot) // 2
    ctx.close()


# ----------------------------------------------------------------------------- score grids


@pytest.mark.parametrize("shape,m,P,kind", [
    ((128, 12, 10), 4, 4, "ftmap"),     # lanes_x = 16 path, ragged y/z tiles
    ((64, 20, 11), 5, 4, "uniform"),    # lanes_x = 8 path
    ((37, 13, 9), 4, 2, "uniform"),     # lanes_x = 4 path, ragged everywhere
    ((40, 24, 24), 8, 3, "uniform"),    # largest probe grid
    ((33, 17, 19), 1, 1, "uniform"),    # m = 1
    ((64, 12, 9), 4, 8, "ftmap"),       # two channel groups (variant 2, 64 translations x 8 rows)
    ((160, 7, 6), 8, 22, "uniform"),    # large-config channels: six groups, 160 translations x 3 rows
    ((96, 10, 7), 6, 13, "uniform"),    # four groups, ragged last group, 128-wide rows over nx = 96
])
@pytest.mark.parametrize("engine", ENGINES)
def test_score_grid_within_tolerance(D, orc, shape, m, P, kind, engine):
    R = g.receptor(kind, shape, P)
    w = g.weights(P)
    ctx = _ctx(D, R, w, m, engine)
    rot = g.rotations(4)
    for i, q in enumerate(rot):
        pr = g.probe(i + 1, m, P) if m > 1 else g.Probe(np.zeros((1, 3)), np.ones((1, P), np.float32), 1)
        S_g, C_g = D.dock_score_grid(ctx, pr, q, per_term=True)
        S_o, A_o = _oracle_SA(orc, R, w, pr, q)
        err = np.abs(S_g.astype(np.float64) - S_o)
        assert (err <= 1e-4 * A_o + 1e-12).all(), f"max err/A {np.max(err / np.maximum(A_o, 1e-30))}"
        # per-term grids are the unweighted C_p: S = sum_p w_p C_p (reading Q6)
        L = orc.voxelize(pr.xyz, pr.coef, m, q, H)
        for p in range(P):
            e = np.eye(P, dtype=np.float32)[p]
            Cp, Ap = orc.score_grid(R, L, e)
            assert (np.abs(C_g[p] - Cp) <= 1e-4 * Ap + 1e-12).all()
    ctx.close()


@pytest.mark.parametrize("engine", [1, 4])   # bf16x3 is exact only to ~2^-24 relative: FFMA and sparse engines
def test_delta_probe_bitwise(D, engine):
    """P4: one atom at the centre, m = 1, coef = e_p -> S == R_p bitwise on the GPU."""
    P = 3
    R = g.receptor_uniform((40, 18, 12), P)
    ctx = _ctx(D, R, np.ones(P, np.float32), 1, engine)
    for p in range(P):
        coef = np.zeros((1, P), np.float32)
        coef[0, p] = 1
        S = D.dock_score_grid(ctx, g.Probe(np.zeros((1, 3)), coef, 1), np.eye(3).reshape(9))
        assert np.array_equal(S, R[p])
    ctx.close()


@pytest.mark.parametrize("engine", [1, 4])
def test_shift_equivariance_bitwise(D, engine):
    """P5: single atom on voxel v0 -> S = roll(R, -v0) bitwise."""
    R = g.receptor_uniform((24, 20, 16), 1)
    ctx = _ctx(D, R, np.ones(1, np.float32), 4, engine)
    for v0 in [(0, 0, 0), (3, 1, 2), (1, 3, 3)]:
        pr = g.voxel_centre_probe([v0], 4, 1)
        S = D.dock_score_grid(ctx, pr, np.eye(3).reshape(9))
        assert np.array_equal(S, np.roll(R[0], (-v0[2], -v0[1], -v0[0]), axis=(0, 1, 2)))
    ctx.close()


@pytest.mark.parametrize("engine", ENGINES)
def test_integer_inputs_bitwise_grid(D, orc, engine):
    """P9: integer-valued inputs -> the FP32 score grid equals the FP64 oracle exactly."""
    P, m = 4, 4
    R = g.receptor_integer((48, 20, 18), P)
    w = g.weights_integer(P)
    ctx = _ctx(D, R, w, m, engine)
    rot = g.rotations(3, with_cube_group=True)[:6]
    for i, q in enumerate(rot):
        pr = g.probe(i, m, P, integer=True)
        S_g = D.dock_score_grid(ctx, pr, q)
        S_o, _ = _oracle_SA(orc, R, w, pr, q)
        assert np.array_equal(S_g.astype(np.float64), S_o)
    ctx.close()


# ----------------------------------------------------------------------------- poses


def _dock_and_validate(D, orc, R, w, probes, rot, k, rho, units=None, engine=0):
    ctx = _ctx(D, R, w, max(p.m for p in probes), engine)
    poses = D.dock_probe_batch(ctx, probes, rot, k=k, rho=rho)
    info = D.dock_get_info(ctx)
    ctx.close()
    n_units = len(probes) * len(rot)
    units = list(range(n_units)) if units is None else units
    SA = _oracle_units(orc, R, w, probes, rot, units)
    mism = 0
    for u, (S, A) in zip(units, SA):
        assert (poses[u]["rot"] == u % len(rot)).all()
        mism += validate_unit(S, A, poses[u]["t_lin"], poses[u]["score"], k, rho)
    return poses, info, mism


@pytest.mark.parametrize("engine", ENGINES)
@pytest.mark.parametrize("rho,k", [(0, 1), (0, 4), (1, 1), (1, 4), (2, 3)])
def test_poses_toy_config(D, orc, rho, k, engine):
    c = g.CONFIGS["toy"]
    R = g.receptor_ftmap_like(c.n, c.P)
    w = g.weights(c.P)
    probes = g.probes(2, c.m, c.P)
    rot = g.rotations(c.n_rot, with_cube_group=True)
    _dock_and_validate(D, orc, R, w, probes, rot, k, rho, engine=engine)


@pytest.mark.parametrize("engine", ENGINES)
@pytest.mark.parametrize("kind", ["ftmap", "uniform"])
@pytest.mark.parametrize("rho", [0, 1])
def test_poses_mid_config(D, orc, kind, rho, engine):
    P, m = 4, 4
    R = g.receptor(kind, (48, 40, 36), P)
    w = g.weights(P)
    probes = g.probes(3, m, P)
    rot = g.rotations(21)
    _, info, mism = _dock_and_validate(D, orc, R, w, probes, rot, 4, rho, engine=engine)
    assert _engine_id(info) == engine
    assert info["fallback_last"] <= 2


def test_tc_dynamic_scheduler_across_rotation_blocks(D, orc):
    """tcgen05 variant 1 runs one persistent CTA per SM that takes 4-tile chunks of (rotation block, tiles)
    from per-CTA segments of the chunk space and then helps other segments: with 3 blocks of 128 rotations
    and 370 tiles per block, a CTA's lists change block mid-stream and every block has many publishers.
    Poses validate against the oracle on units of every block (first / last rotations of each), and the
    bits equal region mode's (DOCK_TUNE_REGIONS > 0: one CTA per (block, region)), other chunk sizes' and
    the exact fallback's."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 37), P)
    w = g.weights(P)
    probes = g.probes(3, m, P)
    rot = g.rotations(110)
    n = len(probes) * len(rot)
    units = sorted({0, 1, 127, 128, 129, 255, 256, 257, n - 1} | set(range(120, 136)))
    poses, info, _ = _dock_and_validate(D, orc, R, w, probes, rot, 4, 1, units=units, engine=2)
    assert info["engine_last"] == 2 and info["tc_variant_last"] == 1
    assert info["regions_last"] == 0 and info["items_last"] <= info["n_sms"]   # dynamic scheduler
    ctx = _ctx(D, R, w, m, 2)

    def bits(p):
        return p["rot"], p["t_lin"], p["score"].view(np.uint32)

    for G in (1, 4):
        D.dock_set_tuning(ctx, D.DOCK_TUNE_REGIONS, G)
        reg = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        assert all(np.array_equal(a, b) for a, b in zip(bits(reg), bits(poses)))
    D.dock_set_tuning(ctx, D.DOCK_TUNE_REGIONS, 0)
    for chunk in (1, 7, 370, 4096):
        D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_CHUNK, chunk)
        for _ in range(2):   # back to back: the scheduler's counters reset themselves between launches
            dyn = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
            assert all(np.array_equal(a, b) for a, b in zip(bits(dyn), bits(poses))), chunk
    D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_CHUNK, 0)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 1)
    fb = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    assert (fb["flags"] & D.DOCK_POSE_FALLBACK).all()
    assert all(np.array_equal(a, b) for a, b in zip(bits(fb), bits(poses)))
    ctx.close()


def test_tc_occupancy_schedule_modes(D, orc):
    """tcgen05 variant 1 runs only the ring stages (4 K-steps) where some rotation of a block has a nonzero
    weight, after grouping the units into blocks with few distinct active stages (DOCK_TUNE_TC_SCHEDULE 0).
    Skipped products are exact zeros, so poses (rotation, t_lin and score bits) equal those of the occupancy
    schedule over consecutive units (1), of the dense schedule (2) and of the exact fallback; the executed
    K-steps per row do not grow 2 -> 1 -> 0 and the clustered schedule runs fewer than the dense one.  Units of every block validate against the oracle; probes of 0..8 atoms (an empty
    probe: all-zero blocks run one padding stage)."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 37), P)
    w = g.weights(P)
    probes = g.probes(6, m, P) + [g.Probe(np.zeros((0, 3)), np.zeros((0, P), np.float32), m)]
    rot = g.rotations(70)
    n = len(probes) * len(rot)
    ctx = _ctx(D, R, w, m, 2)

    def bits(p):
        return p["rot"], p["t_lin"], p["score"].view(np.uint32)

    out, ks = {}, {}
    for sched in (2, 1, 0):
        D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_SCHEDULE, sched)
        out[sched] = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        info = D.dock_get_info(ctx)
        assert info["engine_last"] == 2 and info["tc_variant_last"] == 1
        ks[sched] = info["tc_ksteps_exec_last"]
    assert ks[2] == 48.0 and ks[0] <= ks[1] <= ks[2] and ks[0] < ks[2], ks
    for sched in (1, 0):
        assert all(np.array_equal(a, b) for a, b in zip(bits(out[sched]), bits(out[2]))), sched
    D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 1)
    fb = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 0)
    assert all(np.array_equal(a, b) for a, b in zip(bits(fb), bits(out[0])))
    ctx.close()
    units = sorted({0, 69, 70, 139, 200, 333, 350, 419, n - 70, n - 1})
    SA = _oracle_units(orc, R, w, probes, rot, units)
    mism = 0
    for u, (S, A) in zip(units, SA):
        assert (out[0][u]["rot"] == u % len(rot)).all()
        mism += validate_unit(S, A, out[0][u]["t_lin"], out[0][u]["score"], 4, 1)
    assert mism == 0


def test_tc_occupancy_schedule_two_windows(D, orc):
    """More units than one clustering window (8192): two windows are clustered independently, blocks never
    straddle them, and the clustered schedule's poses equal the dense schedule's bitwise; sampled units of
    both windows validate against the oracle."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 37), P)
    w = g.weights(P)
    probes = g.probes(17, m, P)
    rot = g.rotations(500)   # 8500 units
    n = len(probes) * len(rot)
    ctx = _ctx(D, R, w, m, 2)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_SCHEDULE, 2)
    dense = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_SCHEDULE, 0)
    clus = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    info = D.dock_get_info(ctx)
    ctx.close()
    assert info["tc_variant_last"] == 1 and info["tc_ksteps_exec_last"] < 48.0
    for f in ("rot", "t_lin"):
        assert np.array_equal(clus[f], dense[f])
    assert np.array_equal(clus["score"].view(np.uint32), dense["score"].view(np.uint32))
    units = [0, 4000, 8191, 8192, 8300, n - 1]
    for u, (S, A) in zip(units, _oracle_units(orc, R, w, probes, rot, units)):
        validate_unit(S, A, clus[u]["t_lin"], clus[u]["score"], 4, 1)   # raises on a violation (ties may differ)


def test_tc_occupancy_schedule_integer_exact(D, orc):
    """Clustered occupancy schedule (> 128 units; m = 3 and 2 on the mask histogram, m = 5 on the unit greedy
    where variant 1 runs it) on integer inputs: poses equal the FP64 oracle exactly, ties included (P9)."""
    P = 4
    R = g.receptor_integer((40, 24, 20), P, lo=-2, hi=2)
    w = g.weights_integer(P)
    for m, n_rot in ((3, 60), (2, 50), (5, 50)):   # m = 5: 32-stage masks, the unit greedy (k_tc_cluster)
        probes = g.probes(3, m, P, integer=True)
        rot = g.rotations(n_rot)
        ctx = _ctx(D, R, w, m, 2)
        poses = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        info = D.dock_get_info(ctx)
        assert info["engine_last"] == 2
        if m <= 4:
            assert info["tc_variant_last"] == 1 and info["tc_ksteps_exec_last"] > 0
        ctx.close()
        t_o, s_o, st = orc.dock(R, w, H, probes, rot, 4, 1)
        assert (st == 0).all()
        assert np.array_equal(poses["t_lin"], t_o.astype(np.int32))
        assert np.array_equal(poses["score"].astype(np.float64), s_o)


@pytest.mark.parametrize("world", [2, 3, 8])
def test_block_sharding_emulated_ranks(D, world):
    """DOCK_TUNE_SHARD (multi-GPU block sharding), every rank emulated on this GPU: each rank clusters the whole
    unit range (deterministically: every rank must get the same block order), docks the blocks rank, rank +
    world, ... and writes only its units' rows of an INT32_MIN-filled buffer; the elementwise int32 MAX over the
    ranks' buffers equals the single-GPU result bitwise, and every row was written by exactly one rank."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 37), P)
    w = g.weights(P)
    probes = g.probes(7, m, P)
    rot = g.rotations(90)   # 630 units = 5 blocks (a rank may own none at world = 8)
    n = len(probes) * len(rot)
    ctx = _ctx(D, R, w, m, 2)
    ref = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    import torch
    bufs = []
    for r in range(world):   # device output: rows of other ranks' units keep the INT32_MIN fill
        D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, (world << 16) | r)
        out = torch.full((n, 4, 4), -2 ** 31, dtype=torch.int32, device="cuda")
        D.dock_probe_batch(ctx, probes, rot, k=4, rho=1, out=out)
        D.dock_sync(ctx)
        bufs.append(out.cpu().numpy())
    D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, 1 << 16)
    ctx.close()
    written = np.stack([(b != np.iinfo(np.int32).min).any(axis=(1, 2)) for b in bufs])
    assert (written.sum(0) == 1).all()
    comb = np.maximum.reduce(bufs)
    assert np.array_equal(comb, ref.view(np.int32).reshape(n, 4, 4))


@pytest.mark.parametrize("engine", ENGINES)
@pytest.mark.parametrize("rho,k", [(0, 4), (1, 4), (0, 1)])
def test_integer_inputs_exact_poses(D, orc, rho, k, engine):
    """P9: integer inputs -> poses (t_lin and score) equal the oracle exactly, ties included."""
    P, m = 4, 3
    R = g.receptor_integer((40, 24, 20), P, lo=-2, hi=2)
    w = g.weights_integer(P)
    probes = g.probes(2, m, P, integer=True)
    rot = g.rotations(10)
    ctx = _ctx(D, R, w, m, engine)
    poses = D.dock_probe_batch(ctx, probes, rot, k=k, rho=rho)
    ctx.close()
    t_o, s_o, st = orc.dock(R, w, H, probes, rot, k, rho)
    assert (st == 0).all()
    assert np.array_equal(poses["t_lin"], t_o.astype(np.int32))
    assert np.array_equal(poses["score"].astype(np.float64), s_o)


@pytest.mark.parametrize("engine", ENGINES)
def test_fallback_path_identical(D, engine):
    """The exact full-grid fallback returns the same poses (bitwise: t_lin and score bits) as the
    candidate path, on every engine: the fallback's score grids come from the engine that produced the
    candidates (tcgen05 GRID epilogue for engines 2/3, FFMA for engine 1)."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 36), P)
    w = g.weights(P)
    probes = g.probes(2, m, P)
    rot = g.rotations(13)
    ctx = _ctx(D, R, w, m, engine)
    for rho in (0, 1):
        a = D.dock_probe_batch(ctx, probes, rot, k=4, rho=rho)
        assert _engine_id(D.dock_get_info(ctx)) == engine
        D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 1)
        b = D.dock_probe_batch(ctx, probes, rot, k=4, rho=rho)
        assert D.dock_get_info(ctx)["fallback_last"] == len(probes) * len(rot)
        D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 0)
        assert np.array_equal(a["t_lin"], b["t_lin"])
        assert np.array_equal(a["score"].view(np.uint32), b["score"].view(np.uint32))
        assert (b["flags"] & D.DOCK_POSE_FALLBACK).all()
    ctx.close()


@pytest.mark.parametrize("engine", ENGINES)
def test_invariance_batch_shard_launch(D, engine):
    """Per-rotation results (rotation, t_lin and score bits) are bitwise independent of batch position, batch
    size, regions per batch (launch configuration), candidate cap and shard range.  The DOCK_POSE_FALLBACK
    flag only records which path produced a pose (the candidate lists or the exact fallback, whose score
    bits are the same), and that may depend on the launch configuration."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((64, 48, 40), P)
    w = g.weights(P)
    probes = g.probes(3, m, P)
    rot = g.rotations(19)
    ctx = _ctx(D, R, w, m, engine)
    ref = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    n = len(probes) * len(rot)
    def same(a, b):
        return all(np.array_equal(a[f].view(np.uint32) if f == "score" else a[f],
                                  b[f].view(np.uint32) if f == "score" else b[f]) for f in ("rot", "t_lin", "score"))

    for b, e in [(0, 5), (5, 31), (31, n), (7, 8)]:
        part = D.dock_probe_batch(ctx, probes, rot, unit_begin=b, unit_end=e, k=4, rho=1)
        assert same(part, ref[b:e])
    for G in (1, 3, 7):
        D.dock_set_tuning(ctx, D.DOCK_TUNE_REGIONS, G)
        assert same(D.dock_probe_batch(ctx, probes, rot, k=4, rho=1), ref)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_REGIONS, 0)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_CAND_CAP, 32)   # small cap: overflowing rotations take the fallback
    capped = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    assert np.array_equal(capped["t_lin"], ref["t_lin"])
    assert np.array_equal(capped["score"].view(np.uint32), ref["score"].view(np.uint32))
    D.dock_set_tuning(ctx, D.DOCK_TUNE_CAND_CAP, 1024)
    # reversed rotation order: per-rotation results follow the rotation
    rev = rot[::-1].copy()
    out = D.dock_probe_batch(ctx, probes, rev, k=4, rho=1)
    for pi in range(len(probes)):
        for i in range(len(rot)):
            a = out[pi * len(rot) + i]
            b = ref[pi * len(rot) + len(rot) - 1 - i]
            assert np.array_equal(a["t_lin"], b["t_lin"]) and np.array_equal(a["score"], b["score"])
    ctx.close()


def test_device_resident_io(D):
    """Device-resident inputs/outputs (torch CUDA tensors) give the same poses as host I/O."""
    import torch
    P, m = 4, 4
    R = g.receptor_ftmap_like((40, 32, 32), P)
    w = g.weights(P)
    probes = g.probes(2, m, P)
    rot = g.rotations(9)
    ctx = D.dock_init(torch.from_numpy(R).cuda(), torch.from_numpy(w).cuda(), H, m_max=m)
    host = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    dprobes = [{"xyz": torch.from_numpy(p.xyz).cuda(), "coef": torch.from_numpy(p.coef).cuda(), "m": p.m}
               for p in probes]
    out = torch.empty((len(probes) * len(rot), 4, 4), dtype=torch.int32, device="cuda")
    D.dock_probe_batch(ctx, dprobes, torch.from_numpy(rot).cuda(), k=4, rho=1, out=out)
    D.dock_sync(ctx)
    assert np.array_equal(D.poses_from_device(out), host)
    # a ProbeSet (descriptors marshalled once) over device or host arrays: the same poses, repeatedly
    for ps in (D.dock_probes(ctx, dprobes), D.dock_probes(ctx, probes)):
        for _ in range(2):
            out.fill_(-1)
            D.dock_probe_batch(ctx, ps, torch.from_numpy(rot).cuda(), k=4, rho=1, out=out)
            D.dock_sync(ctx)
            assert np.array_equal(D.poses_from_device(out), host)
    other = D.dock_init(torch.from_numpy(R[:2]).cuda(), torch.from_numpy(w[:2]).cuda(), H, m_max=m)
    with pytest.raises(ValueError):
        D.dock_probe_batch(other, D.dock_probes(ctx, dprobes), rot, k=4, rho=1)
    other.close()
    ctx.close()


@pytest.mark.parametrize("engine", ENGINES)
def test_async_device_output_and_fallback_loop(D, engine):
    """Device output is asynchronous: many calls are queued back to back without a host sync (the exact
    fallback runs as a device-driven CUDA-graph loop over chunks of flagged rotations).  Forcing every
    rotation of 150 units through that loop (several chunks: 128 per chunk on the tensor cores, 64 on
    FFMA) returns the same pose bits as the candidate path, and queued calls equal one-at-a-time calls."""
    import torch
    P, m = 4, 4
    R = g.receptor_ftmap_like((48, 40, 36), P)
    w = g.weights(P)
    probes = g.probes(3, m, P)
    rot = g.rotations(50)
    n = len(probes) * len(rot)
    ctx = _ctx(D, R, w, m, engine)
    ref = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    assert _engine_id(D.dock_get_info(ctx)) == engine
    dprobes = [{"xyz": torch.from_numpy(p.xyz).cuda(), "coef": torch.from_numpy(p.coef).cuda(), "m": p.m}
               for p in probes]
    drot = torch.from_numpy(rot).cuda()
    outs = [torch.full((n, 4, 4), -7, dtype=torch.int32, device="cuda") for _ in range(3)]
    D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 1)
    D.dock_probe_batch(ctx, dprobes, drot, k=4, rho=1, out=outs[0])   # returns before the GPU finishes
    D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 0)
    D.dock_probe_batch(ctx, dprobes, drot, k=4, rho=1, out=outs[1])
    D.dock_probe_batch(ctx, probes, rot, 10, n, k=4, rho=1, out=outs[2][10:])   # host inputs, async output
    D.dock_sync(ctx)
    forced, plain, part = (D.poses_from_device(o) for o in outs)
    assert (forced["flags"] & D.DOCK_POSE_FALLBACK).all()
    for got in (forced, plain):
        assert np.array_equal(got["t_lin"], ref["t_lin"])
        assert np.array_equal(got["score"].view(np.uint32), ref["score"].view(np.uint32))
    assert np.array_equal(part[10:]["t_lin"], ref[10:]["t_lin"])
    assert (outs[2][:10] == -7).all()
    info = D.dock_get_info(ctx)
    assert info["pending"] == 0
    ctx.close()


def test_async_errors_surface_at_sync(D):
    """A device-detected input error of an asynchronous call is reported by dock_sync (and is cleared)."""
    import torch
    P = 1
    R = g.receptor_uniform((16, 16, 16), P)
    ctx = D.dock_init(R, np.ones(P, np.float32), H, m_max=4)
    pr = g.probe(0, 4, P)
    out = torch.empty((1, 1, 4), dtype=torch.int32, device="cuda")
    D.dock_probe_batch(ctx, [pr], np.diag([1.0, 1.0, -1.0]).reshape(1, 9), k=1, rho=0, out=out)   # no raise
    with pytest.raises(D.DockError) as e:
        D.dock_sync(ctx)
    assert e.value.status == -4
    D.dock_sync(ctx)   # cleared
    far = g.Probe(np.array([[4.0, 0, 0]]), np.ones((1, 1), np.float32), 4)
    out3 = torch.empty((3, 1, 4), dtype=torch.int32, device="cuda")
    D.dock_probe_batch(ctx, [far], g.rotations(3), k=1, rho=0, out=out3)
    D.dock_probe_batch(ctx, [pr], g.rotations(3), k=1, rho=0, out=out3)   # a later good call does not hide it
    with pytest.raises(D.DockError) as e:
        D.dock_sync(ctx)
    assert e.value.status == -3
    ctx.close()


def test_sharded_one_rank_nccl(D):
    """The multi-GPU data plane under a 1-rank NCCL group: the docking call writes into this rank's slot of
    the preallocated all-gather buffer and one in-place NCCL all-gather returns the poses, bitwise equal to
    dock_probe_batch."""
    import os
    import socket
    import torch
    import torch.distributed as dist
    from paper_conf_ipps_sukhwanih10_b200 import parallel
    sock = socket.socket()
    sock.bind(("127.0.0.1", 0))
    port = sock.getsockname()[1]
    sock.close()
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("nccl", rank=0, world_size=1, device_id=torch.device("cuda", 0))
    try:
        P, m = 4, 4
        R = g.receptor_ftmap_like((40, 32, 32), P)
        probes = g.probes(2, m, P)
        rot = g.rotations(11)
        ctx = D.dock_init(R, g.weights(P), H, m_max=m, device=0)
        ref = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        for _ in range(2):   # the second call reuses the cached buffer
            full = parallel.dock_probe_sharded(ctx, probes, rot, k=4, rho=1)
            assert np.array_equal(D.poses_from_device(full), ref)
        ctx.close()
    finally:
        dist.destroy_process_group()


def test_errors(D):
    P = 1
    R = g.receptor_uniform((16, 16, 16), P)
    ctx = D.dock_init(R, np.ones(P, np.float32), H, m_max=4)
    pr = g.probe(0, 4, P)
    with pytest.raises(D.DockError) as e:
        D.dock_probe(ctx, pr, np.diag([1.0, 1.0, -1.0]).reshape(1, 9), k=1, rho=0)
    assert e.value.status == -4
    far = g.Probe(np.array([[4.0, 0, 0]]), np.ones((1, 1), np.float32), 4)
    with pytest.raises(D.DockError) as e:
        D.dock_probe(ctx, far, g.rotations(3), k=1, rho=0)
    assert e.value.status == -3
    with pytest.raises(D.DockError) as e:
        D.dock_probe(ctx, pr, g.rotations(3), k=0, rho=0)
    assert e.value.status == -1
    with pytest.raises(D.DockError) as e:
        D.dock_probe(ctx, pr, g.rotations(3), k=1, rho=8)
    assert e.value.status == -1
    with pytest.raises(D.DockError) as e:
        D.dock_probe(ctx, g.probe(0, 5, P), g.rotations(3), k=1, rho=0)
    assert e.value.status == -2
    # the context is still usable after argument errors
    D.dock_probe(ctx, pr, g.rotations(3), k=2, rho=1)
    ctx.close()
    with pytest.raises(D.DockError):
        D.dock_init(np.full((1, 8, 8, 8), np.nan, np.float32), np.ones(1, np.float32), H, m_max=2)


# ----------------------------------------------------------------------------- BASELINE configs


@pytest.mark.parametrize("engine", ENGINES)
def test_c64_config_sampled(D, orc, engine):
    """configs[1]: 64^3, 5^3 probe, 4 terms, 500 rotations, k=4 -- full GPU run, oracle on a sample."""
    c = g.CONFIGS["c64"]
    R = g.receptor_ftmap_like(c.n, c.P)
    w = g.weights(c.P)
    probes = g.probes(1, c.m, c.P)
    rot = g.rotations(c.n_rot)
    units = list(range(0, 500, 25)) + [1, 2, 3, 499]
    _dock_and_validate(D, orc, R, w, probes, rot, c.k, 1, units=units, engine=engine)


@pytest.mark.parametrize("engine", ENGINES)
def test_prod_config_sampled(D, orc, engine):
    """configs[2] (the bench workload, same launch as bench.py): 128^3, 16 probes x 500 rotations,
    k=4, rho=1 -- every unit docked on the GPU, a spread sample validated against the oracle."""
    c = g.CONFIGS["prod"]
    R = g.receptor_ftmap_like(c.n, c.P)
    w = g.weights(c.P)
    probes = g.probes(c.n_probes, c.m, c.P)
    rot = g.rotations(c.n_rot)
    units = [0, 1, 499, 500, 3777, 7999] + list(range(137, 8000, 811))
    _, info, _ = _dock_and_validate(D, orc, R, w, probes, rot, c.k, 1, units=units, engine=engine)
    assert info["fallback_last"] <= 80 and _engine_id(info) == engine


@pytest.mark.parametrize("engine", [1, 3, 4])
def test_large_config_sampled(D, orc, engine):
    """configs[4] shape: 160^3 receptor, 8^3 probe, 22 terms (pairwise-potential channels), k=4, rho=1.
    A 256-rotation slice of the 70k-rotation set is docked on the GPU (FFMA engine, and tcgen05 variant 2:
    six channel groups streamed per z-plane, 160 translations per MMA row); two units are validated
    against the oracle."""
    c = g.CONFIGS["large"]
    R = g.receptor_ftmap_like(c.n, c.P)
    w = g.weights(c.P)
    probes = g.probes(1, c.m, c.P)
    rot = g.rotations(256, seed=3001)
    _, info, _ = _dock_and_validate(D, orc, R, w, probes, rot, c.k, 1, units=[0, 173], engine=engine)
    assert info["fallback_last"] <= 4 and _engine_id(info) == engine


# ----------------------------------------------------------------------------- maximum / degenerate sizes


@pytest.mark.parametrize("engine", ENGINES)
@pytest.mark.parametrize("rho", [0, 1])
def test_max_terms_probe_and_k(D, orc, engine, rho):
    """DOCK_MAX_TERMS = 32 channels (8 tcgen05 channel groups), the largest probe grid m = 8 and
    DOCK_MAX_K = 32 poses per rotation, on a ragged grid; poses validated tie-aware, score grids
    within 1e-4 * A."""
    P, m, k = D.DOCK_MAX_TERMS, D.DOCK_MAX_M, D.DOCK_MAX_K
    R = g.receptor("uniform", (48, 20, 17), P)
    w = g.weights(P)
    probes = g.probes(1, m, P)
    rot = g.rotations(5, with_cube_group=False)
    poses, info, _ = _dock_and_validate(D, orc, R, w, probes, rot, k, rho, engine=engine)
    assert _engine_id(info) == {1: 1, 4: 4}.get(engine, 3)   # 8 channel groups: tcgen05 variant 2
    ctx = _ctx(D, R, w, m, engine)
    S_g = D.dock_score_grid(ctx, probes[0], rot[1])
    ctx.close()
    S_o, A_o = _oracle_SA(orc, R, w, probes[0], rot[1])
    assert (np.abs(S_g.astype(np.float64) - S_o) <= 1e-4 * A_o + 1e-12).all()


def test_empty_unit_range(D):
    """An empty shard (unit_begin == unit_end) is a no-op, not an error."""
    P, m = 4, 4
    R = g.receptor_ftmap_like((32, 32, 32), P)
    ctx = D.dock_init(R, g.weights(P), H, m_max=m)
    out = D.dock_probe_batch(ctx, g.probes(1, m, P), g.rotations(4), unit_begin=2, unit_end=2, k=4, rho=1)
    assert len(out) == 0
    ctx.close()


def test_sparse_engine_edge_cases(D, orc):
    """Sparse-ligand engine limits: a probe without atoms scores 0 everywhere (exact ties -> the greedy picks
    t_lin 0, 2, 4, 6 at rho = 1, tests/golden/filter_constant_grid.txt's reading); a 20-atom probe (about the
    most whose plane ring fits shared memory at m = 4 on 64-translation rows; many multi-atom voxels -> direct
    terms) matches the oracle; 33 atoms (> sp::TMAX) is refused when forced and routed to a dense engine by
    auto."""
    P, m = 3, 4
    R = g.receptor_ftmap_like((40, 24, 20), P)
    w = g.weights(P)
    rot = g.rotations(5)
    ctx = _ctx(D, R, w, m, 4)
    empty = g.Probe(np.zeros((0, 3)), np.zeros((0, P), np.float32), m)
    poses = D.dock_probe_batch(ctx, [empty], rot, k=4, rho=1)
    assert (poses["score"] == 0).all() and (poses["t_lin"] == np.array([0, 2, 4, 6])).all()
    rng = np.random.default_rng(32)
    xyz = rng.normal(size=(20, 3))
    xyz *= (1.5 * rng.random(20) ** (1 / 3) / np.linalg.norm(xyz, axis=1))[:, None]   # inside the box under rotation
    big = g.Probe(xyz, rng.normal(size=(20, P)).astype(np.float32), m)
    poses = D.dock_probe_batch(ctx, [big], rot, k=4, rho=1)
    assert D.dock_get_info(ctx)["engine_last"] == 4
    for r in range(len(rot)):
        L = orc.voxelize(big.xyz, big.coef, m, rot[r], H)
        S, A = orc.score_grid(R, L, w)
        validate_unit(S, A, poses[r]["t_lin"], poses[r]["score"], 4, 1)
    S_g = D.dock_score_grid(ctx, big, rot[2])
    S_o, A_o = _oracle_SA(orc, R, w, big, rot[2])
    assert (np.abs(S_g.astype(np.float64) - S_o) <= 1e-4 * A_o + 1e-12).all()
    huge = g.Probe(np.zeros((33, 3)), np.ones((33, P), np.float32), m)
    with pytest.raises(D.DockError) as e:
        D.dock_probe_batch(ctx, [huge], rot, k=4, rho=1)
    assert e.value.status == -2
    D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, 0)
    D.dock_probe_batch(ctx, [huge], rot, k=4, rho=1)
    assert D.dock_get_info(ctx)["engine_last"] in (1, 2)
    ctx.close()
