"""Pins of the FP64 oracle against what the paper and the mathematics fix (no GPU).

Each test names the pin and the passage it follows.  None of
them re-types the oracle's own loop: they use an independent formulation (Eq. 1's
literal receptor-outer form, FFT, a library convolution), closed forms, invariants,
special cases, or hand-derived fixtures under tests/golden/.
"""
import itertools
import math
import os

import numpy as np
import pytest

import dockgen as g

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")
H = g.SPACING


def _rand_L(rng, P, m, density=0.5):
    L = rng.normal(size=(P, m, m, m))
    L[rng.random(L.shape) > density] = 0.0
    return L


# ----------------------------------------------------------------------------- P1


def _eq1_literal(R, L, w):
    """Eq. 1 written receptor-outer with the ligand as a full N^3 grid.

    E(alpha) = sum_p w_p sum_{i} R_p(i) Lfull_p(i + alpha), Lfull = L zero-padded to N^3,
    indices cyclic.  Reading Q1: the score of translation t is E(alpha = -t mod N).
    Pure-Python loops; tiny grids only.
    """
    P, nz, ny, nx = R.shape
    m = L.shape[-1]
    Lf = np.zeros((P, nz, ny, nx))
    Lf[:, :m, :m, :m] = L
    S = np.zeros((nz, ny, nx))
    for az in range(nz):
        for ay in range(ny):
            for ax in range(nx):
                e = 0.0
                for p in range(P):
                    for i in range(nz):
                        for j in range(ny):
                            for l in range(nx):
                                e += w[p] * R[p, i, j, l] * Lf[p, (i + az) % nz, (j + ay) % ny, (l + ax) % nx]
                S[(-az) % nz, (-ay) % ny, (-ax) % nx] = e
    return S


def test_P1_brute_force_eq1_literal(orc):
    rng = np.random.default_rng(11)
    for (nx, ny, nz), m, P in [((4, 4, 4), 2, 1), ((5, 4, 3), 3, 2), ((6, 5, 4), 2, 3)]:
        R = rng.normal(size=(P, nz, ny, nx)).astype(np.float32)
        L = _rand_L(rng, P, m, 0.7)
        w = rng.normal(size=P).astype(np.float32)
        S, A = orc.score_grid(R, L, w)
        ref = _eq1_literal(R.astype(np.float64), L, w.astype(np.float64))
        assert np.max(np.abs(S - ref)) <= 1e-12 * max(1.0, np.max(A))


# ----------------------------------------------------------------------------- P2


def _fft_score(R, L, w):
    """Independent FFT correlation (direct == FFT per P:L504-505)."""
    P, nz, ny, nx = R.shape
    m = L.shape[-1]
    S = np.zeros((nz, ny, nx))
    for p in range(P):
        Lp = np.zeros((nz, ny, nx))
        Lp[:m, :m, :m] = L[p]
        S += float(w[p]) * np.real(np.fft.ifftn(np.fft.fftn(R[p].astype(np.float64)) * np.conj(np.fft.fftn(Lp))))
    return S


@pytest.mark.parametrize("shape,m,P", [((16, 16, 16), 4, 4), ((12, 10, 9), 3, 2), ((20, 16, 12), 5, 3),
                                       ((9, 9, 9), 8, 1)])
def test_P2_fft_agreement(orc, shape, m, P):
    rng = np.random.default_rng(22)
    nx, ny, nz = shape
    R = g.receptor_uniform(shape, P, seed=5)
    L = _rand_L(rng, P, m, 0.4)
    w = g.weights(P)
    S, A = orc.score_grid(R, L, w)
    assert np.max(np.abs(S - _fft_score(R, L, w))) <= 1e-9 * max(1.0, A.max())


# ----------------------------------------------------------------------------- P3


def test_P3_conv3d_library(orc):
    torch = pytest.importorskip("torch")
    import torch.nn.functional as F
    rng = np.random.default_rng(33)
    for shape, m, P in [((16, 16, 16), 4, 4), ((11, 13, 7), 5, 2)]:
        nx, ny, nz = shape
        R = g.receptor_uniform(shape, P, seed=6)
        L = _rand_L(rng, P, m, 0.5)
        w = g.weights(P)
        S, A = orc.score_grid(R, L, w)
        x = torch.from_numpy(R.astype(np.float64))[None]                      # [1][P][nz][ny][nx]
        x = F.pad(x, (0, m - 1, 0, m - 1, 0, m - 1), mode="circular")
        k = torch.from_numpy(L * w.astype(np.float64)[:, None, None, None])[None]  # [1][P][m][m][m]
        ref = F.conv3d(x, k)[0, 0].numpy()                                  # cross-correlation
        assert np.max(np.abs(S - ref)) <= 1e-9 * max(1.0, A.max())


# ----------------------------------------------------------------------------- P13 (the tolerance scale A)


def test_P13_magnitude_sum_conv3d_library(orc):
    """A[t] = sum_p sum_v |w_p L_p[v] R_p[(t+v) mod n]| (reading Q16) -- the scale of every GPU
    tolerance -- equals a library convolution of |R| (circular padding) with |w_p L_p|."""
    torch = pytest.importorskip("torch")
    import torch.nn.functional as F
    rng = np.random.default_rng(131)
    for shape, m, P in [((12, 10, 9), 4, 4), ((9, 11, 7), 3, 2), ((8, 8, 8), 5, 3)]:
        R = g.receptor_uniform(shape, P, seed=13)
        L = _rand_L(rng, P, m, 0.5)
        w = np.array([1.0, -0.6, 2.5, 0.4][:P], np.float32)   # signs and |w| != 1: a dropped |w_p| fails
        S, A = orc.score_grid(R, L, w)
        x = torch.from_numpy(np.abs(R.astype(np.float64)))[None]
        x = F.pad(x, (0, m - 1, 0, m - 1, 0, m - 1), mode="circular")
        k = torch.from_numpy(np.abs(L * w.astype(np.float64)[:, None, None, None]))[None]
        ref = F.conv3d(x, k)[0, 0].numpy()
        assert np.max(np.abs(A - ref)) <= 1e-12 * A.max()
        assert (A >= np.abs(S) - 1e-12 * A.max()).all()          # triangle inequality


def test_P13_magnitude_sum_single_atom_exact(orc):
    """One atom with coefficients c on voxel v0: A = sum_p |w_p c_p| roll(|R_p|, -v0), bitwise for P = 1;
    and for same-sign terms A == |S| (no cancellation)."""
    R = g.receptor_uniform((9, 8, 7), 2, seed=14)
    for m, v0 in [(3, (2, 0, 1)), (4, (1, 3, 2))]:
        pr = g.voxel_centre_probe([v0], m, 1, coef=np.array([[-1.75]], np.float32))
        L = orc.voxelize(pr.xyz, pr.coef, m, np.eye(3).reshape(9), H)
        w = np.array([0.6], np.float32)
        _, A = orc.score_grid(R[:1], L, w)
        want = (abs(np.float64(w[0])) * 1.75) * np.abs(R[0].astype(np.float64))
        assert np.array_equal(A, np.roll(want, (-v0[2], -v0[1], -v0[0]), axis=(0, 1, 2)))
    Rp = np.abs(R)
    L = np.abs(_rand_L(np.random.default_rng(5), 2, 3, 0.6))
    S, A = orc.score_grid(Rp, L, np.array([0.5, 2.0], np.float32))
    assert np.max(np.abs(A - S)) <= 1e-12 * A.max()


def test_P13_dock_reports_A_at_picks(orc):
    """orc_dock's per-pick A is the score grid's A at the picked cells."""
    R = g.receptor_uniform((10, 9, 8), 3, seed=15)
    w = g.weights(3)
    pr = g.probe(1, 3, 3)
    rot = g.rotations(3)
    t, s, st, a = orc.dock(R, w, H, [pr], rot, 4, 1, with_A=True)
    assert (st == 0).all()
    for r in range(3):
        S, A = orc.score_grid(R, orc.voxelize(pr.xyz, pr.coef, 3, rot[r], H), w)
        assert np.array_equal(a[r], A.reshape(-1)[t[r]])
        assert np.array_equal(s[r], S.reshape(-1)[t[r]])


# ----------------------------------------------------------------------------- P4/P5


def test_P4_delta_probe_identity(orc):
    """One atom at the rotation centre, m = 1, coef = e_p, w_p = 1 -> S == R_p bitwise."""
    R = g.receptor_uniform((7, 6, 5), 3, seed=7)
    for p in range(3):
        coef = np.zeros((1, 3), np.float32)
        coef[0, p] = 1.0
        L = orc.voxelize(np.zeros((1, 3)), coef, 1, np.eye(3).reshape(9), H)
        S, _ = orc.score_grid(R, L, np.ones(3, np.float32))
        assert np.array_equal(S, R[p].astype(np.float64))


@pytest.mark.parametrize("m", [2, 3, 4, 5])
def test_P5_shift_equivariance(orc, m):
    """Single atom on voxel v0 -> S = roll(R, -v0) exactly; moving it by +h in x shifts S by one voxel."""
    R = g.receptor_uniform((9, 8, 7), 1, seed=8)
    rng = np.random.default_rng(m)
    for _ in range(4):
        v0 = tuple(int(a) for a in rng.integers(0, m, size=3))
        pr = g.voxel_centre_probe([v0], m, 1)
        L = orc.voxelize(pr.xyz, pr.coef, m, np.eye(3).reshape(9), H)
        S, _ = orc.score_grid(R, L, np.ones(1, np.float32))
        ref = np.roll(R[0].astype(np.float64), shift=(-v0[2], -v0[1], -v0[0]), axis=(0, 1, 2))
        assert np.array_equal(S, ref)
    if m >= 2:
        pr = g.voxel_centre_probe([(0, 0, 0)], m, 1)
        L0 = orc.voxelize(pr.xyz, pr.coef, m, np.eye(3).reshape(9), H)
        L1 = orc.voxelize(pr.xyz + np.array([[H, 0, 0]]), pr.coef, m, np.eye(3).reshape(9), H)
        S0, _ = orc.score_grid(R, L0, np.ones(1, np.float32))
        S1, _ = orc.score_grid(R, L1, np.ones(1, np.float32))
        assert np.array_equal(S1, np.roll(S0, -1, axis=2))


# ----------------------------------------------------------------------------- P6/P7


def test_P6_checksum(orc):
    """Cyclic identity: sum_t S = sum_p w_p (sum_v L_p)(sum_t R_p)."""
    rng = np.random.default_rng(66)
    R = g.receptor_uniform((10, 9, 8), 4, seed=9)
    L = _rand_L(rng, 4, 4, 0.5)
    w = g.weights(4)
    S, A = orc.score_grid(R, L, w)
    ref = sum(float(w[p]) * L[p].sum() * R[p].astype(np.float64).sum() for p in range(4))
    assert abs(S.sum() - ref) <= 1e-10 * max(1.0, A.sum())


def test_P7_linearity_in_weights(orc):
    rng = np.random.default_rng(77)
    R = g.receptor_uniform((8, 8, 8), 4, seed=10)
    L = _rand_L(rng, 4, 3, 0.6)
    w1 = rng.normal(size=4).astype(np.float32)
    w2 = rng.normal(size=4).astype(np.float32)
    S1, A1 = orc.score_grid(R, L, w1)
    S2, A2 = orc.score_grid(R, L, w2)
    S12, _ = orc.score_grid(R, L, (w1.astype(np.float64) + w2).astype(np.float32))
    tol = 1e-12 * (A1.max() + A2.max())
    w12 = w1.astype(np.float64) + w2
    # S is linear in w: S(w1 + w2) = S(w1) + S(w2) up to the fp32 rounding of w1 + w2
    assert np.allclose(S12, S1 + S2, atol=1e-6 * (A1.max() + A2.max()))
    # per-term decomposition S = sum_p w_p C_p, with C_p from e_p weights
    C = [orc.score_grid(R, L, np.eye(4, dtype=np.float32)[p])[0] for p in range(4)]
    assert np.max(np.abs(S1 - sum(float(w1[p]) * C[p] for p in range(4)))) <= tol
    # argmin(-w) = argmax(w) (reading Q7)
    Sn, _ = orc.score_grid(R, L, -w1)
    assert np.array_equal(Sn, -S1)
    assert int(np.argmin(Sn)) == int(np.argmax(S1))
    del w12


# ----------------------------------------------------------------------------- voxelize / P8


def test_voxelize_golden_cases(orc):
    for line in open(os.path.join(GOLDEN, "voxelize_cases.txt")):
        if line.startswith("#") or not line.strip():
            continue
        m, x, v = line.split()
        m, x, v = int(m), float(x), int(v)
        for axis in range(3):
            xyz = np.zeros((1, 3))
            xyz[0, axis] = x
            if v < 0:
                with pytest.raises(orc.OracleError):
                    orc.voxelize(xyz, np.ones((1, 1), np.float32), m, np.eye(3).reshape(9), H)
                continue
            L = orc.voxelize(xyz, np.ones((1, 1), np.float32), m, np.eye(3).reshape(9), H)
            c = int(math.floor((m - 1) / 2.0 + 0.5))   # the other two axes sit at x = 0
            want = [c, c, c]
            want[axis] = v
            idx = np.argwhere(L[0] != 0)
            assert idx.tolist() == [[want[2], want[1], want[0]]]


def test_voxelize_sums_coincident_atoms(orc):
    xyz = np.array([[0.1, 0.0, 0.0], [-0.1, 0.05, 0.0], [0.8, 0.0, 0.0]])
    coef = np.array([[1.5, -2.0], [0.25, 3.0], [1.0, 1.0]], np.float32)
    L = orc.voxelize(xyz, coef, 3, np.eye(3).reshape(9), H)
    assert L[0, 1, 1, 1] == 1.75 and L[1, 1, 1, 1] == 1.0
    assert L[0, 1, 1, 2] == 1.0 and L[1, 1, 1, 2] == 1.0
    assert np.count_nonzero(L) == 4


def test_voxelize_quarter_turn(orc):
    """90 deg about z maps (x, y) -> (-y, x): an atom at +h x lands one voxel up in y."""
    Rz = np.array([[0, -1, 0], [1, 0, 0], [0, 0, 1]], dtype=np.float64)
    L = orc.voxelize(np.array([[H, 0.0, 0.0]]), np.ones((1, 1), np.float32), 3, Rz.reshape(9), H)
    assert np.argwhere(L[0] != 0).tolist() == [[1, 2, 1]]   # [z][y][x]


@pytest.mark.parametrize("m", [3, 4, 5, 8])
def test_P8_cube_group_permutes_voxels(orc, m):
    """Atoms on voxel centres: each of the 24 cube rotations permutes voxels exactly."""
    rng = np.random.default_rng(m)
    cells = set()
    while len(cells) < min(6, m ** 3):
        cells.add(tuple(int(a) for a in rng.integers(0, m, 3)))
    cells = sorted(cells)
    coef = rng.normal(size=(len(cells), 2)).astype(np.float32)
    pr = g.voxel_centre_probe(cells, m, 2, coef=coef)
    c = (m - 1) / 2.0
    for q in g.cube_group():
        Q = q.reshape(3, 3)
        L = orc.voxelize(pr.xyz, pr.coef, m, q, H)
        want = np.zeros_like(L)
        for (vx, vy, vz), cf in zip(cells, coef):
            d = Q @ np.array([vx - c, vy - c, vz - c])
            wx, wy, wz = (int(round(a + c)) for a in d)
            want[:, wz, wy, wx] += cf
        assert np.array_equal(L, want)


def test_P8_identity_and_quaternion_sign(orc):
    q = g.shoemake_quaternions(16, 3)
    assert np.allclose(g.quat_to_matrix(q), g.quat_to_matrix(-q), atol=0, rtol=0)
    pr = g.probe(3, 4, 2)
    L = orc.voxelize(pr.xyz, pr.coef, 4, g.rotations(1)[0], H)
    v = np.floor(pr.xyz / H + 1.5 + 0.5).astype(int)
    want = np.zeros_like(L)
    for (vx, vy, vz), cf in zip(v, pr.coef):
        want[:, vz, vy, vx] += cf
    assert np.allclose(L, want, atol=1e-6)


def test_rotation_checks(orc):
    assert orc.check_rotation(np.eye(3)) == 0
    for q in g.rotations(50):
        assert orc.check_rotation(q) == 0
    assert orc.check_rotation(np.diag([1.0, 1.0, -1.0])) == -4          # reflection
    assert orc.check_rotation(np.eye(3) * 1.001) == -4                  # not orthogonal
    with pytest.raises(orc.OracleError):
        orc.voxelize(np.array([[5.0, 0, 0]]), np.ones((1, 1), np.float32), 4, np.eye(3).reshape(9), H)


# ----------------------------------------------------------------------------- P10 filter


def _greedy_sorted(S, k, rho):
    """Independent formulation: sort all cells once by (score, t_lin), scan, keep a cell
    if it is not within the cyclic Chebyshev ball of an already kept cell."""
    nz, ny, nx = S.shape
    order = sorted(range(S.size), key=lambda t: (S.reshape(-1)[t], t))
    kept = []
    for t in order:
        x, y, z = t % nx, (t // nx) % ny, t // (nx * ny)
        ok = True
        for u in kept:
            ux, uy, uz = u % nx, (u // nx) % ny, u // (nx * ny)
            d = max(min(abs(x - ux), nx - abs(x - ux)), min(abs(y - uy), ny - abs(y - uy)),
                    min(abs(z - uz), nz - abs(z - uz)))
            if d <= rho:
                ok = False
                break
        if ok:
            kept.append(t)
            if len(kept) == k:
                break
    return kept


def test_P10_filter_golden_constant_grid(orc):
    S = np.zeros((8, 8, 8))
    for line in open(os.path.join(GOLDEN, "filter_constant_grid.txt")):
        if line.startswith("#") or not line.strip():
            continue
        vals = [int(a) for a in line.split()]
        rho, k, picks = vals[0], vals[1], vals[2:]
        t, s = orc.filter_greedy(S, k, rho)
        assert t.tolist() == picks
        assert _greedy_sorted(S, k, rho) == picks


def test_P10_filter_negative_zero_tie(orc):
    S = np.ones((4, 4, 4))
    S[0, 0, 3] = 0.0
    S[0, 0, 1] = -0.0
    t, s = orc.filter_greedy(S, 1, 0)
    assert t.tolist() == [1]                     # -0.0 == +0.0, smaller t_lin wins


@pytest.mark.parametrize("rho", [0, 1, 2])
def test_P10_filter_random_vs_sorted_scan(orc, rho):
    rng = np.random.default_rng(100 + rho)
    for trial in range(6):
        shape = tuple(int(a) for a in rng.integers(5, 9, 3))
        S = rng.integers(-3, 4, size=shape[::-1]).astype(np.float64)   # many ties
        k = int(rng.integers(1, 6))
        t, _ = orc.filter_greedy(S, k, rho)
        assert t.tolist() == _greedy_sorted(S, k, rho)
        if rho == 0:   # plain top-k by (score, t_lin)
            order = np.lexsort((np.arange(S.size), S.reshape(-1)))[:k]
            assert t.tolist() == order.tolist()


# ----------------------------------------------------------------------------- dock composition


def test_dock_composition_and_independence(orc):
    R = g.receptor_ftmap_like((16, 16, 16), 4)
    w = g.weights(4)
    prs = g.probes(3, 4, 4)
    rot = g.rotations(6, with_cube_group=False)
    t, s, st = orc.dock(R, w, H, prs, rot, k=4, rho=1)
    assert (st == 0).all()
    for u in range(len(prs) * len(rot)):
        pr, r = prs[u // len(rot)], u % len(rot)
        L = orc.voxelize(pr.xyz, pr.coef, pr.m, rot[r], H)
        S = orc.score_grid(R, L, w, with_A=False)
        tt, ss = orc.filter_greedy(S, 4, 1)
        assert t[u].tolist() == tt.tolist() and np.array_equal(s[u], ss)
    # per-rotation results independent of the set order and of the shard range
    perm = np.arange(len(rot))[::-1].copy()
    t2, s2, _ = orc.dock(R, w, H, prs, rot[perm], k=4, rho=1)
    for pi in range(len(prs)):
        for i, r in enumerate(perm):
            assert t2[pi * len(rot) + i].tolist() == t[pi * len(rot) + r].tolist()
    t3, s3, _ = orc.dock(R, w, H, prs, rot, k=4, rho=1, unit_begin=5, unit_end=13)
    assert np.array_equal(t3, t[5:13]) and np.array_equal(s3, s[5:13])


def test_dock_status_codes(orc):
    R = g.receptor_uniform((8, 8, 8), 1)
    w = np.ones(1, np.float32)
    bad = g.Probe(xyz=np.array([[3.0, 0, 0]]), coef=np.ones((1, 1), np.float32), m=4)
    good = g.probe(0, 4, 1)
    rot = np.stack([np.eye(3).reshape(9), np.diag([1.0, 1.0, -1.0]).reshape(9)])
    t, s, st = orc.dock(R, w, H, [good, bad], rot, k=2, rho=0)
    assert st.tolist() == [0, -4, -3, -4]
    assert (t[1] == -1).all() and np.isnan(s[1]).all()


# ----------------------------------------------------------------------------- P9 / P12


def test_P9_integer_inputs_exact(orc):
    """Integer receptor, integer coefficients, weights in {1, 2, 1/2}: every partial sum is
    exactly representable, so S is exactly the integer-arithmetic correlation."""
    P, m = 3, 3
    R = g.receptor_integer((6, 5, 7), P)
    pr = g.probe(2, m, P, integer=True)
    w = g.weights_integer(P)
    L = orc.voxelize(pr.xyz, pr.coef, m, np.eye(3).reshape(9), H)
    S, _ = orc.score_grid(R, L, w)
    # exact rational reference: scale by 2 (w has halves) and use python ints
    Li = np.rint(L).astype(np.int64)
    assert np.array_equal(Li, L)
    Ri = R.astype(np.int64)
    w2 = np.rint(2 * w).astype(np.int64)
    ref = np.zeros(S.shape, dtype=np.int64)
    for p, vz, vy, vx in itertools.product(range(P), range(m), range(m), range(m)):
        if Li[p, vz, vy, vx]:
            ref += w2[p] * Li[p, vz, vy, vx] * np.roll(Ri[p], (-vz, -vy, -vx), axis=(0, 1, 2))
    assert np.array_equal(S * 2, ref.astype(np.float64))


def test_P12_fp32_tolerance_realism(orc):
    """An fp32 evaluation of the same sum stays far inside the 1e-4*A tolerance (Q16)."""
    R = g.receptor_ftmap_like((24, 24, 24), 4)
    pr = g.probe(6, 4, 4)
    w = g.weights(4)
    q = g.rotations(3)[2]
    L = orc.voxelize(pr.xyz, pr.coef, 4, q, H)
    S, A = orc.score_grid(R, L, w)
    Lw = (L.astype(np.float32) * w[:, None, None, None]).astype(np.float32)
    S32 = np.zeros(S.shape, np.float32)
    for p, vz, vy, vx in itertools.product(range(4), range(4), range(4), range(4)):
        S32 += Lw[p, vz, vy, vx] * np.roll(R[p], (-vz, -vy, -vx), axis=(0, 1, 2))
    err = np.abs(S32 - S) / np.maximum(A, 1e-30)
    assert err[A > 0].max() < 1e-5
