"""Pins of the FP64 energy-minimisation oracle (oracle/em_oracle.c, Eqs. 4-10 with
readings E1-E6 of DESIGN.md §13) against what the mathematics fixes -- no GPU.

  * forces are the negative gradient of the energy (central finite differences): pins every derivative
    and the chain rule through the Born radii;
  * Newton's third law (all terms are pairwise): the forces sum to zero;
  * rigid-motion invariance of the energy, rotation covariance of the forces, label permutation;
  * closed forms of limiting cases: the Lennard-Jones minimum -eps at rm (Eq. 8 with rc -> inf), the
    shifted form's E(rc) = E'(rc) = 0 (Eq. 8 cut-off), the isolated ion's self energy q^2 / (2 eps_s R)
    (Eq. 5), the Gaussian term at r = sigma (Eq. 6), and the GB pair energy tending to Coulomb's law in the
    solvent 332 q q / (eps_s r) when the Born radii vanish (Eq. 7).
"""
import dataclasses

import numpy as np
import pytest

import dockgen as g


@pytest.fixture(scope="module")
def em():
    import oracle
    oracle.build_em_oracle()
    return oracle


def _small(seed=7, n=24, rc=9.0):
    return g.em_system(n, seed=seed, rc=rc)


def _total(em, s, x):
    e, _ = em.em_eval(s, x, forces=False)
    return float(e.sum())


def test_forces_are_minus_gradient(em):
    s = _small()
    x = g.em_conformations(s, 1, seed=3)[0]
    e, f = em.em_eval(s, x)
    h = 1e-6
    rng = np.random.default_rng(1)
    for a in rng.choice(len(x), 8, replace=False):
        for d in range(3):
            xp, xm = x.copy(), x.copy()
            xp[a, d] += h
            xm[a, d] -= h
            fd = -(_total(em, s, xp) - _total(em, s, xm)) / (2 * h)
            assert abs(fd - f[a, d]) <= 1e-6 * max(1.0, abs(f[a, d])), (a, d, fd, f[a, d])


def test_newton_third_law(em):
    s = g.em_system(150, seed=11)
    _, f = em.em_eval(s, g.em_conformations(s, 3, seed=4))
    assert np.abs(f.sum(axis=1)).max() <= 1e-9 * np.abs(f).sum(axis=1).max()


def test_rigid_motion_and_permutation(em):
    s = g.em_system(120, seed=12)
    x = g.em_conformations(s, 1, seed=5)[0]
    e0, f0 = em.em_eval(s, x)
    q = g.rotations(2, seed=9)[1].reshape(3, 3)
    e1, f1 = em.em_eval(s, x @ q.T + np.array([3.0, -7.5, 11.0]))
    assert np.allclose(e1, e0, rtol=1e-12, atol=1e-9)
    assert np.allclose(f1, f0 @ q.T, rtol=1e-9, atol=1e-9)
    # relabel the atoms (and the pair list accordingly): same energies, permuted forces
    perm = np.random.default_rng(2).permutation(len(x))
    inv = np.argsort(perm)
    p2 = inv[s.pairs]
    p2 = np.sort(p2, axis=1)
    p2 = p2[np.lexsort((p2[:, 1], p2[:, 0]))].astype(np.int32)
    sp = dataclasses.replace(s, x0=s.x0[perm], q=s.q[perm], R=s.R[perm], V=s.V[perm], eps=s.eps[perm], rm=s.rm[perm],
                             type=s.type[perm], pairs=p2)
    e2, f2 = em.em_eval(sp, x[perm])
    assert np.allclose(e2, e0, rtol=1e-12, atol=1e-9)
    assert np.allclose(f2, f0[perm], rtol=1e-9, atol=1e-9)


def _two(q=(0.0, 0.0), rc=9.0, R=(1.5, 1.5), V=(0.0, 0.0), omega=0.0):
    s = g.em_system(2, seed=1, rc=rc)
    return dataclasses.replace(s, q=np.array(q, float), R=np.array(R, float), V=np.array(V, float),
                               eps=np.array([0.1, 0.4]), rm=np.array([1.8, 2.2]), type=np.zeros(2, np.int32),
                               omega=np.full((1, 1), omega), sigma=np.full((1, 1), 3.0), mu=np.full((1, 1), 2.0),
                               pairs=np.array([[0, 1]], np.int32))


def test_vdw_closed_forms(em):
    eps, rm = np.sqrt(0.1 * 0.4), 2.0     # Eq. 9, Eq. 10
    far = _two(rc=1e3)
    e, f = em.em_eval(far, np.array([[0.0, 0, 0], [rm, 0, 0]]))
    assert abs(e[2] + eps) <= 1e-9 and abs(f[0, 0]) <= 1e-9          # LJ minimum -eps at rm, zero force
    near = _two(rc=6.0)
    for r in (5.999999, 6.0, 6.5):
        e, f = em.em_eval(near, np.array([[0.0, 0, 0], [r, 0, 0]]))
        assert abs(e[2]) <= 1e-9 and abs(f[0, 0]) <= 1e-6             # shifted: E(rc) = E'(rc) = 0, 0 beyond
    assert e[0] == 0.0 and e[1] == 0.0                                  # neutral atoms: no electrostatics


def test_self_energy_closed_forms(em):
    eps_s = 80.0
    tau = 1.0 - 1.0 / eps_s
    s = _two(q=(0.3, -0.2), rc=1.0)
    s = dataclasses.replace(s, pairs=np.zeros((0, 2), np.int32))      # isolated ions
    e, _ = em.em_eval(s, np.array([[0.0, 0, 0], [50.0, 0, 0]]))
    want = 332.0 * sum(qi * qi / (2 * eps_s * Ri) for qi, Ri in zip((0.3, -0.2), (1.5, 1.5)))
    assert abs(e[0] - want) <= 1e-12 * want
    # Gaussian term of Eq. 6 alone (V = 0) at r = sigma: s_ik = tau * omega / e
    s = _two(q=(0.3, 0.0), omega=0.01)
    e, _ = em.em_eval(s, np.array([[0.0, 0, 0], [3.0, 0, 0]]))
    want = 332.0 * 0.09 * (1 / (2 * eps_s * 1.5) + tau * 0.01 / np.e)
    assert abs(e[0] - want) <= 1e-12 * want


def test_gb_tends_to_screened_coulomb(em):
    eps_s = 80.0
    s = _two(q=(0.4, -0.3), R=(1e-9, 1e-9))                            # alpha = tau eps_s R -> 0
    r = 5.0
    e, _ = em.em_eval(s, np.array([[0.0, 0, 0], [r, 0, 0]]))
    want = 332.0 * 0.4 * -0.3 / (eps_s * r)                             # 332 qq/r (1 - tau) = 332 qq/(eps_s r)
    assert abs(e[1] - want) <= 1e-9 * abs(want)
