"""GPU parity of the energy-minimisation non-bonded kernels (NEXT-4; include/dock_em.h) against the FP64
oracle (oracle/em_oracle.c), through the C ABI.  Both sides compute in FP64; the GPU sums in a different
(fixed) order, so energies agree to ~1e-12 relative and forces to ~1e-10 of the largest force."""
import dataclasses

import numpy as np
import pytest

import dockgen as g

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def D():
    import torch
    assert torch.cuda.is_available(), "GPU tests need a CUDA device"
    from paper_conf_ipps_sukhwanih10_b200 import build
    build.build_native()
    import paper_conf_ipps_sukhwanih10_b200 as D
    return D


@pytest.fixture(scope="module")
def em():
    import oracle
    oracle.build_em_oracle()
    return oracle


def _close(eg, fg, eo, fo):
    assert np.all(np.abs(eg - eo) <= 1e-10 * (np.abs(eo) + 1.0)), (eg, eo)
    if fo is not None:
        assert np.abs(fg - fo).max() <= 1e-9 * max(1.0, np.abs(fo).max())


@pytest.mark.parametrize("n_atoms,n_conf,seed", [(1, 1, 1), (2, 3, 2), (37, 5, 3), (300, 6, 4)])
def test_em_matches_oracle(D, em, n_atoms, n_conf, seed):
    s = g.em_system(n_atoms, seed=seed)
    x = g.em_conformations(s, n_conf, seed=seed + 10)
    ctx = D.em.em_init(s)
    eg, fg = D.em.em_eval(ctx, x)
    eo, fo = em.em_eval(s, x)
    _close(eg, fg, eo, fo)
    e2, f2 = D.em.em_eval(ctx, x, forces=False)
    assert np.array_equal(e2, eg) and f2 is None
    ctx.close()


def test_em_full_size_sampled(D, em):
    """A protein-sized system (2200 atoms, ~170k pairs within the 9 A cut-off): 64 conformations
    on the GPU, two of them checked against the oracle."""
    s = g.em_system(2200, seed=5001)
    x = g.em_conformations(s, 64)
    ctx = D.em.em_init(s)
    eg, fg = D.em.em_eval(ctx, x)
    for c in (0, 63):
        eo, fo = em.em_eval(s, x[c])
        _close(eg[c], fg[c], eo, fo)
    ctx.close()


def test_em_deterministic_and_batch_invariant(D):
    s = g.em_system(400, seed=8)
    x = g.em_conformations(s, 7, seed=9)
    ctx = D.em.em_init(s)
    e1, f1 = D.em.em_eval(ctx, x)
    e2, f2 = D.em.em_eval(ctx, x)
    assert np.array_equal(e1, e2) and np.array_equal(f1, f2)
    e3, f3 = D.em.em_eval(ctx, x[4:5])
    assert np.array_equal(e3[0], e1[4]) and np.array_equal(f3[0], f1[4])
    ctx.close()


def test_em_device_resident_and_errors(D, em):
    import torch
    s = g.em_system(120, seed=10)
    x = g.em_conformations(s, 3, seed=11)
    ctx = D.em.em_init(s)
    eh, fh = D.em.em_eval(ctx, x)
    ed, fd = D.em.em_eval(ctx, torch.from_numpy(x).cuda())
    assert np.array_equal(ed, eh) and np.array_equal(fd, fh)
    ctx.close()
    bad = dataclasses.replace(s, pairs=s.pairs[::-1].copy())        # unsorted pair list
    with pytest.raises(D.DockError) as e:
        D.em.em_init(bad)
    assert e.value.status == -1
    bad = dataclasses.replace(s, R=np.zeros_like(s.R))               # radius must be > 0
    with pytest.raises(D.DockError):
        D.em.em_init(bad)
