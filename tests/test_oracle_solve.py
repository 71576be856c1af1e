"""Pins for the oracle's CG / CPPCG solves (CPU, no GPU).

The method reaches u* = A^{-1} u^n (A is SPD, so the solution is unique); CG and
CPPCG are two routes to it. Pins:

* dense direct solve (numpy LAPACK) on <= 16x16 meshes, several dt (conditioning);
* DCT-II diagonalisation for uniform density at any size (closed form);
* nx = 1: tridiagonal (Thomas / LAPACK banded) solve;
* invariants: sum(u) conserved at EVERY iteration under reflective boundaries
  (1^T r_0 = 0, A 1 = 1); discrete maximum principle (A is an M-matrix with unit
  row sums); monotone A-norm error of CG (CG minimises it over the Krylov space);
* eq (6) iteration bound, with kappa from the dense spectrum;
* CPPCG field == CG field (same system).
"""
import numpy as np
import pytest
import scipy.fft
import scipy.linalg

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
from test_oracle_operator import dense_A, deck_coeffs


def setup(ora, d):
    Kx, Ky = deck_coeffs(ora, d)
    u0 = d.density * d.energy
    return Kx, Ky, u0


SMALL = [("pipe", 16, 16, 0, 0.004), ("random", 16, 16, 1, 0.4), ("random", 13, 11, 2, 4.0),
         ("random", 12, 12, 3, 40.0), ("random", 16, 5, 4, 4.0)]


@pytest.mark.parametrize("kind,nx,ny,seed,dt", SMALL)
@pytest.mark.parametrize("method", [0, 1])
def test_dense_direct_solve(ora, kind, nx, ny, seed, dt, method):
    d = (inputs.random_fields(nx, ny, seed, dt=dt) if kind == "random"
         else inputs.crooked_pipe(nx, ny))
    Kx, Ky, u0 = setup(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    ustar = np.linalg.solve(A, u0.ravel()).reshape(ny, nx)
    res = ora.solve(Kx, Ky, u0, method=method, eps=1e-15, max_iters=5000, inner_steps=4,
                    presteps=8)
    assert res.status == 0
    err = np.abs(res.u - ustar).max() / np.abs(ustar).max()
    assert err <= 1e-11, err


@pytest.mark.parametrize("nx,ny,rho,method", [(96, 64, 1.0, 0), (64, 96, 0.1, 1),
                                              (80, 80, 2.0, 1)])
def test_uniform_density_dct_solve(ora, nx, ny, rho, method):
    d = inputs.uniform_fields(nx, ny, rho=rho, seed=7)
    rx, ry = ora.mesh_r(d)
    Kx, Ky, u0 = setup(ora, d)
    i, j = np.arange(nx), np.arange(ny)
    lam = (1.0 + 4 * (rx / rho) * np.sin(np.pi * i / (2 * nx))[None, :] ** 2
           + 4 * (ry / rho) * np.sin(np.pi * j / (2 * ny))[:, None] ** 2)
    ustar = scipy.fft.idctn(scipy.fft.dctn(u0, type=2, norm="ortho") / lam, type=2,
                            norm="ortho")
    res = ora.solve(Kx, Ky, u0, method=method, eps=1e-14, max_iters=20000, inner_steps=6)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


@pytest.mark.parametrize("method", [0, 1])
def test_single_column_thomas(ora, method):
    d = inputs.random_fields(1, 200, seed=11, dt=0.4)
    Kx, Ky, u0 = setup(ora, d)
    ky = Ky[:, 0]  # faces 0..ny
    diag = 1.0 + ky[1:] + ky[:-1]
    ab = np.zeros((3, 200))
    ab[0, 1:] = -ky[1:-1]
    ab[1] = diag
    ab[2, :-1] = -ky[1:-1]
    ustar = scipy.linalg.solve_banded((1, 1), ab, u0[:, 0])
    res = ora.solve(Kx, Ky, u0, method=method, eps=1e-15, max_iters=5000, inner_steps=3,
                    presteps=10)
    assert res.status == 0
    np.testing.assert_allclose(res.u[:, 0], ustar, rtol=1e-10)


@pytest.mark.parametrize("method,ks", [(0, range(1, 40, 3)), (1, [31, 32, 35, 40, 45])])
def test_conservation_every_iteration(ora, method, ks):
    d = inputs.crooked_pipe(32)
    Kx, Ky, u0 = setup(ora, d)
    s0 = u0.sum()
    for k in ks:
        res = ora.solve(Kx, Ky, u0, method=method, eps=0.0, max_iters=k, inner_steps=5)
        assert res.stats["iterations"] == k
        assert abs(res.u.sum() - s0) / s0 <= 1e-13


@pytest.mark.parametrize("kind,seed", [("pipe", 0), ("random", 3)])
def test_maximum_principle(ora, kind, seed):
    d = inputs.crooked_pipe(48) if kind == "pipe" else inputs.random_fields(40, 30, seed)
    Kx, Ky, u0 = setup(ora, d)
    for method in (0, 1):
        res = ora.solve(Kx, Ky, u0, method=method, eps=1e-14, max_iters=20000)
        tol = 1e-10 * np.abs(u0).max()
        assert res.u.min() >= u0.min() - tol
        assert res.u.max() <= u0.max() + tol


@pytest.mark.parametrize("nx,dt", [(16, 4.0), (16, 0.4), (12, 40.0)])
def test_cg_monotone_A_norm_error(ora, nx, dt):
    """Reading R16: ||r|| is not monotone in CG, the A-norm error is."""
    d = inputs.random_fields(nx, nx, seed=2, dt=dt)
    Kx, Ky, u0 = setup(ora, d)
    A = dense_A(ora, Kx, Ky, nx, nx)
    ustar = np.linalg.solve(A, u0.ravel())
    e0 = u0.ravel() - ustar
    E0 = np.sqrt(e0 @ A @ e0)
    prev = E0
    for k in range(1, 400):
        res = ora.solve(Kx, Ky, u0, method=0, eps=0.0, max_iters=k)
        e = res.u.ravel() - ustar
        E = np.sqrt(max(e @ A @ e, 0.0))
        if prev < 1e-10 * E0:
            break
        assert E <= prev * (1 + 1e-12), (k, E, prev)
        prev = E


@pytest.mark.parametrize("n", [16, 24])
def test_cg_iteration_bound_eq6(ora, n):
    """eq (6): k <= sqrt(kappa)/2 ln(2/eps_A); for a residual test ||r_k|| < eps ||r_0||
    the A-norm reduction needed is eps/sqrt(kappa)."""
    d = inputs.crooked_pipe(n)
    Kx, Ky, u0 = setup(ora, d)
    ev = np.linalg.eigvalsh(dense_A(ora, Kx, Ky, n, n))
    kappa = ev[-1] / ev[0]
    for eps in (1e-6, 1e-10, 1e-13):
        res = ora.solve(Kx, Ky, u0, method=0, eps=eps, max_iters=100000)
        bound = np.sqrt(kappa) / 2 * np.log(2 * np.sqrt(kappa) / eps)
        assert res.stats["iterations"] <= np.ceil(bound)


@pytest.mark.parametrize("n,s", [(64, 10), (64, 3), (48, 1), (40, 6)])
def test_cppcg_equals_cg(ora, n, s):
    d = inputs.crooked_pipe(n)
    Kx, Ky, u0 = setup(ora, d)
    cg = ora.solve(Kx, Ky, u0, method=0, eps=1e-15, max_iters=100000)
    pp = ora.solve(Kx, Ky, u0, method=1, eps=1e-15, max_iters=100000, inner_steps=s)
    assert cg.status == 0 and pp.status == 0
    assert pp.stats["presteps"] == 30 and pp.stats["outer"] > 0
    assert np.abs(pp.u - cg.u).max() / np.abs(cg.u).max() <= 1e-12
    # communication avoidance: far fewer outer iterations (dot products)
    assert pp.stats["outer"] * (s + 1) >= 0.5 * (cg.stats["iterations"] - 30)
    if s >= 3:
        assert pp.stats["outer"] < cg.stats["iterations"] - 30


def test_zero_residual_returns_immediately(ora):
    d = inputs.uniform_fields(8, 8, rho=1.0, dt=0.0)  # dt = 0 -> A = I exactly
    Kx, Ky, u0 = setup(ora, d)
    for m in (0, 1):
        res = ora.solve(Kx, Ky, u0, method=m, eps=1e-10, max_iters=10)
        assert res.status == 0 and res.stats["iterations"] == 0
        assert np.array_equal(res.u, u0)


def test_not_converged_and_bad_args(ora):
    d = inputs.crooked_pipe(32)
    Kx, Ky, u0 = setup(ora, d)
    res = ora.solve(Kx, Ky, u0, method=0, eps=1e-15, max_iters=5)
    assert res.status == 1 and res.stats["iterations"] == 5
    res = ora.solve(Kx, Ky, u0, method=1, eps=1e-15, max_iters=12, presteps=30)
    assert res.status == 1 and res.stats["iterations"] == 12 and res.stats["outer"] == 0
    d = inputs.crooked_pipe(128)
    Kx, Ky, u0 = setup(ora, d)
    res = ora.solve(Kx, Ky, u0, method=1, eps=1e-15, max_iters=32, presteps=30)
    assert res.status == 1 and res.stats["outer"] == 2
    assert ora.solve(Kx, Ky, u0, method=1, inner_steps=0).status == -1


# ---------------------------------------------------------------- single-reduction CG
@pytest.mark.parametrize("kind,nx,ny,seed,dt", SMALL)
def test_cg1_dense_direct_solve(ora, kind, nx, ny, seed, dt):
    """Chronopoulos-Gear CG (NEXT-2) reaches the dense solution."""
    d = (inputs.random_fields(nx, ny, seed, dt=dt) if kind == "random"
         else inputs.crooked_pipe(nx, ny))
    Kx, Ky, u0 = setup(ora, d)
    ustar = np.linalg.solve(dense_A(ora, Kx, Ky, nx, ny), u0.ravel()).reshape(ny, nx)
    res = ora.solve(Kx, Ky, u0, method=ora.CG1, eps=1e-15, max_iters=5000)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


@pytest.mark.parametrize("n", [64, 128])
def test_cg1_equivalent_to_cg(ora, n):
    """Same Krylov iterates in exact arithmetic: iteration counts within +-2, fields equal,
    and the same residual norm after every fixed iteration count (to rounding)."""
    d = inputs.crooked_pipe(n)
    Kx, Ky, u0 = setup(ora, d)
    cg = ora.solve(Kx, Ky, u0, method=ora.CG, eps=1e-13)
    c1 = ora.solve(Kx, Ky, u0, method=ora.CG1, eps=1e-13)
    assert abs(cg.stats["iterations"] - c1.stats["iterations"]) <= 2
    assert np.abs(cg.u - c1.u).max() / np.abs(cg.u).max() <= 1e-11
    for k in (1, 5, 20):
        a = ora.solve(Kx, Ky, u0, method=ora.CG, eps=0.0, max_iters=k)
        b = ora.solve(Kx, Ky, u0, method=ora.CG1, eps=0.0, max_iters=k)
        assert b.stats["rnorm"] == pytest.approx(a.stats["rnorm"], rel=1e-9)
        assert np.abs(a.u - b.u).max() / np.abs(a.u).max() <= 1e-12


def test_cg1_conservation(ora):
    d = inputs.crooked_pipe(32)
    Kx, Ky, u0 = setup(ora, d)
    for k in (1, 4, 9, 17):
        res = ora.solve(Kx, Ky, u0, method=ora.CG1, eps=0.0, max_iters=k)
        assert abs(res.u.sum() - u0.sum()) / u0.sum() <= 1e-13


# ---------------------------------------------------------------- single-reduction CPPCG
@pytest.mark.parametrize("kind,nx,ny,seed,dt", SMALL)
@pytest.mark.parametrize("s", [4, 10])
@pytest.mark.parametrize("fused", [False, True])
def test_cppcg1_dense_direct_solve(ora, kind, nx, ny, seed, dt, s, fused):
    """Chronopoulos-Gear PCG with M^{-1} = B(A) (NEXT-2 for CPPCG) reaches the
    dense solution: s = A p by recurrence (CPPCG1) and w = A p applied (CPPCG1F, R23)."""
    d = (inputs.random_fields(nx, ny, seed, dt=dt) if kind == "random"
         else inputs.crooked_pipe(nx, ny))
    Kx, Ky, u0 = setup(ora, d)
    ustar = np.linalg.solve(dense_A(ora, Kx, Ky, nx, ny), u0.ravel()).reshape(ny, nx)
    res = ora.solve(Kx, Ky, u0, method=ora.CPPCG1F if fused else ora.CPPCG1, eps=1e-15,
                    max_iters=5000, inner_steps=s, presteps=8)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


@pytest.mark.parametrize("n,s", [(64, 10), (128, 10), (96, 5)])
@pytest.mark.parametrize("fused", [False, True])
def test_cppcg1_equivalent_to_cppcg(ora, n, s, fused):
    """Same Krylov iterates as CPPCG in exact arithmetic: the same presteps and
    eigen-estimate, outer iteration counts within +-2, fields equal, and the same
    residual norm and iterate after every fixed outer count (to rounding)."""
    d = inputs.crooked_pipe(n)
    Kx, Ky, u0 = setup(ora, d)
    m1 = ora.CPPCG1F if fused else ora.CPPCG1
    a = ora.solve(Kx, Ky, u0, method=ora.CPPCG, eps=1e-13, max_iters=100000, inner_steps=s)
    b = ora.solve(Kx, Ky, u0, method=m1, eps=1e-13, max_iters=100000, inner_steps=s)
    assert a.status == b.status == 0
    assert a.stats["presteps"] == b.stats["presteps"] == 30
    assert a.stats["eig_max"] == b.stats["eig_max"]
    assert abs(a.stats["outer"] - b.stats["outer"]) <= 2
    assert np.abs(a.u - b.u).max() / np.abs(a.u).max() <= 1e-11
    for k in (1, 3, 8):
        x = ora.solve(Kx, Ky, u0, method=ora.CPPCG, eps=0.0, max_iters=30 + k, inner_steps=s)
        y = ora.solve(Kx, Ky, u0, method=m1, eps=0.0, max_iters=30 + k, inner_steps=s)
        assert x.stats["outer"] == y.stats["outer"] == k
        assert y.stats["rnorm"] == pytest.approx(x.stats["rnorm"], rel=1e-8)
        assert np.abs(x.u - y.u).max() / np.abs(x.u).max() <= 1e-12
    # matvec accounting: residual + 30 presteps + the restart's s inner steps, then per
    # outer iteration s inner steps + one matvec (CPPCG: A p; CPPCG1: q = A z, plus one at
    # the restart; CPPCG1F: A p and q = A z, plus one at the restart)
    assert a.stats["matvecs"] == 1 + 30 + s + a.stats["outer"] * (s + 1)
    assert b.stats["matvecs"] == 1 + 30 + s + 1 + b.stats["outer"] * (s + (2 if fused else 1))


@pytest.mark.parametrize("n,s", [(64, 10), (96, 5)])
def test_cppcg1f_equals_cppcg1_recurrence(ora, n, s):
    """The two single-reduction forms share their scalars (gam, del, alpha, beta) and differ
    only in how A p enters r: applied (CPPCG1F) or by the recurrence s = q + beta s (CPPCG1);
    the iterates agree to rounding after every fixed outer count."""
    d = inputs.crooked_pipe(n)
    Kx, Ky, u0 = setup(ora, d)
    for k in (1, 2, 5):
        x = ora.solve(Kx, Ky, u0, method=ora.CPPCG1, eps=0.0, max_iters=30 + k, inner_steps=s)
        y = ora.solve(Kx, Ky, u0, method=ora.CPPCG1F, eps=0.0, max_iters=30 + k, inner_steps=s)
        assert y.stats["rnorm"] == pytest.approx(x.stats["rnorm"], rel=1e-8)
        assert np.abs(x.u - y.u).max() / np.abs(x.u).max() <= 1e-12


@pytest.mark.parametrize("fused", [False, True])
def test_cppcg1_conservation_and_limits(ora, fused):
    d = inputs.crooked_pipe(48)
    Kx, Ky, u0 = setup(ora, d)
    m1 = ora.CPPCG1F if fused else ora.CPPCG1
    for k in (31, 33, 40):
        res = ora.solve(Kx, Ky, u0, method=m1, eps=0.0, max_iters=k, inner_steps=6)
        assert res.status == 1 and res.stats["iterations"] == k
        assert abs(res.u.sum() - u0.sum()) / u0.sum() <= 1e-13
    assert ora.solve(Kx, Ky, u0, method=m1, inner_steps=0).status == -1
