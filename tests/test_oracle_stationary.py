"""Pins for the oracle's stand-alone Jacobi and Chebyshev solvers (NEXT-4).

* Jacobi: u_k = u* + G^k (u_0 - u*), G = I - D^{-1} A with D = diag(A) (dense matrix
  powers on small meshes) -- the iteration, not just its fixed point.
* Chebyshev (Saad Alg. 12.1, eq (2)-(3) mapping): after the CG presteps (iterate u_p),
  k Chebyshev updates give u_{p+k} - u* = T_k(xi(A)) / T_k(xi(0)) (u_p - u*), with
  xi(l) = (2 l - (lmax + lmin)) / (lmax - lmin) on the estimated interval (dense
  Chebyshev recurrence on matrices, independent of the vector recurrence).
* Both reach the dense direct solution.
"""
import numpy as np
import pytest

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
from test_oracle_operator import dense_A, deck_coeffs


def setup(ora, d):
    Kx, Ky = deck_coeffs(ora, d)
    return Kx, Ky, d.density * d.energy


@pytest.mark.parametrize("nx,ny,dt", [(9, 7, 0.04), (12, 5, 0.4)])
def test_jacobi_is_matrix_power(ora, nx, ny, dt):
    d = inputs.random_fields(nx, ny, seed=5, dt=dt)
    Kx, Ky, u0 = setup(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    ustar = np.linalg.solve(A, u0.ravel())
    G = np.eye(nx * ny) - np.diag(1.0 / np.diag(A)) @ A
    e0 = u0.ravel() - ustar
    for k in (1, 2, 5, 13):
        res = ora.solve(Kx, Ky, u0, method=ora.JACOBI, eps=0.0, max_iters=k)
        assert res.stats["iterations"] == k
        ek = np.linalg.matrix_power(G, k) @ e0
        np.testing.assert_allclose(res.u.ravel() - ustar, ek, atol=1e-12 * np.abs(u0).max())


def test_jacobi_dense_solve(ora):
    d = inputs.random_fields(10, 8, seed=2, dt=0.04)
    Kx, Ky, u0 = setup(ora, d)
    ustar = np.linalg.solve(dense_A(ora, Kx, Ky, 10, 8), u0.ravel()).reshape(8, 10)
    res = ora.solve(Kx, Ky, u0, method=ora.JACOBI, eps=1e-14, max_iters=200000)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-12


def cheb_matrix(A, lmin, lmax, k):
    n = A.shape[0]
    X = (2 * A - (lmax + lmin) * np.eye(n)) / (lmax - lmin)
    x0 = -(lmax + lmin) / (lmax - lmin)
    Tm, T = np.eye(n), X.copy()
    tm, t = 1.0, x0
    if k == 0:
        return np.eye(n)
    for _ in range(k - 1):
        Tm, T = T, 2 * X @ T - Tm
        tm, t = t, 2 * x0 * t - tm
    return T / t


@pytest.mark.parametrize("n,dt,pre", [(9, 0.4, 4), (8, 4.0, 6)])
def test_chebyshev_error_polynomial(ora, n, dt, pre):
    d = inputs.random_fields(n, n, seed=4, dt=dt)
    Kx, Ky, u0 = setup(ora, d)
    A = dense_A(ora, Kx, Ky, n, n)
    ustar = np.linalg.solve(A, u0.ravel())
    base = ora.solve(Kx, Ky, u0, method=ora.CHEBY, eps=0.0, max_iters=pre, presteps=pre)
    ep = base.u.ravel() - ustar
    for k in (1, 2, 3, 7):
        res = ora.solve(Kx, Ky, u0, method=ora.CHEBY, eps=0.0, max_iters=pre + k, presteps=pre)
        st = res.stats
        assert st["presteps"] == pre and st["outer"] == k
        P = cheb_matrix(A, st["eig_min"], st["eig_max"], k)
        np.testing.assert_allclose(res.u.ravel() - ustar, P @ ep,
                                   atol=1e-11 * np.abs(u0).max())


@pytest.mark.parametrize("kind,n", [("pipe", 16), ("random", 12)])
def test_chebyshev_dense_solve(ora, kind, n):
    d = inputs.crooked_pipe(n) if kind == "pipe" else inputs.random_fields(n, n, 1, dt=0.4)
    Kx, Ky, u0 = setup(ora, d)
    ustar = np.linalg.solve(dense_A(ora, Kx, Ky, n, n), u0.ravel()).reshape(n, n)
    res = ora.solve(Kx, Ky, u0, method=ora.CHEBY, eps=1e-14, max_iters=100000, presteps=8)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11
