"""Pins for the oracle's block-Jacobi preconditioner and PCG (NEXT-1, Sec. IV.C.1).

* M = the 4x4 tridiagonal blocks of A on 4-cell strips (reading R18: along
  y), truncated to 3/2/1 at the mesh edge and at block-row boundaries;
  z = M^{-1} r by the Thomas algorithm == a dense LAPACK solve with the block-diagonal
  part of the assembled A.
* "typically reduces the condition number of the matrix by around 40%":
  on the diffusion-dominated operator (uniform density, rx >> 1) the dense spectra give
  kappa(M^{-1}A) / kappa(A) = 0.595 -> a 40.5% reduction.
* The block-Jacobi PCG reaches the dense direct solution; it needs fewer iterations than
  CG on the pipe (kappa reduction -> sqrt(0.6) fewer, eq (6)).
"""
import numpy as np
import pytest

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
from test_oracle_operator import dense_A, deck_coeffs


def strip_blocks(nx, ny, ybounds):
    for j in range(nx):
        for b in range(len(ybounds) - 1):
            for k0 in range(ybounds[b], ybounds[b + 1], 4):
                yield [k * nx + j for k in range(k0, min(k0 + 4, ybounds[b + 1]))]


def block_diag(A, nx, ny, ybounds):
    M = np.zeros_like(A)
    for idx in strip_blocks(nx, ny, ybounds):
        M[np.ix_(idx, idx)] = A[np.ix_(idx, idx)]
    return M


@pytest.mark.parametrize("nx,ny,ybounds", [(9, 14, [0, 14]), (9, 14, [0, 5, 9, 14]),
                                           (5, 3, [0, 3]), (7, 17, [0, 6, 11, 17]),
                                           (1, 9, [0, 9])])
def test_bj_apply_is_block_diagonal_solve(ora, nx, ny, ybounds):
    d = inputs.random_fields(nx, ny, seed=nx * ny, dt=0.4)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    M = block_diag(A, nx, ny, ybounds)
    sizes = sorted({len(i) for i in strip_blocks(nx, ny, ybounds)})
    assert max(sizes) == min(4, max(np.diff(ybounds)))
    r = np.random.default_rng(3).standard_normal((ny, nx))
    z = ora.bj_apply(Kx, Ky, r, ybounds)
    np.testing.assert_allclose(z.ravel(), np.linalg.solve(M, r.ravel()), rtol=1e-12,
                               atol=1e-14 * np.abs(z).max())


@pytest.mark.parametrize("dt", [4.0, 40.0])
def test_bj_condition_number_reduction_40pct(ora, dt):
    n = 32
    d = inputs.uniform_fields(n, n, rho=1.0, dt=dt)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, n, n)
    M = block_diag(A, n, n, [0, n])
    ev = np.linalg.eigvalsh(A)
    Li = np.linalg.inv(np.linalg.cholesky(M))
    evp = np.linalg.eigvalsh(Li @ A @ Li.T)
    reduction = 1 - (evp[-1] / evp[0]) / (ev[-1] / ev[0])
    assert 0.38 <= reduction <= 0.43, reduction  # "around 40%"


@pytest.mark.parametrize("kind,n,dt,yb", [("pipe", 16, 0.004, None), ("random", 13, 4.0, None),
                                           ("random", 12, 40.0, [0, 5, 12])])
def test_bjcg_dense_solve(ora, kind, n, dt, yb):
    d = inputs.crooked_pipe(n) if kind == "pipe" else inputs.random_fields(n, n, 2, dt=dt)
    Kx, Ky = deck_coeffs(ora, d)
    u0 = d.density * d.energy
    ustar = np.linalg.solve(dense_A(ora, Kx, Ky, n, n), u0.ravel()).reshape(n, n)
    res = ora.solve(Kx, Ky, u0, method=ora.BJCG, eps=1e-15, max_iters=5000, ybounds=yb)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


def test_bjcg_fewer_iterations_than_cg(ora):
    d = inputs.crooked_pipe(128)
    Kx, Ky = deck_coeffs(ora, d)
    u0 = d.density * d.energy
    cg = ora.solve(Kx, Ky, u0, method=ora.CG, eps=1e-12)
    bj = ora.solve(Kx, Ky, u0, method=ora.BJCG, eps=1e-12)
    assert bj.status == 0 and cg.status == 0
    assert bj.stats["iterations"] < 0.85 * cg.stats["iterations"]
    assert np.abs(bj.u - cg.u).max() / np.abs(cg.u).max() <= 1e-11
