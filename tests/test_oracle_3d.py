"""Pins for the oracle's 3D 7-point operator and solves.

* dense structure: symmetric, diag = 1 + sum|off| (P:L341-343 carried to 3D), 7-point
  sparsity, A1 = 1, lambda_min = 1;
* uniform density: spectrum = 1 + sum_d 4 (r_d/rho) sin^2(pi i_d / 2 n_d) with distinct
  rx, ry, rz (catches an axis swap); DCT-III x3 closed-form solve;
* nz = 1: the 3D solve equals the 2D Listing-1 solve bitwise (the z terms are exact zeros);
* CG / CPPCG / CG1 / Jacobi / Chebyshev reach the dense solution.
"""
import numpy as np
import pytest
import scipy.fft

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs


def dense_A3(ora, Kx, Ky, Kz, nx, ny, nz):
    n = nx * ny * nz
    A = np.zeros((n, n))
    for c in range(n):
        e = np.zeros(n)
        e[c] = 1.0
        A[:, c] = ora.apply_A3(Kx, Ky, Kz, e.reshape(nz, ny, nx)).ravel()
    return A


def coeffs3(ora, d):
    rx, ry, rz = ora.mesh_r3(d)
    return ora.face_coefficients3(d.nx, d.ny, d.nz, rx, ry, rz, d.density)


@pytest.mark.parametrize("nx,ny,nz", [(5, 4, 3), (3, 6, 5), (1, 4, 6), (6, 1, 1)])
def test_dense_structure_3d(ora, nx, ny, nz):
    d = inputs.random_fields3(nx, ny, nz, seed=nx + 10 * ny + 100 * nz, dt=0.04)
    Kx, Ky, Kz = coeffs3(ora, d)
    A = dense_A3(ora, Kx, Ky, Kz, nx, ny, nz)
    assert np.array_equal(A, A.T)
    off = A - np.diag(np.diag(A))
    assert (off <= 0).all()
    np.testing.assert_allclose(np.diag(A), 1.0 + np.abs(off).sum(axis=1), rtol=1e-14)
    for row in range(nx * ny * nz):
        nzs = np.nonzero(off[row])[0]
        assert len(nzs) <= 6
    np.testing.assert_allclose(A.sum(axis=1), 1.0, atol=1e-12 * np.abs(off).max() + 1e-15)
    assert np.linalg.eigvalsh(A)[0] == pytest.approx(1.0, rel=1e-10)


def test_uniform_spectrum_and_dct_solve_3d(ora):
    nx, ny, nz = 6, 5, 4
    rho = 0.5
    d = inputs.uniform_fields3(nx, ny, nz, rho=rho, dt=0.05, extent=(0, 3, 0, 7, 0, 2))
    rx, ry, rz = ora.mesh_r3(d)
    Kx, Ky, Kz = coeffs3(ora, d)
    A = dense_A3(ora, Kx, Ky, Kz, nx, ny, nz)
    lam = (1.0 + 4 * (rx / rho) * np.sin(np.pi * np.arange(nx) / (2 * nx))[None, None, :] ** 2
           + 4 * (ry / rho) * np.sin(np.pi * np.arange(ny) / (2 * ny))[None, :, None] ** 2
           + 4 * (rz / rho) * np.sin(np.pi * np.arange(nz) / (2 * nz))[:, None, None] ** 2)
    np.testing.assert_allclose(np.linalg.eigvalsh(A), np.sort(lam.ravel()), rtol=1e-12)
    u0 = d.density * d.energy
    ustar = scipy.fft.idctn(scipy.fft.dctn(u0, type=2, norm="ortho") / lam, type=2, norm="ortho")
    for m in (ora.CG, ora.CPPCG, ora.CG1):
        res = ora.solve3(Kx, Ky, Kz, u0, method=m, eps=1e-14, max_iters=5000, inner_steps=4,
                         presteps=6)
        assert res.status == 0
        assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


def test_nz1_equals_2d_bitwise(ora):
    d2 = inputs.random_fields(9, 7, seed=3, dt=0.04)
    d3 = inputs.Deck3(9, 7, 1, d2.xmin, d2.xmax, d2.ymin, d2.ymax, 0.0, 1.0, d2.dt,
                      d2.density[None].copy(), d2.energy[None].copy())
    rx, ry = ora.mesh_r(d2)
    Kx2, Ky2 = ora.face_coefficients(9, 7, rx, ry, d2.density)
    Kx, Ky, Kz = coeffs3(ora, d3)
    assert np.array_equal(Kx[0], Kx2) and np.array_equal(Ky[0], Ky2) and not Kz.any()
    u0 = d2.density * d2.energy
    for m in (ora.CG, ora.CPPCG, ora.CG1, ora.JACOBI, ora.CHEBY):
        a = ora.solve(Kx2, Ky2, u0, method=m, eps=0.0, max_iters=37, inner_steps=5, presteps=8)
        b = ora.solve3(Kx, Ky, Kz, u0[None], method=m, eps=0.0, max_iters=37, inner_steps=5,
                       presteps=8)
        assert np.array_equal(a.u, b.u[0]), m


@pytest.mark.parametrize("method", [0, 1, 3, 4, 5])
def test_dense_solve_3d(ora, method):
    d = inputs.crooked_pipe3(6, 5, 7)
    d.dt = 0.4
    Kx, Ky, Kz = coeffs3(ora, d)
    A = dense_A3(ora, Kx, Ky, Kz, 6, 5, 7)
    u0 = d.density * d.energy
    ustar = np.linalg.solve(A, u0.ravel()).reshape(u0.shape)
    res = ora.solve3(Kx, Ky, Kz, u0, method=method, eps=1e-14, max_iters=200000, inner_steps=4,
                     presteps=30)
    assert res.status == 0
    assert np.abs(res.u - ustar).max() / np.abs(ustar).max() <= 1e-11


def test_chebyshev_divergence_is_reported(ora):
    """a pure Chebyshev solver "cannot cope" when the interval misses the
    top of the spectrum: with 8 presteps lambda_max is under-estimated here (9.6 < 11.1)
    and the iteration diverges -- reported as breakdown, not as a result."""
    d = inputs.crooked_pipe3(6, 5, 7)
    d.dt = 0.4
    Kx, Ky, Kz = coeffs3(ora, d)
    u0 = d.density * d.energy
    res = ora.solve3(Kx, Ky, Kz, u0, method=ora.CHEBY, eps=1e-14, max_iters=200000, presteps=8)
    assert res.status == ora.ERR_BREAKDOWN
