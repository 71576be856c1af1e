"""Pins for the oracle's Chebyshev preconditioner and Lanczos eigen-estimate.

* eq (2): B(l) l = 1 - T_m(xi(l))/T_m(xi(0)), eq (3) xi(l) =
  (2l - (lmax+lmin))/(lmax-lmin); with s matvecs m = s+1 (reading R9). Checked on
  exact eigenvectors (DCT-II modes of a uniform-density mesh) against numpy's
  Chebyshev T_m (a library closed form, independent of the recurrence).
* eq (4)-(5): spec(B(A) A) in [1-e_m, 1+e_m], e_m = 1/|T_m((lmax+lmin)/(lmax-lmin))|
  when [lmin, lmax] brackets spec(A); B(A) symmetric positive definite.
* Lanczos (reading R7): eigenvalues of T built from CG's alpha/beta equal the
  eigenvalues of A once the Krylov space is the whole space; T equals the
  projection R^T A R onto the normalised CG residuals (an explicit Lanczos basis).
* Sturm bisection eigenvalues vs LAPACK eigvalsh on random tridiagonals.
"""
import numpy as np
import numpy.polynomial.chebyshev as npc
import pytest

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
from test_oracle_operator import dense_A, deck_coeffs


def T(m, x):
    c = np.zeros(m + 1)
    c[m] = 1.0
    return npc.chebval(x, c)


def cheb_closed_form(lam, lmin, lmax, m):
    xi = lambda l: (2 * l - (lmax + lmin)) / (lmax - lmin)
    return 1.0 - T(m, xi(lam)) / T(m, xi(0.0))


@pytest.mark.parametrize("s", [1, 2, 3, 5, 10])
@pytest.mark.parametrize("rho,extent", [(1.0, (0, 10, 0, 10)), (0.05, (0, 3, 0, 5))])
def test_cheb_identity_on_eigenvectors(ora, s, rho, extent):
    nx, ny = 12, 10
    d = inputs.uniform_fields(nx, ny, rho=rho, dt=0.05, extent=extent)
    rx, ry = ora.mesh_r(d)
    Kx, Ky = deck_coeffs(ora, d)
    lam_all = (1.0 + 4 * (rx / rho) * np.sin(np.pi * np.arange(nx) / (2 * nx))[None, :] ** 2
               + 4 * (ry / rho) * np.sin(np.pi * np.arange(ny) / (2 * ny))[:, None] ** 2)
    lmin, lmax = 0.9, 1.1 * lam_all.max()
    theta, a, b = ora.cheb_coeffs(lmin, lmax, s)
    assert theta == pytest.approx((lmax + lmin) / 2, rel=1e-15)
    x = (np.arange(nx) + 0.5) / nx
    y = (np.arange(ny) + 0.5) / ny
    for (i, j) in [(0, 0), (1, 0), (0, 1), (3, 2), (nx - 1, ny - 1), (5, 7)]:
        v = np.cos(np.pi * j * y)[:, None] * np.cos(np.pi * i * x)[None, :]
        lam = lam_all[j, i]
        z = ora.cheb_apply(Kx, Ky, s, theta, a, b, v)
        big = np.abs(v) > 0.2
        ratio = (z[big] / v[big]) * lam
        expect = cheb_closed_form(lam, lmin, lmax, s + 1)
        np.testing.assert_allclose(ratio, expect, rtol=1e-10, atol=1e-12)


@pytest.mark.parametrize("s", [1, 2, 4, 10])
def test_preconditioned_spectrum_bound(ora, s):
    nx = ny = 8
    d = inputs.random_fields(nx, ny, seed=4, dt=0.05)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    ev = np.linalg.eigvalsh(A)
    lmin, lmax = ev[0], ev[-1]
    theta, a, b = ora.cheb_coeffs(lmin, lmax, s)
    n = nx * ny
    B = np.zeros((n, n))
    for c in range(n):
        e = np.zeros(n)
        e[c] = 1.0
        B[:, c] = ora.cheb_apply(Kx, Ky, s, theta, a, b, e.reshape(ny, nx)).ravel()
    np.testing.assert_allclose(B, B.T, atol=1e-12 * np.abs(B).max())
    assert np.linalg.eigvalsh((B + B.T) / 2)[0] > 0
    BA = B @ A
    mu = np.sort(np.linalg.eigvals(BA).real)
    m = s + 1
    eps_m = 1.0 / abs(T(m, (lmax + lmin) / (lmax - lmin)))
    assert mu[0] >= 1 - eps_m - 1e-9 and mu[-1] <= 1 + eps_m + 1e-9
    # eq (4): condition number bound
    assert mu[-1] / mu[0] <= (1 + eps_m) / (1 - eps_m) * (1 + 1e-9)


def test_tridiag_bisection_vs_lapack(ora):
    rng = np.random.default_rng(0)
    for n in (1, 2, 3, 7, 30, 64):
        dd = rng.uniform(-5, 20, n)
        ee = rng.standard_normal(max(n - 1, 0)) * 3
        M = np.diag(dd) + np.diag(ee, 1) + np.diag(ee, -1)
        np.testing.assert_allclose(ora.tridiag_eigs(dd, ee), np.linalg.eigvalsh(M),
                                   rtol=1e-13, atol=1e-12)
    # clustered / repeated eigenvalues
    dd = np.array([2.0, 2.0, 2.0, 5.0])
    ee = np.array([0.0, 0.0, 1e-9])
    M = np.diag(dd) + np.diag(ee, 1) + np.diag(ee, -1)
    np.testing.assert_allclose(ora.tridiag_eigs(dd, ee), np.linalg.eigvalsh(M), atol=1e-13)


def _textbook_cg(A, b, nsteps):
    """Hestenes-Stiefel CG (independent test-side loop) returning alpha, beta, residuals."""
    x = np.zeros_like(b)
    r = b.copy()
    p = r.copy()
    rr = r @ r
    alphas, betas, res = [], [], [r.copy()]
    for _ in range(nsteps):
        w = A @ p
        al = rr / (p @ w)
        x += al * p
        r -= al * w
        rrn = r @ r
        be = rrn / rr
        p = r + be * p
        rr = rrn
        alphas.append(al)
        betas.append(be)
        res.append(r.copy())
    return np.array(alphas), np.array(betas), res


def test_lanczos_T_is_projection_and_ritz_values(ora):
    nx, ny = 3, 3
    d = inputs.random_fields(nx, ny, seed=9, dt=0.05)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    b = np.random.default_rng(1).standard_normal(nx * ny)
    n = nx * ny
    al, be, res = _textbook_cg(A, b, n)
    dd, ee = ora.lanczos_T(al, be[: n - 1])
    # projection onto normalised residuals (Lanczos vectors up to sign)
    k = 5
    R = np.stack([res[i] / np.linalg.norm(res[i]) * (-1) ** i for i in range(k)], axis=1)
    P = R.T @ A @ R
    np.testing.assert_allclose(np.diag(P), dd[:k], rtol=1e-9)
    np.testing.assert_allclose(np.abs(np.diag(P, 1)), np.abs(ee[: k - 1]), rtol=1e-8)
    # full Krylov space: Ritz values are A's eigenvalues
    ritz = ora.tridiag_eigs(dd, ee)
    np.testing.assert_allclose(ritz, np.linalg.eigvalsh(A), rtol=1e-8)
    st, (rmin, rmax, lmin, lmax) = ora.eig_estimate(al, be[: n - 1])
    assert st == 0
    assert rmin == pytest.approx(np.linalg.eigvalsh(A)[0], rel=1e-8)
    assert lmin == pytest.approx(0.95 * rmin) and lmax == pytest.approx(1.05 * rmax)


def test_eig_estimate_within_gershgorin(ora):
    """Ritz values lie inside [1, Gershgorin] (reading R8 sanity bounds)."""
    d = inputs.crooked_pipe(128)
    Kx, Ky = deck_coeffs(ora, d)
    res = ora.solve(Kx, Ky, d.density * d.energy, method=1, eps=1e-15, max_iters=10000)
    st = res.stats
    assert 1.0 <= st["ritz_min"] <= st["ritz_max"]
    gersh = 1 + 2 * (Kx[:, :-1] + Kx[:, 1:]).max() + 2 * (Ky[:-1] + Ky[1:]).max()
    assert st["ritz_max"] <= gersh


def test_eig_estimate_breakdown(ora):
    st, _ = ora.eig_estimate(np.array([-1.0]), np.array([]))
    assert st == -4
