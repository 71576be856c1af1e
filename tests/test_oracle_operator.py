"""Pins for the oracle's operator A and face coefficients (CPU, no GPU).

Each check is fixed by the paper or by mathematics, not by re-typing the
oracle's formula:

* P:L341-343 (Sec. IV.A): "The diagonal is one plus the sum of the rest of the
  nonzero elements on the row, making A diagonally dominant" -> diag = 1 + sum|off|.
* Listing 1 is symmetric by construction of shared faces ->
  A == A^T exactly; reflective boundary (reading R3) -> A 1 = 1, lambda_min = 1.
* Uniform density: A = I + (rx/rho) Lx (+) (ry/rho) Ly with Neumann Laplacians,
  whose spectrum is the textbook 4 sin^2(pi i / 2n) (closed form).
* Two-cell problem: eigenvalues 1 and 1 + 2K with K the face value of reading R1.
"""
import numpy as np
import pytest

from paper_conf_cluster_mcintosh_smithm17_b200 import inputs


def dense_A(ora, Kx, Ky, nx, ny):
    n = nx * ny
    A = np.zeros((n, n))
    for c in range(n):
        e = np.zeros(n)
        e[c] = 1.0
        A[:, c] = ora.apply_A(Kx, Ky, e.reshape(ny, nx)).ravel()
    return A


def deck_coeffs(ora, d, mean_mode=0):
    rx, ry = ora.mesh_r(d)
    return ora.face_coefficients(d.nx, d.ny, rx, ry, d.density, mean_mode)


DECKS = [
    ("pipe", 16, 16, 0),
    ("random", 12, 9, 1),
    ("random", 7, 13, 2),
    ("random", 1, 11, 3),
    ("random", 10, 1, 4),
]


@pytest.mark.parametrize("kind,nx,ny,seed", DECKS)
def test_dense_structure(ora, kind, nx, ny, seed):
    d = inputs.deck(kind, nx, ny, seed=seed) if kind != "pipe" else inputs.crooked_pipe(nx, ny)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    # exact symmetry (shared faces)
    assert np.array_equal(A, A.T)
    off = A - np.diag(np.diag(A))
    # off-diagonals are non-positive (M-matrix) and diag = 1 + sum |off|
    assert (off <= 0).all()
    np.testing.assert_allclose(np.diag(A), 1.0 + np.abs(off).sum(axis=1), rtol=1e-14)
    # reflective boundary: row sums are exactly one up to rounding -> A 1 = 1
    one = ora.apply_A(Kx, Ky, np.ones((ny, nx)))
    np.testing.assert_allclose(one, 1.0, rtol=0, atol=1e-12 * max(1.0, np.abs(off).max()))
    ev = np.linalg.eigvalsh(A)
    # SPD, lambda_min = 1 (the constant vector), lambda_max <= Gershgorin bound
    assert ev[0] == pytest.approx(1.0, rel=1e-10)
    assert ev[-1] <= (np.diag(A) + np.abs(off).sum(axis=1)).max() * (1 + 1e-14)
    # 5-point sparsity: at most 4 off-diagonal entries per row, all nearest neighbours
    for row in range(nx * ny):
        nz = np.nonzero(off[row])[0]
        assert len(nz) <= 4
        k, j = divmod(row, nx)
        for c in nz:
            kk, jj = divmod(c, nx)
            assert abs(kk - k) + abs(jj - j) == 1


@pytest.mark.parametrize("nx,ny,extent,rho", [
    (8, 6, (0.0, 10.0, 0.0, 10.0), 1.0),
    (9, 5, (0.0, 3.0, -1.0, 7.0), 0.25),   # rx != ry, nx != ny: catches an x/y swap
    (5, 12, (2.0, 4.0, 0.0, 1.0), 40.0),
])
def test_uniform_density_closed_form_spectrum(ora, nx, ny, extent, rho):
    d = inputs.uniform_fields(nx, ny, rho=rho, seed=1, dt=0.05, extent=extent)
    rx, ry = ora.mesh_r(d)
    Kx, Ky = deck_coeffs(ora, d)
    A = dense_A(ora, Kx, Ky, nx, ny)
    i = np.arange(nx)
    j = np.arange(ny)
    lam = (1.0 + 4 * (rx / rho) * np.sin(np.pi * i / (2 * nx))[None, :] ** 2
           + 4 * (ry / rho) * np.sin(np.pi * j / (2 * ny))[:, None] ** 2)
    np.testing.assert_allclose(np.linalg.eigvalsh(A), np.sort(lam.ravel()), rtol=1e-12)


@pytest.mark.parametrize("r1,r2", [(1.0, 1.0), (0.1, 100.0), (3.0, 0.5)])
def test_two_cell_face_value(ora, r1, r2):
    """nx=2, ny=1: A = [[1+K,-K],[-K,1+K]], K = rx (r1+r2)/(2 r1 r2) (reading R1);
    mean_mode=1 gives K = rx (r1+r2)/2 (the literal 'averaged density')."""
    rho = np.array([[r1, r2]])
    rx = 0.37
    for mode, K in ((0, rx * (r1 + r2) / (2 * r1 * r2)), (1, rx * (r1 + r2) / 2)):
        Kx, Ky = ora.face_coefficients(2, 1, rx, 0.9, rho, mode)
        A = dense_A(ora, Kx, Ky, 2, 1)
        np.testing.assert_allclose(np.linalg.eigvalsh(A), [1.0, 1.0 + 2 * K], rtol=1e-14)
        assert np.all(Ky == 0.0)  # both y faces are physical boundaries


def test_low_density_conducts_more(ora):
    """the low-density pipe has the higher heat conduction."""
    d = inputs.crooked_pipe(32)
    Kx, Ky = deck_coeffs(ora, d)
    rho = d.density
    inside = (rho[:, :-1] == 0.1) & (rho[:, 1:] == 0.1)
    outside = (rho[:, :-1] == 100.0) & (rho[:, 1:] == 100.0)
    assert Kx[:, 1:-1][inside].min() > 100 * Kx[:, 1:-1][outside].max()


def test_listing1_dot_is_pw(ora):
    """eq (9): the oracle's dot is the plain sum p.w in loop order."""
    rng = np.random.default_rng(5)
    a, b = rng.standard_normal((7, 9)), rng.standard_normal((7, 9))
    assert ora.dot(a, b) == pytest.approx(float(np.sum(a * b)), rel=1e-13)


@pytest.mark.parametrize("nx,ny,seed", [(17, 13, 0), (40, 31, 1), (1, 25, 2), (23, 1, 3)])
def test_energy_form_of_zAz(ora, nx, ny, seed):
    """z.(A z) = sum_c z_c^2 + sum_faces K_f (z_i - z_j)^2 (A = I + L, L the face-weighted graph
    Laplacian of Listing 1): the identity the GPU's CPPCG1F last pass uses to form del = z.q
    from z alone, each face counted once by its west / south cell (reading R23)."""
    d = inputs.random_fields(nx, ny, seed, dt=0.4)
    rx, ry = ora.mesh_r(d)
    Kx, Ky = ora.face_coefficients(nx, ny, rx, ry, d.density)
    z = np.random.default_rng(seed).standard_normal((ny, nx))
    lhs = ora.dot(z, ora.apply_A(Kx, Ky, z))
    # Kx[k, j] = face between cells j-1 and j (0 at the boundary columns), Ky[k, j] likewise
    faces = np.sum(Kx[:, 1:nx] * (z[:, 1:] - z[:, :-1]) ** 2) + \
        np.sum(Ky[1:ny, :] * (z[1:, :] - z[:-1, :]) ** 2)
    rhs = np.sum(z * z) + faces
    assert lhs == pytest.approx(rhs, rel=1e-13)
    assert np.all(Kx[:, 0] == 0) and np.all(Kx[:, nx] == 0)  # reflective boundary (R3)
