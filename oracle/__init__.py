"""CPU oracle for the TeaLeaf CG / CPPCG hot path -- TEST INFRASTRUCTURE ONLY.

Thin ctypes wrapper around ``oracle/tea_oracle.c`` (serial fp64 C, built with
``-O2 -ffp-contract=off``). Only ``tests/``, ``__graft_entry__.smoke()`` and the
``cpu_baseline`` / ``--impl reference`` legs of ``bench.py`` may import this
package. The product package never imports it, and it imports nothing from the
product package (inputs come in as plain numpy arrays).

Parity status: every exported function is pinned by ``tests/test_oracle_*.py``
(dense direct solves, closed-form spectra, DCT/Thomas solves, Chebyshev
closed form, invariants, an independent survey computation). Not pinned beyond
the +-2 rule: the exact iteration count and Ritz values of a particular run
("parity unpinned").
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "tea_oracle.c")
_LIB = os.path.join(_HERE, "libtea_oracle.so")
CFLAGS = ["-O2", "-ffp-contract=off", "-fno-fast-math", "-std=c99", "-fPIC", "-shared"]

CG, CPPCG, BJCG, CG1, JACOBI, CHEBY, CPPCG1, CPPCG1F = 0, 1, 2, 3, 4, 5, 6, 7
OK, NOT_CONVERGED, ERR_ARG, ERR_BREAKDOWN = 0, 1, -1, -4
PRESTEPS = 30  # reading R6


class OraStats(C.Structure):
    _fields_ = [("iterations", C.c_int), ("presteps", C.c_int), ("outer", C.c_int),
                ("inner_matvecs", C.c_int), ("matvecs", C.c_int),
                ("r0", C.c_double), ("rnorm", C.c_double),
                ("eig_min", C.c_double), ("eig_max", C.c_double),
                ("ritz_min", C.c_double), ("ritz_max", C.c_double)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


def build(force: bool = False) -> str:
    """Compile the oracle shared library (gcc, plain C)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", *CFLAGS, "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _LIB)
    return _LIB


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = C.CDLL(_LIB)
        dp = np.ctypeslib.ndpointer(dtype=np.float64, flags="C_CONTIGUOUS")
        i, d = C.c_int, C.c_double
        L.ora_face_coefficients.argtypes = [i, i, d, d, dp, i, dp, dp]
        L.ora_apply_A.argtypes = [i, i, dp, dp, dp, dp]
        L.ora_dot.argtypes = [C.c_long, dp, dp]
        L.ora_dot.restype = d
        L.ora_tridiag_eigs.argtypes = [i, dp, dp, dp]
        L.ora_lanczos_T.argtypes = [i, dp, dp, dp, dp]
        L.ora_eig_estimate.argtypes = [i, dp, dp, C.POINTER(d), C.POINTER(d),
                                       C.POINTER(d), C.POINTER(d)]
        L.ora_cheb_coeffs.argtypes = [d, d, i, C.POINTER(d), dp, dp]
        L.ora_cheb_apply.argtypes = [i, i, dp, dp, i, d, dp, dp, dp, dp, dp, dp, dp]
        L.ora_solve.argtypes = [i, i, dp, dp, dp, dp, i, d, i, i, i, C.POINTER(OraStats)]
        ip = np.ctypeslib.ndpointer(dtype=np.int32, flags="C_CONTIGUOUS")
        L.ora_solve_ex.argtypes = [i, i, dp, dp, dp, dp, i, d, i, i, i, i, ip,
                                   C.POINTER(OraStats)]
        L.ora_bj_apply.argtypes = [i, i, dp, dp, i, ip, dp, dp]
        L.ora_face_coefficients3.argtypes = [i, i, i, d, d, d, dp, i, dp, dp, dp]
        L.ora_apply_A3.argtypes = [i, i, i, dp, dp, dp, dp, dp]
        L.ora_solve3.argtypes = [i, i, i, dp, dp, dp, dp, dp, i, d, i, i, i,
                                 C.POINTER(OraStats)]
        L.ora_timestep.argtypes = [i, i, d, d, d, d, dp, dp, d, i, d, i, i, i, i, dp,
                                   C.POINTER(OraStats)]
        _lib = L
    return _lib


def _c(a):
    return np.ascontiguousarray(a, dtype=np.float64)


# --------------------------------------------------------------------------- ops
def mesh_r(deck):
    """rx = dt/dx^2, ry = dt/dy^2 (north_star)."""
    dx = (deck.xmax - deck.xmin) / deck.nx
    dy = (deck.ymax - deck.ymin) / deck.ny
    return deck.dt / (dx * dx), deck.dt / (dy * dy)


def face_coefficients(nx, ny, rx, ry, rho, mean_mode=0):
    Kx = np.zeros((ny, nx + 1))
    Ky = np.zeros((ny + 1, nx))
    lib().ora_face_coefficients(nx, ny, rx, ry, _c(rho), mean_mode, Kx, Ky)
    return Kx, Ky


def apply_A(Kx, Ky, p):
    ny, nx = p.shape
    w = np.zeros((ny, nx))
    lib().ora_apply_A(nx, ny, _c(Kx), _c(Ky), _c(p), w)
    return w


def dot(a, b):
    a, b = _c(a).ravel(), _c(b).ravel()
    return lib().ora_dot(a.size, a, b)


def tridiag_eigs(d, e):
    d, e = _c(d), _c(e)
    n = d.size
    out = np.zeros(n)
    ee = np.zeros(max(n, 1))
    ee[: e.size] = e
    lib().ora_tridiag_eigs(n, d, ee, out)
    return out


def lanczos_T(alpha, beta):
    alpha, beta = _c(alpha), _c(beta)
    n = alpha.size
    bb = np.zeros(max(n, 1))
    bb[: beta.size] = beta
    d, e = np.zeros(n), np.zeros(max(n, 1))
    lib().ora_lanczos_T(n, alpha, bb, d, e)
    return d, e[: n - 1]


def eig_estimate(alpha, beta):
    alpha, beta = _c(alpha), _c(beta)
    n = alpha.size
    bb = np.zeros(max(n, 1))
    bb[: beta.size] = beta
    vals = [C.c_double() for _ in range(4)]
    st = lib().ora_eig_estimate(n, alpha, bb, *[C.byref(v) for v in vals])
    return st, tuple(v.value for v in vals)  # (ritz_min, ritz_max, lmin, lmax)


def cheb_coeffs(lmin, lmax, s):
    a, b = np.zeros(s), np.zeros(s)
    th = C.c_double()
    lib().ora_cheb_coeffs(lmin, lmax, s, C.byref(th), a, b)
    return th.value, a, b


def cheb_apply(Kx, Ky, s, theta, a, b, r):
    ny, nx = r.shape
    z, rt, sd, w = (np.zeros((ny, nx)) for _ in range(4))
    lib().ora_cheb_apply(nx, ny, _c(Kx), _c(Ky), s, theta, _c(a), _c(b), _c(r), z, rt, sd, w)
    return z


def bj_apply(Kx, Ky, r, ybounds=None):
    """z = M^{-1} r, M = block-Jacobi strips of 4 along y (reading R18)."""
    ny, nx = r.shape
    yb = np.ascontiguousarray([0, ny] if ybounds is None else ybounds, dtype=np.int32)
    z = np.zeros((ny, nx))
    lib().ora_bj_apply(nx, ny, _c(Kx), _c(Ky), yb.size - 1, yb, _c(r), z)
    return z


@dataclass
class Result:
    u: np.ndarray
    status: int
    stats: dict


def solve(Kx, Ky, u0, u_init=None, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
          presteps=PRESTEPS, ybounds=None):
    """One linear solve A u = u0 from initial guess u_init (default u0). ybounds: the
    block-row boundaries that truncate the block-Jacobi strips (default one block)."""
    ny, nx = u0.shape
    u = _c(u0 if u_init is None else u_init).copy()
    st = OraStats()
    yb = np.ascontiguousarray([0, ny] if ybounds is None else ybounds, dtype=np.int32)
    s = lib().ora_solve_ex(nx, ny, _c(Kx), _c(Ky), _c(u0), u, method, eps, max_iters,
                           inner_steps, presteps, yb.size - 1, yb, C.byref(st))
    return Result(u, s, st.as_dict())


def timestep(deck, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
             presteps=PRESTEPS, mean_mode=0):
    """One implicit timestep from the deck's fields (u0 = rho*e)."""
    u = np.zeros((deck.ny, deck.nx))
    st = OraStats()
    s = lib().ora_timestep(deck.nx, deck.ny, deck.xmin, deck.xmax, deck.ymin, deck.ymax,
                           _c(deck.density), _c(deck.energy), deck.dt, method, eps,
                           max_iters, inner_steps, presteps, mean_mode, u, C.byref(st))
    return Result(u, s, st.as_dict())


def run(deck, steps=1, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
        presteps=PRESTEPS, mean_mode=0, ybounds=None):
    """`steps` implicit timesteps: u^{n+1} = A^{-1} u^n, u^0 = rho*e (reading R4).

    Returns (u, [stats per step], [status per step]).
    """
    rx, ry = mesh_r(deck)
    Kx, Ky = face_coefficients(deck.nx, deck.ny, rx, ry, deck.density, mean_mode)
    u = _c(deck.density) * _c(deck.energy)  # reading R4 (TeaLeaf): u = rho * e
    stats, statuses = [], []
    for _ in range(steps):
        res = solve(Kx, Ky, u, None, method, eps, max_iters, inner_steps, presteps, ybounds)
        u = res.u
        stats.append(res.stats)
        statuses.append(res.status)
    return u, stats, statuses


# --------------------------------------------------------------------------- 3D
def mesh_r3(deck):
    """rx, ry, rz = dt/dx^2, dt/dy^2, dt/dz^2."""
    dx = (deck.xmax - deck.xmin) / deck.nx
    dy = (deck.ymax - deck.ymin) / deck.ny
    dz = (deck.zmax - deck.zmin) / deck.nz
    return deck.dt / (dx * dx), deck.dt / (dy * dy), deck.dt / (dz * dz)


def face_coefficients3(nx, ny, nz, rx, ry, rz, rho, mean_mode=0):
    Kx = np.zeros((nz, ny, nx + 1))
    Ky = np.zeros((nz, ny + 1, nx))
    Kz = np.zeros((nz + 1, ny, nx))
    lib().ora_face_coefficients3(nx, ny, nz, rx, ry, rz, _c(rho), mean_mode, Kx, Ky, Kz)
    return Kx, Ky, Kz


def apply_A3(Kx, Ky, Kz, p):
    nz, ny, nx = p.shape
    w = np.zeros((nz, ny, nx))
    lib().ora_apply_A3(nx, ny, nz, _c(Kx), _c(Ky), _c(Kz), _c(p), w)
    return w


def solve3(Kx, Ky, Kz, u0, u_init=None, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
           presteps=PRESTEPS):
    nz, ny, nx = u0.shape
    u = _c(u0 if u_init is None else u_init).copy()
    st = OraStats()
    s = lib().ora_solve3(nx, ny, nz, _c(Kx), _c(Ky), _c(Kz), _c(u0), u, method, eps, max_iters,
                         inner_steps, presteps, C.byref(st))
    return Result(u, s, st.as_dict())


def run3(deck, steps=1, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
         presteps=PRESTEPS, mean_mode=0):
    rx, ry, rz = mesh_r3(deck)
    Kx, Ky, Kz = face_coefficients3(deck.nx, deck.ny, deck.nz, rx, ry, rz, deck.density,
                                    mean_mode)
    u = _c(deck.density) * _c(deck.energy)
    stats, statuses = [], []
    for _ in range(steps):
        res = solve3(Kx, Ky, Kz, u, None, method, eps, max_iters, inner_steps, presteps)
        u = res.u
        stats.append(res.stats)
        statuses.append(res.status)
    return u, stats, statuses
