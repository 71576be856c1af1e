"""Seeded synthetic inputs shared by the CUDA path and the CPU oracle.

This module holds *data generation only*: it produces the cell-centred
density and energy fields and the mesh/timestep of a test deck. It contains
none of the method's arithmetic (no u = rho*e, no face coefficients, no
operator, no solver) so that the oracle (`oracle/`) and the CUDA library can
both consume its output without sharing any code of the method itself.

Workloads:

* ``crooked_pipe(n)`` -- the paper's test case, "a dense material of low heat
  conduction" crossed by "a crooked pipe of lower density material that has a
  higher heat conduction ... from one side of the problem domain to the other
  with a number of kinks" (Sec. V.B). The paper gives no
  numeric deck; the states below are the documented reading SURVEY.md §8(c)
  c12 (TeaLeaf ``tea_bm``-style): domain [0,10]^2, dt = 0.004, background
  rho = 100, e = 1e-4; pipe segments at rho = 0.1 (inlet e = 25, rest
  e = 0.1). A cell belongs to a rectangle when its centre lies in the
  half-open rectangle [x0,x1) x [y0,y1); later states override earlier ones.
* ``random_fields(nx, ny, seed)`` -- robustness/parity fields: rho
  log-uniform in [0.1, 100], e uniform in [1e-3, 25]
  (``numpy.random.default_rng(seed)``), SURVEY.md §8(d).
* ``uniform_fields(nx, ny, rho, seed)`` -- constant density (closed-form
  spectrum cases), random energy.

All arrays are float64, C-contiguous, shape (ny, nx): row k holds cells
j = 0..nx-1, i.e. global index k*nx + j ("x fastest"), the layout the C ABI
(`include/tea.h`) takes.
"""
from __future__ import annotations

from dataclasses import dataclass, field

import numpy as np

__all__ = ["Deck", "Deck3", "crooked_pipe", "random_fields", "uniform_fields", "deck",
           "crooked_pipe3", "random_fields3", "uniform_fields3"]


@dataclass
class Deck:
    """One synthetic problem: mesh extents, timestep and the two input fields."""

    nx: int
    ny: int
    xmin: float
    xmax: float
    ymin: float
    ymax: float
    dt: float
    density: np.ndarray = field(repr=False)
    energy: np.ndarray = field(repr=False)
    name: str = ""

    @property
    def shape(self):
        return (self.ny, self.nx)


# (x0, x1, y0, y1, rho, e) -- SURVEY.md §8(c) c12; later rows override.
PIPE_STATES = (
    (0.0, 1.0, 1.0, 2.0, 0.1, 25.0),   # inlet (hot)
    (1.0, 6.0, 1.0, 2.0, 0.1, 0.1),    # first leg
    (5.0, 6.0, 1.0, 8.0, 0.1, 0.1),    # kink: vertical leg
    (5.0, 10.0, 7.0, 8.0, 0.1, 0.1),   # outlet leg
)
PIPE_BACKGROUND = (100.0, 1.0e-4)
PIPE_DOMAIN = (0.0, 10.0, 0.0, 10.0)
PIPE_DT = 0.004


def crooked_pipe(nx: int, ny: int | None = None) -> Deck:
    """The crooked-pipe deck on an nx x ny mesh (default square)."""
    ny = nx if ny is None else ny
    xmin, xmax, ymin, ymax = PIPE_DOMAIN
    dx = (xmax - xmin) / nx
    dy = (ymax - ymin) / ny
    xc = xmin + (np.arange(nx) + 0.5) * dx
    yc = ymin + (np.arange(ny) + 0.5) * dy
    X, Y = np.meshgrid(xc, yc)  # shape (ny, nx)
    rho = np.full((ny, nx), PIPE_BACKGROUND[0])
    e = np.full((ny, nx), PIPE_BACKGROUND[1])
    for x0, x1, y0, y1, r, en in PIPE_STATES:
        m = (X >= x0) & (X < x1) & (Y >= y0) & (Y < y1)
        rho[m] = r
        e[m] = en
    return Deck(nx, ny, xmin, xmax, ymin, ymax, PIPE_DT,
                np.ascontiguousarray(rho), np.ascontiguousarray(e),
                name=f"crooked_pipe_{nx}x{ny}")


def random_fields(nx: int, ny: int, seed: int = 0, dt: float = 0.004,
                  extent: tuple = PIPE_DOMAIN) -> Deck:
    """rho log-uniform in [0.1, 100], e uniform in [1e-3, 25]; seeded."""
    rng = np.random.default_rng(seed)
    rho = np.exp(rng.uniform(np.log(0.1), np.log(100.0), size=(ny, nx)))
    e = rng.uniform(1.0e-3, 25.0, size=(ny, nx))
    xmin, xmax, ymin, ymax = extent
    return Deck(nx, ny, xmin, xmax, ymin, ymax, dt,
                np.ascontiguousarray(rho), np.ascontiguousarray(e),
                name=f"random_{nx}x{ny}_s{seed}")


def uniform_fields(nx: int, ny: int, rho: float = 1.0, seed: int = 0,
                   dt: float = 0.004, extent: tuple = PIPE_DOMAIN) -> Deck:
    """Constant density rho, energy uniform in [1e-3, 25]; seeded."""
    rng = np.random.default_rng(seed)
    e = rng.uniform(1.0e-3, 25.0, size=(ny, nx))
    xmin, xmax, ymin, ymax = extent
    return Deck(nx, ny, xmin, xmax, ymin, ymax, dt,
                np.full((ny, nx), float(rho)), np.ascontiguousarray(e),
                name=f"uniform_{nx}x{ny}_rho{rho}_s{seed}")


def deck(kind: str, nx: int, ny: int | None = None, seed: int = 0, **kw) -> Deck:
    """Dispatch by name: 'pipe', 'random', 'uniform'."""
    ny = nx if ny is None else ny
    if kind == "pipe":
        return crooked_pipe(nx, ny)
    if kind == "random":
        return random_fields(nx, ny, seed, **kw)
    if kind == "uniform":
        return uniform_fields(nx, ny, seed=seed, **kw)
    raise ValueError(f"unknown deck kind {kind!r}")


# ------------------------------------------------------------------ 3D
@dataclass
class Deck3:
    """A 3D problem: fields of shape (nz, ny, nx), index (l*ny + k)*nx + j."""

    nx: int
    ny: int
    nz: int
    xmin: float
    xmax: float
    ymin: float
    ymax: float
    zmin: float
    zmax: float
    dt: float
    density: np.ndarray = field(repr=False)
    energy: np.ndarray = field(repr=False)
    name: str = ""


def crooked_pipe3(nx: int, ny: int | None = None, nz: int | None = None) -> Deck3:
    """The 2D crooked-pipe states extruded along z over [0,10], plus a vertical leg
    [5,6)x[7,8)x[0,10) -> z in [2,10) connecting the outlet upward (reading R20: the
    paper gives no 3D deck; this keeps the pipe 'crooked' in all three directions)."""
    ny = nx if ny is None else ny
    nz = nx if nz is None else nz
    lo, hi = 0.0, 10.0
    xc = lo + (np.arange(nx) + 0.5) * (hi - lo) / nx
    yc = lo + (np.arange(ny) + 0.5) * (hi - lo) / ny
    zc = lo + (np.arange(nz) + 0.5) * (hi - lo) / nz
    Z, Y, X = np.meshgrid(zc, yc, xc, indexing="ij")
    rho = np.full((nz, ny, nx), PIPE_BACKGROUND[0])
    e = np.full((nz, ny, nx), PIPE_BACKGROUND[1])
    slab = (Z >= 0.0) & (Z < 2.0)
    for x0, x1, y0, y1, r, en in PIPE_STATES:
        m = (X >= x0) & (X < x1) & (Y >= y0) & (Y < y1) & slab
        rho[m] = r
        e[m] = en
    m = (X >= 5.0) & (X < 6.0) & (Y >= 7.0) & (Y < 8.0) & (Z >= 2.0) & (Z < 10.0)
    rho[m] = 0.1
    e[m] = 0.1
    return Deck3(nx, ny, nz, lo, hi, lo, hi, lo, hi, PIPE_DT, np.ascontiguousarray(rho),
                 np.ascontiguousarray(e), name=f"crooked_pipe3_{nx}x{ny}x{nz}")


def random_fields3(nx: int, ny: int, nz: int, seed: int = 0, dt: float = 0.004) -> Deck3:
    rng = np.random.default_rng(seed)
    rho = np.exp(rng.uniform(np.log(0.1), np.log(100.0), size=(nz, ny, nx)))
    e = rng.uniform(1.0e-3, 25.0, size=(nz, ny, nx))
    return Deck3(nx, ny, nz, 0.0, 10.0, 0.0, 10.0, 0.0, 10.0, dt, np.ascontiguousarray(rho),
                 np.ascontiguousarray(e), name=f"random3_{nx}x{ny}x{nz}_s{seed}")


def uniform_fields3(nx: int, ny: int, nz: int, rho: float = 1.0, seed: int = 0,
                    dt: float = 0.004, extent=(0.0, 10.0, 0.0, 10.0, 0.0, 10.0)) -> Deck3:
    rng = np.random.default_rng(seed)
    e = rng.uniform(1.0e-3, 25.0, size=(nz, ny, nx))
    return Deck3(nx, ny, nz, *extent, dt, np.full((nz, ny, nx), float(rho)),
                 np.ascontiguousarray(e), name=f"uniform3_{nx}x{ny}x{nz}")
