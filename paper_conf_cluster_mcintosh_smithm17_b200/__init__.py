"""B200-native TeaLeaf CG / CPPCG hot path -- Python binding of the C ABI.

Argument marshalling only: every step of the solve runs in the CUDA kernels of
``libtea_b200.so`` (``include/tea.h``). PyTorch provides device memory (the
workspace tensor), the caller's CUDA stream and, for multi-GPU runs, the process
group used to broadcast the NCCL unique id. There is no CPU fallback: without
the CUDA library or a CUDA device every entry point raises.

Names follow the paper: ``solve(method=CG|CPPCG, eps, max_iters,
inner_steps)`` is one implicit timestep of Sec. II (L134-148) by CG (Sec. III.A)
or CPPCG (Sec. III.B-D); ``halo_depth`` is the matrix-powers depth of Sec. IV.C.2.
"""
from __future__ import annotations

import ctypes as C
import os
from dataclasses import dataclass

import numpy as np

from . import _build

CG, CPPCG, BJCG, CG1, JACOBI, CHEBY, CPPCG1, CPPCG1F = 0, 1, 2, 3, 4, 5, 6, 7
OK, NOT_CONVERGED = 0, 1
ERR_ARG, ERR_CUDA, ERR_NCCL, ERR_BREAKDOWN, ERR_STATE = -1, -2, -3, -4, -5
KERNELS = ["init", "residual", "spmv", "update", "cheb_first", "cheb_step", "cheb_last", "eig",
           "pack", "unpack", "scalar", "tb_first", "tb_mid", "tb_last", "bj", "cg1",
           "cg1_w", "stat", "persist"]
SYMBOLS = ["tea_version", "tea_abi_version", "tea_get_nccl_id", "tea_workspace_bytes", "tea_init",
           "tea_solve", "tea_fetch", "tea_set_u", "tea_kernel_times", "tea_launch_count",
           "tea_finalize", "tea_last_error", "tea_block_extent", "tea_cheb_schedule",
           "tea_halo_order", "tea_tb_plan", "tea_trace_read"]


class TeaError(RuntimeError):
    def __init__(self, status, msg):
        super().__init__(f"tea status {status}: {msg}")
        self.status = status


class Mesh(C.Structure):
    _fields_ = [("nx", C.c_int), ("ny", C.c_int), ("xmin", C.c_double), ("xmax", C.c_double),
                ("ymin", C.c_double), ("ymax", C.c_double), ("nz", C.c_int),
                ("zmin", C.c_double), ("zmax", C.c_double)]


ABI_VERSION = 5  # include/tea.h TEA_ABI_VERSION (tea_opts layout)


class Dist(C.Structure):
    _fields_ = [("rank", C.c_int), ("nranks", C.c_int), ("px", C.c_int), ("py", C.c_int),
                ("halo_depth", C.c_int), ("nccl_id", C.c_void_p)]


class Opts(C.Structure):
    _fields_ = [("presteps", C.c_int), ("eig_margin_lo", C.c_double),
                ("eig_margin_hi", C.c_double), ("mean_mode", C.c_int), ("loop_mode", C.c_int),
                ("check_interval", C.c_int), ("profile", C.c_int), ("tile_rows", C.c_int),
                ("tb_steps", C.c_int), ("tb_rows", C.c_int), ("persist", C.c_int),
                ("overlap", C.c_int), ("kform", C.c_int), ("trace", C.c_int)]


class Stats(C.Structure):
    _fields_ = [("iterations", C.c_int), ("presteps", C.c_int), ("outer", C.c_int),
                ("inner_matvecs", C.c_int), ("matvecs", C.c_int), ("status", C.c_int),
                ("r0", C.c_double), ("rnorm", C.c_double), ("eig_min", C.c_double),
                ("eig_max", C.c_double), ("ritz_min", C.c_double), ("ritz_max", C.c_double),
                ("seconds", C.c_double)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


_lib = None


def lib(build_if_needed: bool = True):
    """Load libtea_b200.so (building it with nvcc if it is missing or stale)."""
    global _lib
    if _lib is not None:
        return _lib
    path = os.environ.get("TEA_B200_LIB")  # experiments: an alternative build of the same ABI
    if path is None:
        if build_if_needed and _build.stale():
            _build.build()
        path = _build.LIB
    if not os.path.exists(path):
        raise ImportError(f"CUDA library {path} is missing; run __graft_entry__.build()")
    L = C.CDLL(path)
    vp, i, d = C.c_void_p, C.c_int, C.c_double
    L.tea_version.restype = C.c_char_p
    L.tea_abi_version.restype = i
    if L.tea_abi_version() != ABI_VERSION:
        raise ImportError(f"{path}: ABI version {L.tea_abi_version()} != {ABI_VERSION} "
                          "(stale build; run __graft_entry__.build())")
    L.tea_get_nccl_id.argtypes = [vp]
    L.tea_workspace_bytes.argtypes = [C.POINTER(Mesh), C.POINTER(Dist), C.POINTER(C.c_size_t)]
    L.tea_init.argtypes = [C.POINTER(vp), C.POINTER(Mesh), vp, vp, d, C.POINTER(Dist),
                           C.POINTER(Opts), vp, C.c_size_t, vp]
    L.tea_solve.argtypes = [vp, i, d, i, i, C.POINTER(Stats)]
    L.tea_fetch.argtypes = [vp, vp]
    L.tea_set_u.argtypes = [vp, vp]
    L.tea_kernel_times.argtypes = [vp, vp, vp, vp, i]
    L.tea_launch_count.argtypes = [vp]
    L.tea_launch_count.restype = C.c_longlong
    L.tea_finalize.argtypes = [vp]
    L.tea_last_error.argtypes = [vp]
    L.tea_last_error.restype = C.c_char_p
    L.tea_block_extent.argtypes = [C.POINTER(Mesh), i, i, i] + [C.POINTER(C.c_int)] * 4
    L.tea_cheb_schedule.argtypes = [i, i, vp, i]
    L.tea_halo_order.argtypes = [C.POINTER(Mesh), i, i, i, i, i, i, i, vp, i]
    L.tea_tb_plan.argtypes = [i, i, i, i, i]
    L.tea_trace_read.argtypes = [vp, i, vp, vp, vp, vp, i]
    _lib = L
    return L


def version() -> str:
    return lib().tea_version().decode()


def make_mesh(nx, ny, xmin=0.0, xmax=10.0, ymin=0.0, ymax=10.0, nz=1, zmin=0.0,
              zmax=1.0) -> Mesh:
    return Mesh(nx, ny, xmin, xmax, ymin, ymax, nz, zmin, zmax)


def mesh_of(deck) -> Mesh:
    """Mesh of a 2D Deck or a 3D Deck3 (inputs.py)."""
    nz = getattr(deck, "nz", 1)
    return Mesh(deck.nx, deck.ny, deck.xmin, deck.xmax, deck.ymin, deck.ymax, nz,
                getattr(deck, "zmin", 0.0), getattr(deck, "zmax", 1.0))


def workspace_bytes(mesh: Mesh, dist: Dist | None = None) -> int:
    n = C.c_size_t()
    st = lib().tea_workspace_bytes(C.byref(mesh), C.byref(dist) if dist else None, C.byref(n))
    if st != OK:
        raise TeaError(st, lib().tea_last_error(None).decode())
    return n.value


def get_nccl_id() -> bytes:
    buf = C.create_string_buffer(128)
    st = lib().tea_get_nccl_id(buf)
    if st != OK:
        raise TeaError(st, "ncclGetUniqueId failed")
    return buf.raw


def block_extent(mesh: Mesh, px: int, py: int, b: int):
    v = [C.c_int() for _ in range(4)]
    st = lib().tea_block_extent(C.byref(mesh), px, py, b, *[C.byref(x) for x in v])
    if st != OK:
        raise TeaError(st, "bad block")
    return tuple(x.value for x in v)


def cheb_schedule(s: int, d: int):
    buf = (C.c_int * 512)()
    n = lib().tea_cheb_schedule(s, d, buf, 256)
    if n < 0:
        raise TeaError(n, "bad schedule arguments")
    return [(buf[2 * i], buf[2 * i + 1]) for i in range(n)]


def tb_plan(levels: int, width: int, height: int, ctas_per_sm: int = 3, nsm: int = 148) -> int:
    """Rows per tile of a fused Chebyshev pass (the library's cost model, host-only)."""
    n = lib().tea_tb_plan(levels, width, height, ctas_per_sm, nsm)
    if n < 0:
        raise TeaError(n, "bad tb_plan arguments")
    return n


def halo_order(mesh: Mesh, px: int, py: int, nranks: int, rank: int, depth: int,
               corners: bool = True, nfields: int = 1):
    """Cross-process halo messages of `rank` in the order tea_solve posts them (host-only):
    [(op 0 send / 1 recv, peer, sending block, receiving block, direction, length)]."""
    n = lib().tea_halo_order(C.byref(mesh), px, py, nranks, rank, depth, int(corners), nfields,
                             None, 0)
    if n < 0:
        raise TeaError(n, "bad halo_order arguments")
    buf = (C.c_longlong * (6 * max(n, 1)))()
    lib().tea_halo_order(C.byref(mesh), px, py, nranks, rank, depth, int(corners), nfields,
                         buf, n)
    return [tuple(buf[6 * k:6 * k + 6]) for k in range(n)]


def _f64(a):
    a = np.ascontiguousarray(a, dtype=np.float64)
    return a, a.ctypes.data_as(C.c_void_p)


@dataclass
class SolveResult:
    status: int
    stats: dict


class Tea:
    """One TeaLeaf context: this rank's blocks of the mesh resident in HBM.

    density, energy: host float64 arrays of shape (ny, nx) (global mesh).
    dist: None (one block) or dict(rank, nranks, px, py, halo_depth[, nccl_id]).
    """

    def __init__(self, mesh: Mesh, density, energy, dt: float, dist: dict | None = None,
                 presteps: int = 30, eig_margins=(0.95, 1.05), mean_mode: int = 0,
                 loop_mode: int = 0, check_interval: int = 0, profile: bool = False,
                 tile_rows: int = 0, tb_steps: int = 0, tb_rows: int = 0, persist: int = 0,
                 overlap: int = 0, kform: int = 0, trace: bool = False, device=None,
                 stream=None):
        import torch
        if not torch.cuda.is_available():
            raise RuntimeError("paper_conf_cluster_mcintosh_smithm17_b200 needs a CUDA device "
                               "(no CPU fallback)")
        self._torch = torch
        self.L = lib()
        self.mesh = mesh
        self.device = torch.device(device) if device is not None else torch.device(
            "cuda", torch.cuda.current_device())
        self._dist = None
        self._nccl_id = None
        if dist is not None:
            nid = dist.get("nccl_id")
            if nid is not None:
                self._nccl_id = C.create_string_buffer(bytes(nid), 128)
            self._dist = Dist(dist.get("rank", 0), dist.get("nranks", 1), dist.get("px", 1),
                              dist.get("py", 1), dist.get("halo_depth", 1),
                              C.cast(self._nccl_id, C.c_void_p) if self._nccl_id else None)
        self.opts = Opts(presteps, eig_margins[0], eig_margins[1], mean_mode, loop_mode,
                         check_interval, 1 if profile else 0, tile_rows, tb_steps, tb_rows,
                         persist, overlap, kform, 1 if trace else 0)
        with torch.cuda.device(self.device):
            nbytes = workspace_bytes(mesh, self._dist)
            self.workspace = torch.empty(nbytes, dtype=torch.uint8, device=self.device)
            self.stream = stream if stream is not None else torch.cuda.current_stream(self.device)
            rho, prho = _f64(density)
            en, pen = _f64(energy)
            assert rho.size == mesh.nx * mesh.ny * max(mesh.nz, 1) and en.size == rho.size
            ctx = C.c_void_p()
            st = self.L.tea_init(C.byref(ctx), C.byref(mesh), prho, pen, float(dt),
                                 C.byref(self._dist) if self._dist else None, C.byref(self.opts),
                                 C.c_void_p(self.workspace.data_ptr()), nbytes,
                                 C.c_void_p(self.stream.cuda_stream))
            if st != OK:
                raise TeaError(st, self.L.tea_last_error(None).decode())
            self.ctx = ctx

    # -- one implicit timestep
    def solve(self, method=CG, eps=1e-10, max_iters=10000, inner_steps=10,
              raise_on_error=True) -> SolveResult:
        s = Stats()
        st = self.L.tea_solve(self.ctx, int(method), float(eps), int(max_iters),
                              int(inner_steps), C.byref(s))
        if st < 0 and raise_on_error:
            raise TeaError(st, self.L.tea_last_error(self.ctx).decode())
        return SolveResult(st, s.as_dict())

    def fetch(self, out=None):
        if out is None:
            shape = ((self.mesh.nz,) if self.mesh.nz > 1 else ()) + (self.mesh.ny, self.mesh.nx)
            out = np.zeros(shape)
        assert out.flags.c_contiguous and out.dtype == np.float64
        st = self.L.tea_fetch(self.ctx, out.ctypes.data_as(C.c_void_p))
        if st != OK:
            raise TeaError(st, self.L.tea_last_error(self.ctx).decode())
        return out

    def set_u(self, u):
        u, pu = _f64(u)
        st = self.L.tea_set_u(self.ctx, pu)
        if st != OK:
            raise TeaError(st, self.L.tea_last_error(self.ctx).decode())

    def kernel_times(self, reset=False):
        """{kernel class: (total ms, launches, algorithmic bytes)} in profile mode."""
        ms = (C.c_double * len(KERNELS))()
        n = (C.c_longlong * len(KERNELS))()
        by = (C.c_double * len(KERNELS))()
        self.L.tea_kernel_times(self.ctx, ms, n, by, 1 if reset else 0)
        return {k: (ms[i], n[i], by[i]) for i, k in enumerate(KERNELS)}

    def trace(self, reset=False):
        """In-graph kernel timing (trace=True): [(kernel class, algorithmic bytes per launch,
        launches, total ms)] -- device durations of the launches that did their work, taken
        inside whatever graphs / loop mode the solve ran in."""
        cap = 64
        kid = (C.c_int * cap)()
        by = (C.c_double * cap)()
        n = (C.c_longlong * cap)()
        ms = (C.c_double * cap)()
        k = self.L.tea_trace_read(self.ctx, cap, kid, by, n, ms, 1 if reset else 0)
        if k < 0:
            raise TeaError(k, self.L.tea_last_error(self.ctx).decode())
        return [(KERNELS[kid[i]], by[i], n[i], ms[i]) for i in range(min(k, cap))]

    def launch_count(self) -> int:
        return int(self.L.tea_launch_count(self.ctx))

    def close(self):
        if getattr(self, "ctx", None):
            self.L.tea_finalize(self.ctx)
            self.ctx = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


def run(deck, steps=1, method=CG, eps=1e-10, max_iters=10000, inner_steps=10, **kw):
    """Convenience: `steps` timesteps on one device; returns (u, [stats])."""
    t = Tea(mesh_of(deck), deck.density, deck.energy, deck.dt, **kw)
    stats = []
    try:
        for _ in range(steps):
            stats.append(t.solve(method, eps, max_iters, inner_steps).stats)
        return t.fetch(), stats
    finally:
        t.close()
