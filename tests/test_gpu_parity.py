"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle.

Bar (BASELINE.json north_star): max relative field error <= 1e-10 in fp64 and
iteration counts within +-2 of the oracle on the same generated inputs. The
field is positive (u >= 0.01 on the pipe; > 0 on the random decks), so the
pointwise relative error max|u_gpu - u_ora| / |u_ora| is well defined.

Sizes: small cases the oracle runs on the spot (several 256-column CTA tiles,
ragged tails in x and y, 1-wide meshes, odd sizes); full-size cases (1024^2
converged, 4096^2 fixed iteration counts) against tests/golden/oracle_*.npz,
written by tests/golden/make_golden.py from the oracle alone, compared at the
stored sample of cells plus sum/min/max.
"""
import os

import numpy as np
import pytest

pytestmark = pytest.mark.gpu

HERE = os.path.dirname(os.path.abspath(__file__))


@pytest.fixture(scope="module")
def tea():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    tea.lib()
    return tea


def rel_err(a, b):
    """Pointwise relative error (the north_star metric; the pipe has u >= 0.01)."""
    return float(np.max(np.abs(a - b) / np.abs(b)))


def field_err(a, b, kind):
    """The north_star metric on every deck: max pointwise relative error (u > 0 on the pipe
    and on the random decks; measured on the random decks: <= 3e-12 where the pipe gives
    ~1e-13, profiles/r02_random_metric.txt). `kind` is kept for the call sites."""
    return rel_err(a, b)


def iter_err(a, b, kind):
    """Fixed-iteration (mid-solve) iterates: pointwise on the pipe; on the random decks
    normwise max|du| / max|u|. A mid-solve iterate u_0 + sum_k alpha_k p_k is a sum of terms
    of size max|u|, and the two sides round each term differently (R13): a cell whose value
    is a small remnant of cancelling terms carries an absolute error of O(eps max|u|), not
    O(eps |u_i|) (measured on the 1000 x 777 random deck after 2 CG iterations: 1.6e-10
    pointwise, 2e-14 normwise). Converged fields are compared pointwise (field_err) and the
    fixed-iteration random cases also against the rigorous bound of reading R22."""
    if kind == "pipe":
        return rel_err(a, b)
    return float(np.max(np.abs(a - b)) / np.max(np.abs(b)))


def residual_bound(ora, deck, *fields):
    """Sum of the TRUE residual norms ||u^n - A u||_2 of the given fields (oracle operator).
    lambda_min(A) >= 1 (A = I + dt L, L positive semidefinite: pinned in
    tests/test_oracle_operator.py), so ||u - u*||_2 <= ||u^n - A u||_2 for ANY field u, and
    two fields differ by at most the sum at every cell (reading R22)."""
    rx, ry = ora.mesh_r(deck)
    Kx, Ky = ora.face_coefficients(deck.nx, deck.ny, rx, ry, deck.density)
    u0 = deck.density * deck.energy
    return sum(float(np.linalg.norm(u0 - ora.apply_A(Kx, Ky, u))) for u in fields)


def gpu_run(tea, deck, steps=1, **kw):
    solve_kw = {k: kw.pop(k) for k in ("method", "eps", "max_iters", "inner_steps") if k in kw}
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, **kw)
    stats = []
    for _ in range(steps):
        r = t.solve(**solve_kw)
        stats.append(dict(r.stats, ret=r.status))
    u = t.fetch()
    t.close()
    return u, stats


def deck_of(kind, nx, ny, seed=0, dt=0.004):
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    if kind == "pipe":
        return inputs.crooked_pipe(nx, ny)
    return inputs.random_fields(nx, ny, seed, dt=dt)


SHAPES = [("pipe", 128, 128), ("random", 300, 200), ("random", 1000, 777), ("random", 257, 65),
          ("random", 1, 97), ("random", 95, 1), ("random", 3, 5), ("random", 64, 64)]


@pytest.mark.parametrize("kind,nx,ny", SHAPES)
@pytest.mark.parametrize("k", [1, 2, 7])
@pytest.mark.parametrize("persist", [0, -1])
def test_fixed_cg_iterations(tea, ora, kind, nx, ny, k, persist):
    """k CG iterations with eps = 0: exercises residual, spmv (+ lazy u update),
    update and the finalize path on ragged shapes (persist 0: the auto choice -- the
    persistent solver at these sizes; -1: the graph path)."""
    deck = deck_of(kind, nx, ny, seed=nx + ny, dt=0.04)
    u_o, st_o, _ = ora.run(deck, steps=1, method=0, eps=0.0, max_iters=k)
    u_g, st_g = gpu_run(tea, deck, method=0, eps=0.0, max_iters=k, persist=persist)
    assert st_g[0]["iterations"] == st_o[0]["iterations"] == k
    assert st_g[0]["ret"] == 1  # TEA_NOT_CONVERGED
    assert iter_err(u_g, u_o, kind) <= 1e-12
    assert float(np.max(np.abs(u_g - u_o))) <= residual_bound(ora, deck, u_g, u_o)
    assert st_g[0]["r0"] == pytest.approx(st_o[0]["r0"], rel=1e-12)


@pytest.mark.parametrize("kind,nx,ny", SHAPES[:5])
@pytest.mark.parametrize("method", [0, 1])
@pytest.mark.parametrize("persist", [0, -1])
def test_converged_solve(tea, ora, kind, nx, ny, method, persist):
    # dt = 0.004 (the deck's): kappa ~ 1e3-1e4. At kappa ~ 1e6 (dt = 0.4, 3700 CG
    # iterations) CG's finite-precision iteration count drifts by ~10 between any two
    # summation orders, so +-2 is not a meaningful bar there.
    deck = deck_of(kind, nx, ny, seed=3, dt=0.004)
    kw = dict(method=method, eps=1e-13, max_iters=20000, inner_steps=6)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, persist=persist, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, kind) <= 1e-10
    if method == 1 and st_o[0]["outer"] > 0:
        assert st_g[0]["presteps"] == st_o[0]["presteps"]
        assert st_g[0]["eig_min"] == pytest.approx(st_o[0]["eig_min"], rel=1e-9)
        assert st_g[0]["eig_max"] == pytest.approx(st_o[0]["eig_max"], rel=1e-9)


def test_config1_pipe128_cg_10_steps(tea, ora):
    """BASELINE.json configs[0]: 128x128, CG, fp64, 10 timesteps, eps = 1e-15 (graph path;
    the persistent solver: test_persist_config1_10_steps)."""
    deck = deck_of("pipe", 128, 128)
    kw = dict(method=0, eps=1e-15, max_iters=10000)
    u_o, st_o, _ = ora.run(deck, steps=10, **kw)
    u_g, st_g = gpu_run(tea, deck, steps=10, persist=-1, **kw)
    for a, b in zip(st_g, st_o):
        assert abs(a["iterations"] - b["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("s", [1, 2, 3, 10])
def test_cppcg_inner_steps(tea, ora, s):
    deck = deck_of("pipe", 256, 256)
    kw = dict(method=1, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert abs(st_g[0]["outer"] - st_o[0]["outer"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("loop_mode", [0, 1, 2])
def test_loop_modes_identical(tea, loop_mode):
    """WHILE graph, chunked graphs and eager launches run the same kernels with the
    same launch geometry: bitwise identical results (deterministic reductions)."""
    deck = deck_of("pipe", 200, 136)
    ref, st_ref = gpu_run(tea, deck, method=1, eps=1e-12, max_iters=5000, inner_steps=5,
                          loop_mode=2)
    u, st = gpu_run(tea, deck, method=1, eps=1e-12, max_iters=5000, inner_steps=5,
                    loop_mode=loop_mode, check_interval=6)
    assert st[0]["iterations"] == st_ref[0]["iterations"]
    assert np.array_equal(u, ref)


def test_run_to_run_bitwise(tea):
    deck = deck_of("random", 333, 222, seed=5)
    a, _ = gpu_run(tea, deck, method=0, eps=1e-12, max_iters=3000)
    b, _ = gpu_run(tea, deck, method=0, eps=1e-12, max_iters=3000)
    assert np.array_equal(a, b)


def test_conservation_and_max_principle(tea):
    deck = deck_of("pipe", 512, 512)
    u0 = deck.density * deck.energy
    for method in (0, 1):
        u, st = gpu_run(tea, deck, method=method, eps=1e-12, max_iters=20000)
        assert abs(u.sum() - u0.sum()) / u0.sum() <= 1e-12
        assert u.min() >= u0.min() * (1 - 1e-12) and u.max() <= u0.max() * (1 + 1e-12)


def test_checkpoint_resume_bitwise(tea):
    """N steps == k steps, fetch, re-init with e = u/rho, N-k steps."""
    deck = deck_of("pipe", 128, 96)
    full, _ = gpu_run(tea, deck, steps=4, method=0, eps=1e-14, max_iters=5000)
    half, _ = gpu_run(tea, deck, steps=2, method=0, eps=1e-14, max_iters=5000)
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt)
    t.set_u(half)
    for _ in range(2):
        t.solve(method=0, eps=1e-14, max_iters=5000)
    resumed = t.fetch()
    t.close()
    assert np.array_equal(resumed, full)


def test_errors(tea):
    deck = deck_of("random", 16, 16)
    m = tea.mesh_of(deck)
    with pytest.raises(tea.TeaError):
        tea.Tea(m, deck.density, deck.energy, deck.dt, dist=dict(px=3, py=1, nranks=2))
    with pytest.raises(tea.TeaError):
        tea.Tea(m, deck.density, deck.energy, deck.dt, dist=dict(px=1, py=1, halo_depth=17))
    bad = deck.density.copy()
    bad[0, 0] = 0.0
    with pytest.raises(tea.TeaError):
        tea.Tea(m, bad, deck.energy, deck.dt)
    t = tea.Tea(m, deck.density, deck.energy, deck.dt)
    r = t.solve(method=1, inner_steps=0, raise_on_error=False)
    assert r.status == tea.ERR_ARG
    r = t.solve(method=0, eps=1e-10, max_iters=1000)  # still usable after ERR_ARG
    assert r.status == tea.OK
    t.close()


def test_zero_residual(tea):
    deck = deck_of("random", 40, 30)
    deck.dt = 0.0  # A = I: r0 == 0, zero iterations
    u, st = gpu_run(tea, deck, method=1, eps=1e-10, max_iters=100)
    assert st[0]["iterations"] == 0 and st[0]["ret"] == 0
    assert np.array_equal(u, deck.density * deck.energy)


# ---------------------------------------------------------------- full sizes
def load_golden(name):
    p = os.path.join(HERE, "golden", f"oracle_{name}.npz")
    if not os.path.exists(p):
        pytest.skip(f"{p} missing (run tests/golden/make_golden.py)")
    return dict(np.load(p))


@pytest.mark.parametrize("name", ["pipe1024_cg", "pipe1024_cppcg", "pipe4096_cg_fixed50",
                                  "pipe4096_cppcg_fixed33"])
def test_full_size_against_golden(tea, name):
    g = load_golden(name)
    n = int(g["n"])
    deck = deck_of("pipe", n, n)
    u, st = gpu_run(tea, deck, method=int(g["method"]), eps=float(g["eps"]),
                    max_iters=int(g["max_iters"]), inner_steps=int(g["inner_steps"]))
    assert abs(st[0]["iterations"] - int(g["iterations"])) <= 2
    if int(g["method"]) == 1:
        assert st[0]["presteps"] == int(g["presteps"])
        assert st[0]["eig_max"] == pytest.approx(float(g["eig_max"]), rel=1e-9)
    vals = u.ravel()[g["idx"]]
    assert rel_err(vals, g["vals"]) <= 1e-10
    assert u.sum() == pytest.approx(float(g["sum"]), rel=1e-12)
    assert u.min() == pytest.approx(float(g["umin"]), rel=1e-10)
    assert u.max() == pytest.approx(float(g["umax"]), rel=1e-10)


# ---------------------------------------------------------------- decomposition
# px x py blocks in ONE process on one GPU (nranks = 1): the multi-GPU code path
# (extended bounds, matrix-powers schedule, pack / unpack of depth-d halos with
# corners, cross-block reductions) with device copies as the halo transport.
@pytest.mark.parametrize("px,py,d", [(2, 1, 1), (1, 2, 1), (2, 2, 2), (3, 2, 3), (4, 2, 5),
                                     (2, 3, 10), (4, 4, 16)])
@pytest.mark.parametrize("method", [0, 1])
def test_multiblock_matches_oracle(tea, ora, px, py, d, method):
    deck = deck_of("pipe", 200, 168)
    kw = dict(method=method, eps=1e-13, max_iters=20000, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=d, nranks=1), **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("px,py,d", [(2, 2, 1), (3, 3, 4), (2, 1, 7)])
def test_multiblock_fixed_iterations(tea, ora, px, py, d):
    """eps = 0 and a fixed iteration count: field agrees to rounding (1e-12)."""
    deck = deck_of("random", 150, 121, seed=9, dt=0.04)
    for method, k in ((0, 9), (1, 33)):
        u_o, st_o, _ = ora.run(deck, steps=1, method=method, eps=0.0, max_iters=k,
                               inner_steps=6)
        u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=d, nranks=1),
                            method=method, eps=0.0, max_iters=k, inner_steps=6)
        assert st_g[0]["iterations"] == k
        assert iter_err(u_g, u_o, "random") <= 1e-12
        # the reported residual norm is the global one (reductions are not replayed after
        # the solve ends)
        assert st_g[0]["rnorm"] == pytest.approx(st_o[0]["rnorm"], rel=1e-9)


# ---------------------------------------------------------------- fused passes
# Temporally blocked Chebyshev passes (tea_cheb_tb.cu, on-chip matrix powers): M steps
# per kernel; tb_steps = 1 is the one-kernel-per-step path.
@pytest.mark.parametrize("tb", [1, 2, 3, 4, 5])
@pytest.mark.parametrize("s", [1, 2, 3, 5, 10, 13])
def test_fused_passes_converged(tea, ora, tb, s):
    deck = deck_of("pipe", 256, 200)
    kw = dict(method=1, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("kind,nx,ny", [("random", 300, 200), ("random", 257, 65),
                                        ("random", 1, 97), ("random", 95, 1),
                                        ("random", 3, 5), ("pipe", 128, 128)])
@pytest.mark.parametrize("tb", [2, 4, 5])
def test_fused_passes_fixed_iterations(tea, ora, kind, nx, ny, tb):
    """30 presteps + 3 outer iterations, eps = 0, on ragged shapes: the fused passes
    agree with the one-kernel-per-step path to rounding (1e-12), and with the oracle
    to 1e-12 on 2D meshes. On the 1-cell-wide random meshes A has an eigenvalue 1.0006
    next to its exact lambda_min = 1 (a nearly insulated stretch of the random density),
    below the estimated Chebyshev interval [1.08, 58]: the mid-solve iterates carry
    rounding-driven components in that near-null pair that the oracle's Saad-form and the
    GPU's three-term preconditioner round differently (measured 3e-8 / 7e-8 pointwise after
    one outer iteration, 3e-15 at convergence: profiles/r02_random_metric.txt). There the
    oracle comparison is the rigorous computed bound of reading R22 -- every cell within
    the sum of the two true residual norms -- and the converged tests give the 1e-10 bar."""
    deck = deck_of(kind, nx, ny, seed=4, dt=0.04)
    kw = dict(method=1, eps=0.0, max_iters=33, inner_steps=7)
    u_1, st_1 = gpu_run(tea, deck, tb_steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert st_g[0]["iterations"] == st_1[0]["iterations"] == 33
    assert iter_err(u_g, u_1, "random") <= 1e-12
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    if min(nx, ny) > 1:
        assert iter_err(u_g, u_o, kind) <= 1e-12
    else:
        # (the residual norms themselves differ by up to 13% at this point)
        assert float(np.max(np.abs(u_g - u_o))) <= residual_bound(ora, deck, u_g, u_o)
    kw = dict(method=1, eps=1e-13, max_iters=5000, inner_steps=7)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_c, st_c = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert abs(st_c[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_c, u_o, kind) <= 1e-10


@pytest.mark.parametrize("tb_rows", [16, 32, 64, 128])
def test_fused_pass_tile_heights(tea, ora, tb_rows):
    deck = deck_of("pipe", 384, 300)
    kw = dict(method=1, eps=1e-12, max_iters=20000, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=4, tb_rows=tb_rows, **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


# ---------------------------------------------------------------- block Jacobi (NEXT-1)
def ybounds_of(tea, deck, px, py):
    m = tea.mesh_of(deck)
    return [tea.block_extent(m, px, py, bj * px)[2] for bj in range(py)] + [deck.ny]


@pytest.mark.parametrize("kind,nx,ny", [("pipe", 128, 128), ("pipe", 256, 200),
                                        ("random", 300, 203), ("random", 257, 65),
                                        ("random", 1, 97), ("random", 95, 1), ("random", 3, 5)])
def test_bjcg_converged(tea, ora, kind, nx, ny):
    deck = deck_of(kind, nx, ny, seed=6)
    kw = dict(method=2, eps=1e-13, max_iters=20000)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, kind) <= 1e-10


@pytest.mark.parametrize("kind,nx,ny,k", [("random", 300, 203, 5), ("pipe", 130, 97, 12),
                                          ("random", 64, 7, 3)])
def test_bjcg_fixed_iterations(tea, ora, kind, nx, ny, k):
    deck = deck_of(kind, nx, ny, seed=8, dt=0.04)
    kw = dict(method=2, eps=0.0, max_iters=k)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert st_g[0]["iterations"] == k
    assert iter_err(u_g, u_o, kind) <= 1e-12


@pytest.mark.parametrize("px,py", [(2, 1), (1, 3), (3, 2), (2, 4)])
def test_bjcg_multiblock(tea, ora, px, py):
    """Strips are truncated at block-row boundaries: the oracle gets the
    same boundaries (ybounds)."""
    deck = deck_of("pipe", 200, 170)
    yb = ybounds_of(tea, deck, px, py)
    kw = dict(method=2, eps=1e-13, max_iters=20000)
    u_o, st_o, _ = ora.run(deck, steps=1, ybounds=yb, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=1, nranks=1), **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


# ---------------------------------------------------------------- single-reduction CG (NEXT-2)
@pytest.mark.parametrize("kind,nx,ny", [("pipe", 128, 128), ("pipe", 256, 200),
                                        ("random", 300, 203), ("random", 1, 97),
                                        ("random", 95, 1), ("random", 3, 5)])
def test_cg1_converged(tea, ora, kind, nx, ny):
    deck = deck_of(kind, nx, ny, seed=6)
    kw = dict(method=3, eps=1e-13, max_iters=20000)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, kind) <= 1e-10


@pytest.mark.parametrize("k", [1, 2, 9])
def test_cg1_fixed_iterations(tea, ora, k):
    deck = deck_of("random", 300, 203, seed=8, dt=0.04)
    kw = dict(method=3, eps=0.0, max_iters=k)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert st_g[0]["iterations"] == k
    assert iter_err(u_g, u_o, "random") <= 1e-12


@pytest.mark.parametrize("px,py", [(2, 1), (1, 3), (2, 2), (4, 2)])
def test_cg1_multiblock(tea, ora, px, py):
    deck = deck_of("pipe", 200, 170)
    kw = dict(method=3, eps=1e-13, max_iters=20000)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=1, nranks=1), **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


# ---------------------------------------------------------------- single-reduction CPPCG
@pytest.mark.parametrize("kind,nx,ny,s,tb", [("pipe", 128, 128, 10, 0), ("pipe", 256, 200, 10, 5),
                                             ("pipe", 256, 200, 10, 1), ("random", 300, 203, 4, 0),
                                             ("random", 97, 61, 3, 0), ("random", 1000, 777, 10, 0)])
def test_cppcg1_converged(tea, ora, kind, nx, ny, s, tb):
    """Single-reduction CPPCG (TEA_CPPCG1): converged solve against the oracle (+-2 outer
    iterations, 1e-10), with the fused passes (tb 5, and auto at 1000 x 777) and with one
    kernel per step (tb 1)."""
    deck = deck_of(kind, nx, ny, seed=6)
    kw = dict(method=6, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert st_g[0]["presteps"] == st_o[0]["presteps"]
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert st_g[0]["matvecs"] == 1 + st_g[0]["iterations"] + s * (st_g[0]["outer"] + 1) + 1
    assert field_err(u_g, u_o, kind) <= 1e-10
    # same solution as CPPCG on the GPU, one reduction per outer iteration instead of two
    u_c, st_c = gpu_run(tea, deck, tb_steps=tb, **dict(kw, method=1))
    assert abs(st_c[0]["outer"] - st_g[0]["outer"]) <= 2
    assert rel_err(u_g, u_c) <= 1e-10


@pytest.mark.parametrize("k", [1, 2, 7])
@pytest.mark.parametrize("tb", [1, 5])
def test_cppcg1_fixed_iterations(tea, ora, k, tb):
    deck = deck_of("random", 300, 203, seed=8, dt=0.04)
    kw = dict(method=6, eps=0.0, max_iters=30 + k, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert st_g[0]["iterations"] == 30 + k and st_g[0]["outer"] == k
    assert iter_err(u_g, u_o, "random") <= 1e-12
    assert st_g[0]["rnorm"] == pytest.approx(st_o[0]["rnorm"], rel=1e-9)


@pytest.mark.parametrize("px,py,d,tb", [(2, 1, 11, 5), (2, 2, 11, 5), (1, 3, 2, 0), (4, 2, 4, 0)])
@pytest.mark.parametrize("loop_mode", [0, 2])
def test_cppcg1_multiblock(tea, ora, px, py, d, tb, loop_mode):
    deck = deck_of("pipe", 200, 170)
    kw = dict(method=6, eps=1e-13, max_iters=20000, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=d, nranks=1), tb_steps=tb,
                        loop_mode=loop_mode, **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("method", [2, 3, 6])
@pytest.mark.parametrize("loop_mode", [1, 2])
def test_new_methods_loop_modes_identical(tea, method, loop_mode):
    deck = deck_of("pipe", 200, 136)
    ref, st_ref = gpu_run(tea, deck, method=method, eps=1e-12, max_iters=5000)
    u, st = gpu_run(tea, deck, method=method, eps=1e-12, max_iters=5000, loop_mode=loop_mode,
                    check_interval=6)
    assert st[0]["iterations"] == st_ref[0]["iterations"]
    assert np.array_equal(u, ref)


# ---------------------------------------------------------------- Jacobi / Chebyshev (NEXT-4)
@pytest.mark.parametrize("method", [4, 5])
@pytest.mark.parametrize("kind,nx,ny", [("pipe", 64, 64), ("random", 130, 97), ("random", 1, 40),
                                        ("random", 33, 1)])
def test_stationary_converged(tea, ora, method, kind, nx, ny):
    deck = deck_of(kind, nx, ny, seed=2, dt=0.004)
    kw = dict(method=method, eps=1e-12, max_iters=200000)
    u_o, st_o, s_o = ora.run(deck, steps=1, presteps=10, **kw)
    u_g, st_g = gpu_run(tea, deck, presteps=10, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, kind) <= 1e-10


@pytest.mark.parametrize("method,k", [(4, 1), (4, 2), (4, 7), (5, 11), (5, 12), (5, 20)])
def test_stationary_fixed_iterations(tea, ora, method, k):
    deck = deck_of("random", 200, 150, seed=3, dt=0.04)
    kw = dict(method=method, eps=0.0, max_iters=k)
    u_o, st_o, _ = ora.run(deck, steps=1, presteps=10, **kw)
    u_g, st_g = gpu_run(tea, deck, presteps=10, **kw)
    assert st_g[0]["iterations"] == k
    assert iter_err(u_g, u_o, "random") <= 1e-12


@pytest.mark.parametrize("method", [4, 5])
@pytest.mark.parametrize("px,py", [(2, 1), (2, 3)])
def test_stationary_multiblock(tea, ora, method, px, py):
    deck = deck_of("pipe", 96, 72)
    kw = dict(method=method, eps=1e-12, max_iters=200000)
    u_o, st_o, _ = ora.run(deck, steps=1, presteps=10, **kw)
    u_g, st_g = gpu_run(tea, deck, presteps=10, dist=dict(px=px, py=py, halo_depth=1, nranks=1),
                        **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


# ---------------------------------------------------------------- 3D (NEXT-4)
def deck3_of(kind, nx, ny, nz, seed=0, dt=0.004):
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    if kind == "pipe":
        return inputs.crooked_pipe3(nx, ny, nz)
    return inputs.random_fields3(nx, ny, nz, seed, dt=dt)


@pytest.mark.parametrize("method", [0, 1, 3, 4, 5, 6, 7])
@pytest.mark.parametrize("kind,nx,ny,nz", [("pipe", 40, 36, 28), ("random", 33, 17, 9),
                                           ("random", 70, 5, 2)])
def test_3d_converged(tea, ora, method, kind, nx, ny, nz):
    deck = deck3_of(kind, nx, ny, nz, seed=1)
    kw = dict(method=method, eps=1e-12, max_iters=200000, inner_steps=6)
    u_o, st_o, s_o = ora.run3(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, kind) <= 1e-10


@pytest.mark.parametrize("method,k", [(0, 3), (1, 33), (3, 4), (4, 5), (5, 35), (6, 33), (7, 33)])
def test_3d_fixed_iterations(tea, ora, method, k):
    deck = deck3_of("random", 45, 23, 11, seed=2, dt=0.04)
    kw = dict(method=method, eps=0.0, max_iters=k, inner_steps=5)
    u_o, st_o, _ = ora.run3(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, **kw)
    assert st_g[0]["iterations"] == k
    assert iter_err(u_g, u_o, "random") <= 1e-12


def test_3d_rejections(tea):
    deck = deck3_of("random", 16, 16, 8)
    with pytest.raises(tea.TeaError):
        tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt,
                dist=dict(px=2, py=1, nranks=1))
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt)
    assert t.solve(method=2, raise_on_error=False).status == tea.ERR_ARG  # block Jacobi: 2D
    t.close()


@pytest.mark.parametrize("loop_mode", [1, 2])
def test_loop_modes_identical_fused_passes(tea, loop_mode):
    """The WHILE graph, chunked graphs and eager launches agree bitwise on a mesh large
    enough for the fused Chebyshev passes (>= 2M cells)."""
    deck = deck_of("pipe", 2048, 1100)
    kw = dict(method=1, eps=1e-10, max_iters=2000, inner_steps=10)
    ref, st_ref = gpu_run(tea, deck, loop_mode=0, **kw)
    u, st = gpu_run(tea, deck, loop_mode=loop_mode, check_interval=6, **kw)
    assert st[0]["iterations"] == st_ref[0]["iterations"]
    assert np.array_equal(u, ref)


# ---------------------------------------------------------------- sanitizers
@pytest.mark.parametrize("tool", ["memcheck", "racecheck"])
def test_compute_sanitizer(tea, tool):
    """compute-sanitizer over small solves of every path (tools/sanitize.py): no memory
    errors, no shared-memory races (the fused passes' delay lines, the grid reductions)."""
    import shutil
    import subprocess
    import sys
    # opt-in: the GPU pool closed compute-sanitizer in round 2 (runs under it had left GPUs
    # needing a reset); the committed reports are under profiles/sanitizers/
    if os.environ.get("TEA_RUN_SANITIZER") != "1":
        pytest.skip("compute-sanitizer runs are opt-in (TEA_RUN_SANITIZER=1)")
    exe = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
    if not os.path.exists(exe):
        pytest.skip("compute-sanitizer not found")
    root = os.path.dirname(HERE)
    out = subprocess.run([exe, "--tool", tool, "--error-exitcode", "9", sys.executable,
                          os.path.join(root, "tools", "sanitize.py")], capture_output=True,
                         text=True, timeout=900, cwd=root)
    if "closed on this pool" in out.stdout + out.stderr:
        pytest.skip("compute-sanitizer is closed on this GPU pool")
    assert out.returncode == 0, out.stdout[-3000:] + out.stderr[-3000:]
    assert "0 errors" in out.stdout or "0 hazards" in out.stdout


# ---------------------------------------------------------------- fused passes on blocks
@pytest.mark.parametrize("px,py,d,s,tb", [(2, 2, 11, 10, 5), (3, 2, 12, 10, 4), (2, 1, 16, 10, 5),
                                          (1, 3, 6, 5, 3), (4, 2, 4, 3, 2), (2, 2, 11, 10, 1)])
def test_fused_passes_on_extended_bounds(tea, ora, px, py, d, s, tb):
    """Matrix powers on chip across blocks: one depth-d exchange of r per
    outer iteration, fused passes on bounds extended by 1 + (steps after the pass)."""
    deck = deck_of("pipe", 240, 200)
    kw = dict(method=1, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=d, nranks=1),
                        tb_steps=tb, **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10
    u_1, _ = gpu_run(tea, deck, tb_steps=tb, **kw)
    assert rel_err(u_g, u_1) <= 1e-10


def test_fused_passes_blocks_fixed_iterations(tea, ora):
    deck = deck_of("random", 200, 150, seed=12, dt=0.04)
    kw = dict(method=1, eps=0.0, max_iters=34, inner_steps=10)
    u_o, _, _ = ora.run(deck, steps=1, **kw)
    u_g, st = gpu_run(tea, deck, dist=dict(px=3, py=2, halo_depth=11, nranks=1), tb_steps=5,
                      **kw)
    assert st[0]["iterations"] == 34
    assert iter_err(u_g, u_o, "random") <= 1e-12


@pytest.mark.parametrize("nx,ny,px,py,d,s,tb", [(240, 200, 2, 2, 11, 10, 5),
                                                (201, 143, 3, 2, 12, 10, 4),
                                                (150, 90, 1, 3, 6, 5, 3),
                                                (36, 24, 3, 2, 11, 10, 5)])
@pytest.mark.parametrize("loop_mode", [0, 1, 2])
def test_overlap_bitwise(tea, nx, ny, px, py, d, s, tb, loop_mode):
    """Halo/compute overlap (tea_opts.overlap): the first fused pass split
    into the halo-free interior (concurrent with the exchange on the second stream) and the
    frame after it gives bitwise the same fields and scalars as the unsplit pass, down to
    the smallest legal blocks (12 x 12 at d = 11: a 2 x 2 interior)."""
    deck = deck_of("random", nx, ny, seed=nx * ny, dt=0.04)
    kw = dict(method=1, eps=0.0, max_iters=30 + 6, inner_steps=s, tb_steps=tb,
              loop_mode=loop_mode, dist=dict(px=px, py=py, halo_depth=d, nranks=1))
    u_a, st_a = gpu_run(tea, deck, overlap=1, **kw)
    u_b, st_b = gpu_run(tea, deck, overlap=-1, **kw)
    assert st_a[0]["iterations"] == st_b[0]["iterations"] == 36
    assert np.array_equal(u_a, u_b)
    assert st_a[0]["rnorm"] == st_b[0]["rnorm"]


def test_overlap_converged_against_oracle(tea, ora):
    deck = deck_of("pipe", 256, 192)
    kw = dict(method=1, eps=1e-13, max_iters=20000, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=2, **kw)
    u_g, st_g = gpu_run(tea, deck, steps=2, dist=dict(px=2, py=2, halo_depth=11, nranks=1),
                        tb_steps=5, overlap=1, **kw)
    for a, b in zip(st_g, st_o):
        assert a["ret"] == 0 and abs(a["iterations"] - b["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


# ---------------------------------------------------------------- persistent solver
# tea_opts.persist = 1: the whole solve in ONE cooperative launch (k_persist, grid-wide
# barriers between the phases). Same device bodies as the graph path.
@pytest.mark.parametrize("kind,nx,ny", SHAPES[:7])
@pytest.mark.parametrize("k", [1, 7])
def test_persist_fixed_cg_iterations(tea, ora, kind, nx, ny, k):
    deck = deck_of(kind, nx, ny, seed=nx + ny, dt=0.04)
    u_o, st_o, _ = ora.run(deck, steps=1, method=0, eps=0.0, max_iters=k)
    u_g, st_g = gpu_run(tea, deck, method=0, eps=0.0, max_iters=k, persist=1)
    assert st_g[0]["iterations"] == st_o[0]["iterations"] == k
    assert st_g[0]["ret"] == 1
    assert iter_err(u_g, u_o, kind) <= 1e-12


@pytest.mark.parametrize("kind,nx,ny", [("pipe", 128, 128), ("random", 300, 200),
                                        ("random", 257, 65)])
@pytest.mark.parametrize("method", [0, 1])
def test_persist_converged(tea, ora, kind, nx, ny, method):
    deck = deck_of(kind, nx, ny, seed=3, dt=0.004)
    kw = dict(method=method, eps=1e-13, max_iters=20000, inner_steps=6)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_p, st_p = gpu_run(tea, deck, persist=1, **kw)
    u_g, st_g = gpu_run(tea, deck, persist=-1, **kw)
    assert s_o[0] == 0 and st_p[0]["ret"] == 0
    assert abs(st_p[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert abs(st_p[0]["iterations"] - st_g[0]["iterations"]) <= 1
    assert field_err(u_p, u_o, kind) <= 1e-10
    assert field_err(u_p, u_g, kind) <= 1e-11
    if method == 1 and st_o[0]["outer"] > 0:
        assert st_p[0]["presteps"] == st_o[0]["presteps"]
        assert st_p[0]["eig_max"] == pytest.approx(st_o[0]["eig_max"], rel=1e-9)


def test_persist_config1_10_steps(tea, ora):
    """BASELINE configs[0] (128^2 CG, 10 timesteps, eps 1e-15) through one launch per step."""
    deck = deck_of("pipe", 128, 128)
    kw = dict(method=0, eps=1e-15, max_iters=10000)
    u_o, st_o, _ = ora.run(deck, steps=10, **kw)
    u_g, st_g = gpu_run(tea, deck, steps=10, persist=1, **kw)
    for a, b in zip(st_g, st_o):
        assert abs(a["iterations"] - b["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("tile_rows", [1, 3, 8])
def test_persist_many_tiles_per_cta(tea, tile_rows):
    """1024^2 with short tiles: more tiles than co-resident CTAs, so each CTA walks
    several tiles per phase; 30 presteps + 3 outer against the graph path."""
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(1024)
    kw = dict(method=1, eps=0.0, max_iters=33, inner_steps=10, tile_rows=tile_rows)
    u_p, st_p = gpu_run(tea, deck, persist=1, **kw)
    u_g, st_g = gpu_run(tea, deck, persist=-1, **kw)
    assert st_p[0]["iterations"] == st_g[0]["iterations"] == 33
    assert st_p[0]["outer"] == st_g[0]["outer"] == 3
    assert rel_err(u_p, u_g) <= 1e-12


# ---------------------------------------------------------------- kform
@pytest.mark.gpu
@pytest.mark.parametrize("kind,nx,ny", [("pipe", 128, 128), ("random", 300, 200),
                                        ("random", 1000, 777), ("random", 257, 65),
                                        ("random", 1, 97), ("random", 95, 1)])
@pytest.mark.parametrize("method,tb,persist", [(0, 0, -1), (1, 5, -1), (1, 1, -1), (1, 3, -1),
                                               (2, 0, -1), (3, 0, -1), (6, 5, -1), (6, 1, -1),
                                               (0, 0, 1), (1, 1, 1), (4, 0, -1), (5, 0, -1)])
@pytest.mark.parametrize("mean_mode", [0, 1])
def test_kform_bitwise(tea, kind, nx, ny, method, tb, persist, mean_mode):
    """Faces formed on the fly from g = 1/rho (kform 1) and read as the stored Kx, Ky
    (kform -1) are the same numbers (the stored faces are computed by the kernels'
    expression), so the whole solve is bitwise identical: fixed iterations and converged,
    for every 2D stencil kernel (SpMV, fused passes, per-step Chebyshev, CG1 / CPPCG1,
    block Jacobi, the persistent solver, Jacobi / Chebyshev iterations)."""
    stationary = method in (4, 5)
    deck = deck_of(kind, nx, ny, seed=5, dt=0.004 if stationary else 0.04)
    for eps, its in ((0.0, 37), (1e-13, 3000 if stationary else 20000)):
        kw = dict(method=method, eps=eps, max_iters=its, inner_steps=6, tb_steps=tb,
                  persist=persist, mean_mode=mean_mode, presteps=10 if stationary else 30)
        u_g, st_g = gpu_run(tea, deck, kform=1, **dict(kw))
        u_k, st_k = gpu_run(tea, deck, kform=-1, **dict(kw))
        assert st_g[0]["iterations"] == st_k[0]["iterations"]
        assert np.array_equal(u_g, u_k)


@pytest.mark.gpu
@pytest.mark.parametrize("blocks,d", [((2, 2), 1), ((2, 2), 7), ((3, 2), 4)])
@pytest.mark.parametrize("method", [0, 1, 6])
def test_kform_bitwise_blocks(tea, ora, blocks, d, method):
    """Decomposed (blocks in one process, halo depth d): g carries real neighbour values in
    the margin and mirrored ghosts at the physical boundary -- bitwise equal to the stored
    faces, and within the parity bar of the oracle."""
    deck = deck_of("random", 301, 203, seed=6, dt=0.04)
    dist = dict(rank=0, nranks=1, px=blocks[0], py=blocks[1], halo_depth=d)
    kw = dict(method=method, eps=1e-13, max_iters=20000, inner_steps=6)
    u_g, st_g = gpu_run(tea, deck, dist=dist, kform=1, **dict(kw))
    u_k, st_k = gpu_run(tea, deck, dist=dist, kform=-1, **dict(kw))
    assert st_g[0]["iterations"] == st_k[0]["iterations"]
    assert np.array_equal(u_g, u_k)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert field_err(u_g, u_o, "random") <= 1e-10


# ---------------------------------------------------------------- single-reduction CPPCG, fused
# TEA_CPPCG1F (oracle ORA_CPPCG1F, reading R23): one block with the fused passes = two kernels
# per outer iteration (the first pass carries the outer update, the last q = A z_s and the
# three dots); blocks / one kernel per step: k_cg1f_pre + chain (+ k_cg1_w) + one reduction.
@pytest.mark.parametrize("kind,nx,ny,s,tb", [("pipe", 128, 128, 10, 0), ("pipe", 256, 200, 10, 5),
                                             ("pipe", 256, 200, 10, 1), ("random", 300, 203, 4, 0),
                                             ("random", 97, 61, 3, 5), ("random", 1000, 777, 10, 0),
                                             ("random", 257, 65, 7, 4), ("random", 1, 97, 6, 5),
                                             ("random", 95, 1, 6, 5)])
def test_cppcg1f_converged(tea, ora, kind, nx, ny, s, tb):
    deck = deck_of(kind, nx, ny, seed=6)
    kw = dict(method=7, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, s_o = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, persist=-1, **kw)
    assert s_o[0] == 0 and st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    if st_g[0]["outer"] > 0 and st_o[0]["outer"] > 0:  # (1-wide decks can converge at the
        assert st_g[0]["presteps"] == st_o[0]["presteps"]  # prestep boundary, +-1)
        assert st_g[0]["matvecs"] == 1 + st_g[0]["presteps"] + s + 1 + st_g[0]["outer"] * (s + 2)
    assert field_err(u_g, u_o, kind) <= 1e-10
    u_c, st_c = gpu_run(tea, deck, tb_steps=tb, persist=-1, **dict(kw, method=1))
    assert abs(st_c[0]["outer"] - st_g[0]["outer"]) <= 2
    assert rel_err(u_g, u_c) <= 1e-10


@pytest.mark.parametrize("s", [2, 3, 4, 5, 7, 10, 11, 13])
def test_cppcg1f_pass_splits(tea, ora, s):
    """Every inner-step count: the one-block fused path splits the chain into an even number
    of passes (the first pass's output never aliases the z_s it reads), pre + post levels."""
    deck = deck_of("pipe", 256, 200)
    kw = dict(method=7, eps=1e-13, max_iters=20000, inner_steps=s)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=5, persist=-1, **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("k", [1, 2, 7])
@pytest.mark.parametrize("tb", [1, 3, 5])
def test_cppcg1f_fixed_iterations(tea, ora, k, tb):
    deck = deck_of("random", 300, 203, seed=8, dt=0.04)
    kw = dict(method=7, eps=0.0, max_iters=30 + k, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, tb_steps=tb, persist=-1, **kw)
    assert st_g[0]["iterations"] == 30 + k and st_g[0]["outer"] == k
    assert iter_err(u_g, u_o, "random") <= 1e-12
    assert float(np.max(np.abs(u_g - u_o))) <= residual_bound(ora, deck, u_g, u_o)
    assert st_g[0]["rnorm"] == pytest.approx(st_o[0]["rnorm"], rel=1e-9)


@pytest.mark.parametrize("px,py,d,tb", [(2, 1, 11, 5), (2, 2, 11, 5), (3, 2, 12, 4), (1, 3, 2, 0),
                                        (4, 2, 4, 0), (2, 2, 1, 0)])
@pytest.mark.parametrize("loop_mode", [0, 2])
def test_cppcg1f_multiblock(tea, ora, px, py, d, tb, loop_mode):
    deck = deck_of("pipe", 200, 170)
    kw = dict(method=7, eps=1e-13, max_iters=20000, inner_steps=10)
    u_o, st_o, _ = ora.run(deck, steps=1, **kw)
    u_g, st_g = gpu_run(tea, deck, dist=dict(px=px, py=py, halo_depth=d, nranks=1), tb_steps=tb,
                        loop_mode=loop_mode, **kw)
    assert st_g[0]["ret"] == 0
    assert abs(st_g[0]["iterations"] - st_o[0]["iterations"]) <= 2
    assert rel_err(u_g, u_o) <= 1e-10


@pytest.mark.parametrize("loop_mode", [1, 2])
def test_cppcg1f_loop_modes_identical(tea, loop_mode):
    deck = deck_of("pipe", 1000, 700)
    kw = dict(method=7, eps=1e-12, max_iters=5000, inner_steps=10)
    ref, st_ref = gpu_run(tea, deck, **kw)
    u, st = gpu_run(tea, deck, loop_mode=loop_mode, check_interval=6, **kw)
    assert st[0]["iterations"] == st_ref[0]["iterations"]
    assert np.array_equal(u, ref)


@pytest.mark.parametrize("nx,ny,px,py,d", [(240, 200, 2, 2, 11), (201, 143, 3, 2, 12), (150, 96, 1, 3, 6)])
@pytest.mark.parametrize("loop_mode", [0, 2])
def test_cppcg1f_blocks_overlap_bitwise(tea, ora, nx, ny, px, py, d, loop_mode):
    """CPPCG1F across blocks with the fused passes: the outer update on ext(d), z_s exchanged
    at depth d + 1 while the one reduction is in flight (on the second stream with overlap on,
    NEXT-2 / P:L817-821): bitwise the same as without the overlap, and the oracle's solution."""
    deck = deck_of("random", nx, ny, seed=nx + ny, dt=0.04)
    s = d - 1
    kw = dict(method=7, eps=0.0, max_iters=30 + 5, inner_steps=s, tb_steps=5, loop_mode=loop_mode,
              dist=dict(px=px, py=py, halo_depth=d, nranks=1))
    u_a, st_a = gpu_run(tea, deck, overlap=1, **kw)
    u_b, st_b = gpu_run(tea, deck, overlap=-1, **kw)
    assert st_a[0]["iterations"] == st_b[0]["iterations"] == 35
    assert np.array_equal(u_a, u_b)
    assert st_a[0]["rnorm"] == st_b[0]["rnorm"]
    u_o, st_o, _ = ora.run(deck, steps=1, method=7, eps=0.0, max_iters=35, inner_steps=s)
    assert iter_err(u_a, u_o, "random") <= 1e-12
    assert st_a[0]["rnorm"] == pytest.approx(st_o[0]["rnorm"], rel=1e-9)


@pytest.mark.parametrize("method", [0, 2, 4, 5])
@pytest.mark.parametrize("px,py", [(2, 2), (3, 1)])
@pytest.mark.parametrize("loop_mode", [0, 2])
def test_reduce_exchange_overlap_bitwise(tea, method, px, py, loop_mode):
    """CG / block-Jacobi / Jacobi / Chebyshev across blocks: the depth-1 halo exchange issued
    on the second stream together with the iteration's reduction (overlap on) gives bitwise
    the same solve as exchange-after-reduction (overlap off)."""
    deck = deck_of("random", 130, 97, seed=11, dt=0.04)
    kw = dict(method=method, eps=1e-12, max_iters=3000, presteps=10, loop_mode=loop_mode,
              dist=dict(px=px, py=py, halo_depth=1, nranks=1))
    u_a, st_a = gpu_run(tea, deck, overlap=1, **kw)
    u_b, st_b = gpu_run(tea, deck, overlap=-1, **kw)
    assert st_a[0]["iterations"] == st_b[0]["iterations"]
    assert np.array_equal(u_a, u_b)
