"""Full-size parity, element by element (VERDICT r01 "next 1"): BASELINE.json configs[2]/[3]
(4096^2) and configs[4] (16384^2) against the CPU oracle run live in the test, every cell.

The oracle (serial C, 1 host core) runs a fixed number of iterations (eps = 0): 50 CG
iterations and 30 CG presteps + 3 CPPCG outer iterations at 4096^2 (~6-9 s each), 30 presteps
+ 1 outer at 16384^2 (~2 min, ~30 GB of host memory). The GPU runs the same iterations in the
launch configuration bench.py times (one block: the wave-fitted SpMV tiles and the tall fused
Chebyshev passes only this size reaches) and in the 8-GPU decomposition (2 x 4 blocks in one
process, halo depth s + 1 = 11 for CPPCG, 1 for CG: the extended-bounds fused passes, the deep
exchange with corners, the cross-block reductions). Bar: the north_star's max pointwise
relative field error 1e-10 (the pipe has u >= 0.01 everywhere), identical iteration counts,
residual norm and eigen-estimate to 1e-9. The measured errors are printed (pytest -s).
"""
import numpy as np
import pytest

pytestmark = pytest.mark.gpu

TOL = 1e-10


@pytest.fixture(scope="module")
def tea():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    tea.lib()
    return tea


def gpu_run(tea, deck, dist=None, **kw):
    import torch
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt, dist=dist)
    r = t.solve(**kw)
    u = t.fetch()
    t.close()
    del t
    torch.cuda.empty_cache()
    return u, r


def pointwise(a, b):
    return float(np.max(np.abs(a - b) / np.abs(b)))


_cache = {}


def oracle_case(ora, n, method, its):
    key = (n, method, its)
    if key not in _cache:
        from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
        deck = inputs.crooked_pipe(n)
        u, st, status = ora.run(deck, steps=1, method=method, eps=0.0, max_iters=its,
                                inner_steps=10)
        _cache[key] = (deck, u, st[0], status[0])
    return _cache[key]


@pytest.mark.parametrize("method,its", [(0, 50), (1, 33), (7, 33)])
@pytest.mark.parametrize("blocks", [None, (2, 4)])
def test_4096_every_cell(tea, ora, method, its, blocks):
    deck, u_o, st_o, s_o = oracle_case(ora, 4096, method, its)
    dist = None
    if blocks:
        dist = dict(rank=0, nranks=1, px=blocks[0], py=blocks[1],
                    halo_depth=11 if method in (1, 7) else 1)
    u_g, r = gpu_run(tea, deck, dist, method=method, eps=0.0, max_iters=its, inner_steps=10)
    err = pointwise(u_g, u_o)
    print(f"\n4096^2 method={method} its={its} blocks={blocks}: max pointwise rel err "
          f"{err:.3e} over {u_o.size} cells; rnorm gpu {r.stats['rnorm']:.6e} oracle "
          f"{st_o['rnorm']:.6e}")
    assert s_o == 1 and r.status == 1  # TEA_NOT_CONVERGED: the fixed count was run
    assert r.stats["iterations"] == st_o["iterations"] == its
    assert r.stats["rnorm"] == pytest.approx(st_o["rnorm"], rel=1e-9)
    if method in (1, 7):
        assert r.stats["presteps"] == st_o["presteps"] == 30
        assert r.stats["outer"] == st_o["outer"] == its - 30
        assert r.stats["eig_min"] == pytest.approx(st_o["eig_min"], rel=1e-9)
        assert r.stats["eig_max"] == pytest.approx(st_o["eig_max"], rel=1e-9)
    assert err <= TOL


def test_16384_every_cell(tea, ora):
    """configs[4]: 16384^2 CPPCG (s = 10), 30 presteps + 1 outer iteration: one block and
    the 2 x 4 decomposition (depth 11) against the oracle, all 268M cells."""
    import torch
    free, _ = torch.cuda.mem_get_info()
    if free < 40 << 30:
        pytest.skip(f"needs ~35 GB of free HBM, {free >> 30} GB free")
    deck, u_o, st_o, s_o = oracle_case(ora, 16384, 1, 31)
    u_1, r1 = gpu_run(tea, deck, None, method=1, eps=0.0, max_iters=31, inner_steps=10)
    e1 = pointwise(u_1, u_o)
    u_8, r8 = gpu_run(tea, deck, dict(rank=0, nranks=1, px=2, py=4, halo_depth=11), method=1,
                      eps=0.0, max_iters=31, inner_steps=10)
    e8 = pointwise(u_8, u_o)
    e18 = pointwise(u_8, u_1)
    print(f"\n16384^2 CPPCG 30+1: 1 block vs oracle {e1:.3e}, 2x4 vs oracle {e8:.3e}, "
          f"2x4 vs 1 block {e18:.3e} over {u_o.size} cells")
    for r in (r1, r8):
        assert r.status == 1
        assert r.stats["iterations"] == st_o["iterations"] == 31
        assert r.stats["outer"] == st_o["outer"] == 1
        assert r.stats["rnorm"] == pytest.approx(st_o["rnorm"], rel=1e-9)
        assert r.stats["eig_max"] == pytest.approx(st_o["eig_max"], rel=1e-9)
    assert e1 <= TOL and e8 <= TOL and e18 <= TOL


_conv = {}


@pytest.mark.parametrize("method", [0, 1, 7])
def test_1024_converged_every_cell(tea, ora, method):
    """configs[1]: 1024^2, CG vs CPPCG (and the single-reduction CPPCG), converged to
    eps = 1e-12 in the bench's configuration, against the oracle run live: every cell within
    the north_star's 1e-10, iteration counts within +-2; CG and CPPCG within the R22 bound."""
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(1024)
    u_o, st_o, s_o = ora.run(deck, steps=1, method=method, eps=1e-12, max_iters=20000,
                             inner_steps=10)
    u_g, r = gpu_run(tea, deck, None, method=method, eps=1e-12, max_iters=20000, inner_steps=10)
    err = pointwise(u_g, u_o)
    print(f"\n1024^2 method={method}: iterations gpu {r.stats['iterations']} oracle "
          f"{st_o[0]['iterations']}, max pointwise rel err {err:.3e}")
    assert s_o[0] == 0 and r.status == 0
    assert abs(r.stats["iterations"] - st_o[0]["iterations"]) <= 2
    assert err <= TOL
    _conv[method] = u_g
    if 0 in _conv and method != 0:
        # CG and CPPCG stop at the same relative residual, not at the same error: their fields
        # differ by ~kappa eps (1e-9 here), bounded per cell by the two true residual norms
        # (lambda_min(A) = 1, reading R22)
        rx, ry = ora.mesh_r(deck)
        Kx, Ky = ora.face_coefficients(1024, 1024, rx, ry, deck.density)
        u0 = deck.density * deck.energy
        bound = sum(float(np.linalg.norm(u0 - ora.apply_A(Kx, Ky, u))) for u in (u_g, _conv[0]))
        assert float(np.max(np.abs(u_g - _conv[0]))) <= bound
