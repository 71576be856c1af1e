"""CPU-side checks of the C-ABI library (no GPU, no compute calls):

* libtea_b200.so builds for sm_100a, loads, and exports every function that
  include/tea.h declares; the SASS is sm_100a;
* the host-only helpers: block decomposition (remainder to the low
  blocks) and the matrix-powers Chebyshev schedule: every step's
  operands are valid where it reads them, exchanges are at most depth d, and the
  final z covers the 1-cell ring the next SpMV needs;
* workspace sizing and argument validation (TEA_ERR_ARG paths).
"""
import os
import re
import subprocess

import pytest

import paper_conf_cluster_mcintosh_smithm17_b200 as tea
from paper_conf_cluster_mcintosh_smithm17_b200 import _build

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def L():
    _build.build()
    return tea.lib()


def header_functions():
    src = open(os.path.join(ROOT, "include", "tea.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(tea_[a-z_0-9]+)\s*\(", src)))


def test_exports_every_declared_symbol(L):
    names = header_functions()
    assert len(names) >= 14
    out = subprocess.check_output(["nm", "-D", "--defined-only", _build.LIB]).decode()
    exported = set(re.findall(r" T (tea_\w+)", out))
    missing = [n for n in names if n not in exported]
    assert not missing, missing
    for n in names:
        getattr(L, n)
    assert sorted(tea.SYMBOLS) == names


def test_sm100a_sass():
    out = subprocess.check_output(["cuobjdump", "--list-elf", _build.LIB]).decode()
    assert "sm_100a" in out


def test_version(L):
    import re
    assert "sm_100a" in tea.version()
    hdr = open(os.path.join(ROOT, "include", "tea.h")).read()
    v = int(re.search(r"#define TEA_ABI_VERSION (\d+)", hdr).group(1))
    assert L.tea_abi_version() == v == tea.ABI_VERSION
    # the binding's tea_opts mirrors the header's field list (same order)
    body = hdr[hdr.index("typedef struct {", hdr.index("Solver options")):hdr.index("} tea_opts;")]
    fields = re.findall(r"^\s+(?:int|double)\s+(\w+);", body, re.M)
    assert fields == [f for f, _ in tea.Opts._fields_]


@pytest.mark.parametrize("nx,ny,px,py", [(4096, 4096, 2, 4), (1000, 777, 3, 2), (17, 5, 4, 1),
                                         (128, 128, 1, 8)])
def test_block_extent_partition(L, nx, ny, px, py):
    m = tea.make_mesh(nx, ny)
    cover = [[0] * nx for _ in range(1)]
    xs, ys = set(), set()
    for b in range(px * py):
        x0, x1, y0, y1 = tea.block_extent(m, px, py, b)
        xs.add((x0, x1))
        ys.add((y0, y1))
        assert x1 - x0 in (nx // px, nx // px + 1)
        assert y1 - y0 in (ny // py, ny // py + 1)
        # remainder on low-index blocks
        bi, bj = b % px, b // px
        if bi < nx % px:
            assert x1 - x0 == nx // px + 1
    assert sorted(xs)[0][0] == 0 and sorted(xs)[-1][1] == nx
    assert sum(b - a for a, b in xs) == nx
    assert sum(b - a for a, b in ys) == ny
    del cover


def simulate_schedule(ops, s, d):
    """Track the valid depth of each operand; return the final z extension."""
    valid = {"r": 0}
    zs = {}
    step = 0
    max_ex = 0
    for code, arg in ops:
        if code == 1:
            assert 1 <= arg <= d
            valid["r"] = arg
            max_ex = max(max_ex, arg)
        elif code == 3:
            assert 1 <= arg <= d and step >= 1
            zs[step] = arg
            if step >= 2:
                zs[step - 1] = arg
            max_ex = max(max_ex, arg)
        elif code == 4:
            assert step == s and arg == 1
            zs[step] = 1
        else:
            step += 1
            e = arg
            assert e >= 0
            if step == 1:  # z1 = r/theta: stencil on r
                assert valid["r"] >= e + 1
            else:
                assert zs[step - 1] >= e + 1  # stencil operand
                if step == 2:
                    assert valid["r"] >= e  # z_0 = r/theta pointwise
                else:
                    assert zs[step - 2] >= e
                assert valid["r"] >= e
            zs[step] = e
    assert step == s
    return zs[s], max_ex


@pytest.mark.parametrize("s", [1, 2, 3, 5, 10, 16])
@pytest.mark.parametrize("d", [1, 2, 3, 5, 10, 16])
def test_cheb_schedule_valid(L, s, d):
    ops = tea.cheb_schedule(s, d)
    final, max_ex = simulate_schedule(ops, s, d)
    assert final >= 1  # the next SpMV reads z on the 1-cell ring
    assert max_ex <= d
    n_ex = sum(1 for c, _ in ops if c != 2)
    # matrix powers: about one exchange per d matvecs
    assert n_ex <= -(-s // max(d - 1, 1)) + 2
    if d == 1:
        assert n_ex == s + 1


def test_cheb_schedule_bad_args(L):
    with pytest.raises(tea.TeaError):
        tea.cheb_schedule(0, 2)
    with pytest.raises(tea.TeaError):
        tea.cheb_schedule(10, 17)


def test_workspace_bytes_and_validation(L):
    m = tea.make_mesh(4096, 4096)
    one = tea.workspace_bytes(m)
    # 14 pitched fp64 fields dominate (u0, u, Kx, Ky, g, r x2, p x2, w, z x4; block Jacobi
    # keeps its Thomas coefficients in two z fields it does not use): ~14 x 4096^2 x 8 B
    assert 14 * 4096 * 4096 * 8 <= one <= 1.05 * 14 * 4110 * 4200 * 8 + (8 << 20)
    d8 = tea.Dist(0, 8, 2, 4, 10, None)
    part = tea.workspace_bytes(m, d8)
    assert part < one / 6
    with pytest.raises(tea.TeaError):
        tea.workspace_bytes(m, tea.Dist(0, 3, 2, 2, 1, None))  # 4 blocks over 3 ranks
    with pytest.raises(tea.TeaError):
        tea.workspace_bytes(tea.make_mesh(8, 8), tea.Dist(0, 1, 8, 1, 2, None))  # too thin
    with pytest.raises(tea.TeaError):
        tea.workspace_bytes(m, tea.Dist(0, 1, 1, 1, 17, None))


def test_no_cpu_fallback():
    """The product package never imports the oracle and has no CPU solve path."""
    pkg = os.path.dirname(tea.__file__)
    for root, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".h", ".cpp")):
                txt = open(os.path.join(root, f)).read()
                assert "import oracle" not in txt and "from oracle" not in txt
                assert "tea_oracle" not in txt


def test_fused_pass_tile_plan_matches_measured_optima():
    """The fused passes' tile-height model (tea_tb_plan, host-only) picks the
    heights the B200 sweeps measured best (profiles/r02_tbrows_model.txt, r02_tbrows_4096.jsonl):
    4096^2 187 rows (one wave at 3 CTAs/SM: 2219 it/s vs 2021-2150 for 160-293), 1024^2 18
    (14.5 / 17.8 us per pass vs 17.5 / 20.1 at 25), the 2 x 4 blocks' first pass on ext(6)
    (2060 x 1036) ~36 (2 CTAs per SM; 24-row tiles at 3 per SM measured slower), 2048^2 a
    3-per-SM wave near 50 (60 and 71 measured slower)."""
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    assert tea.tb_plan(5, 4096, 4096) == 187
    assert tea.tb_plan(5, 1024, 1024) == 18
    assert 34 <= tea.tb_plan(5, 2060, 1036) <= 38
    assert 44 <= tea.tb_plan(5, 2048, 2048) <= 52
    for lv, w, h in [(1, 64, 3), (6, 16384, 16384), (3, 100, 1), (5, 333, 4097)]:
        ty = tea.tb_plan(lv, w, h)
        assert 1 <= ty <= min(h, 512)
    with pytest.raises(tea.TeaError):
        tea.tb_plan(0, 10, 10)
