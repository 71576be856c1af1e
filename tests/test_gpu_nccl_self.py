"""The multi-process NCCL code path on ONE GPU (TEA_NCCL_SELF=1).

NCCL refuses two ranks on one device, so gpurun's single-GPU boxes cannot run the library's
multi-process transport (tests/test_gpu_multirank.py skips there). With TEA_NCCL_SELF=1 a
single process that owns every block of a px x py decomposition sends its halos through a
1-rank NCCL communicator instead of the on-device copy kernel:
  * pack kernel -> grouped ncclSend / ncclRecv to self in the canonical (sending block,
    receiving block, direction) order (several messages per rank pair: the case that order
    exists for) -> unpack kernel;
  * the dot products through ncclAllReduce (after the cross-block combine and mask kernels);
  * the deep exchange on the second stream with the split communicator, overlapped with the
    interior pass and with the allreduce (auto-on, as across processes);
  * chunked CUDA graphs with captured NCCL kernels (the multi-process loop mode) and the
    polled host waits with ncclCommGetAsyncError.
The transport moves the same bytes and every reduction sums the same values, so the fields,
iteration counts and residual norms must equal those of the device-copy run bit for bit, and
the oracle within the north_star bar.
"""
import os

import numpy as np
import pytest

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def tea():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    tea.lib()
    return tea


def run(tea, deck, nccl_self, px, py, d, method, s, eps=1e-12, max_iters=20000, **kw):
    old = os.environ.get("TEA_NCCL_SELF")
    if nccl_self:
        os.environ["TEA_NCCL_SELF"] = "1"
    else:
        os.environ.pop("TEA_NCCL_SELF", None)
    try:
        t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt,
                    dist=dict(rank=0, nranks=1, px=px, py=py, halo_depth=d), **kw)
        r = t.solve(method=method, eps=eps, max_iters=max_iters, inner_steps=s)
        u = t.fetch()
        t.close()
    finally:
        if old is None:
            os.environ.pop("TEA_NCCL_SELF", None)
        else:
            os.environ["TEA_NCCL_SELF"] = old
    return u, r


# (method, d, s): CG (depth-1 exchange + allreduce per iteration, overlapped), CPPCG on the
# fused passes (d = s + 1: the deep (r, w) exchange overlapping the p.w allreduce), CPPCG with
# one kernel per step (d = 2: the matrix-powers schedule), single-reduction CG / CPPCG, the
# fused single-reduction CPPCG (z_s exchange overlapping its one allreduce), block Jacobi
CASES = [("CG", 1, 10), ("CPPCG", 11, 10), ("CPPCG", 2, 10), ("CG1", 1, 10), ("CPPCG1", 11, 10),
         ("CPPCG1F", 11, 10), ("BJCG", 1, 10)]


@pytest.mark.parametrize("px,py", [(2, 2), (3, 2)])
@pytest.mark.parametrize("name,d,s", CASES)
def test_nccl_self_bitwise_and_oracle(tea, ora, px, py, name, d, s):
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(512, 384)
    method = getattr(tea, name)
    u_n, r_n = run(tea, deck, True, px, py, d, method, s)
    u_c, r_c = run(tea, deck, False, px, py, d, method, s)
    assert r_n.status == 0 and r_c.status == 0
    assert r_n.stats["iterations"] == r_c.stats["iterations"]
    assert np.array_equal(u_n, u_c), float(np.max(np.abs(u_n - u_c)))
    u_o, st_o, _ = ora.run(deck, steps=1, method=getattr(ora, name), eps=1e-12,
                           max_iters=20000, inner_steps=s)
    assert abs(r_n.stats["iterations"] - st_o[0]["iterations"]) <= 2
    assert float(np.max(np.abs(u_n - u_o) / np.abs(u_o))) <= 1e-10


@pytest.mark.parametrize("loop_mode", [1, 2])
def test_nccl_self_loop_modes(tea, loop_mode):
    """Chunked graphs (1, the multi-process default) and eager launches (2) over NCCL give the
    same fields, bitwise, as the device-copy transport in the same loop mode."""
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    deck = inputs.crooked_pipe(300, 260)
    for name, d in (("CPPCG", 11), ("CG", 1)):
        u_n, r_n = run(tea, deck, True, 2, 2, d, getattr(tea, name), 10, loop_mode=loop_mode)
        u_c, r_c = run(tea, deck, False, 2, 2, d, getattr(tea, name), 10, loop_mode=loop_mode)
        assert r_n.stats["iterations"] == r_c.stats["iterations"]
        assert np.array_equal(u_n, u_c)
