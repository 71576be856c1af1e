"""Multi-process (gloo, CPU) tests of the multi-GPU host logic.

One process per "GPU" (torch.distributed gloo on 127.0.0.1). Each rank owns the
block the LIBRARY assigns (tea_block_extent) and applies the Chebyshev
preconditioner z = B(A) r following the LIBRARY's matrix-powers schedule
(tea_cheb_schedule: exchange depths, extended bounds, final fix-up), with
halo exchanges (faces + corners) over gloo send/recv and the dot products by
all_reduce. The gathered z must equal the serial oracle's B(A) r, and the
distributed dots the serial ones. A wrong extent, depth, corner or schedule
step breaks the agreement. This is a test-only numpy model of the block
arithmetic (SURVEY §4 "fake backend"); it shares nothing with the CUDA kernels.

Also: the NCCL unique id made by tea_get_nccl_id on rank 0 survives a
process-group broadcast byte for byte (the plumbing tea_init relies on).
"""
import os
import socket
import sys

import numpy as np
import pytest
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

DX = [-1, 1, 0, 0, -1, 1, -1, 1]
DY = [0, 0, -1, 1, -1, -1, 1, 1]


def free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def folded_coeffs(theta, a, b):
    """Per-step coefficients of z_i = cX X + cZ z_{i-2} + cR r - cA A X."""
    out = []
    for i, (ai, bi) in enumerate(zip(a, b)):
        if i == 0:
            out.append(((1 + ai) / theta + bi, 0.0, 0.0, bi / theta))
        elif i == 1:
            out.append((1 + ai, 0.0, bi - ai / theta, bi))
        else:
            out.append((1 + ai, -ai, bi, bi))
    return out


def _worker(rank, world, port, cfg, q):
    try:
        sys.path.insert(0, ROOT)
        os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
        import torch
        import torch.distributed as dist
        dist.init_process_group("gloo", rank=rank, world_size=world)
        import oracle
        import paper_conf_cluster_mcintosh_smithm17_b200 as tea
        from paper_conf_cluster_mcintosh_smithm17_b200 import inputs

        nx, ny, px, py, d, s = cfg
        deck = inputs.crooked_pipe(nx, ny)
        rx, ry = oracle.mesh_r(deck)
        Kx_g, Ky_g = oracle.face_coefficients(nx, ny, rx, ry, deck.density)
        r_g = np.random.default_rng(7).standard_normal((ny, nx))
        mesh = tea.mesh_of(deck)
        x0, x1, y0, y1 = tea.block_extent(mesh, px, py, rank)
        bx, by = x1 - x0, y1 - y0
        bi, bj = rank % px, rank // px
        nbr = []
        for k in range(8):
            ni, nj = bi + DX[k], bj + DY[k]
            nbr.append(nj * px + ni if 0 <= ni < px and 0 <= nj < py else -1)
        H = d + 2

        def field():
            return np.zeros((by + 2 * H, bx + 2 * H))

        def sl(j0, j1, k0, k1):
            return (slice(k0 + H, k1 + H), slice(j0 + H, j1 + H))

        # local face coefficients from the global ones (0 outside the mesh)
        Kx, Ky = field(), field()
        for k in range(-H, by + H):
            gk = y0 + k
            for j in range(-H, bx + H):
                gj = x0 + j
                if 0 <= gk < ny and 0 <= gj <= nx:
                    Kx[k + H, j + H] = Kx_g[gk, gj]
                if 0 <= gk <= ny and 0 <= gj < nx:
                    Ky[k + H, j + H] = Ky_g[gk, gj]
        r = field()
        r[sl(0, bx, 0, by)] = r_g[y0:y1, x0:x1]

        def ext(e):
            return (-e if nbr[0] >= 0 else 0, bx + (e if nbr[1] >= 0 else 0),
                    -e if nbr[2] >= 0 else 0, by + (e if nbr[3] >= 0 else 0))

        def send_box(k, dep):
            j0, j1, k0, k1 = 0, bx, 0, by
            if DX[k] < 0: j1 = dep
            if DX[k] > 0: j0 = bx - dep
            if DY[k] < 0: k1 = dep
            if DY[k] > 0: k0 = by - dep
            return j0, j1, k0, k1

        def recv_box(k, dep):
            j0, j1, k0, k1 = 0, bx, 0, by
            if DX[k] < 0: j0, j1 = -dep, 0
            if DX[k] > 0: j0, j1 = bx, bx + dep
            if DY[k] < 0: k0, k1 = -dep, 0
            if DY[k] > 0: k0, k1 = by, by + dep
            return j0, j1, k0, k1

        def exchange(fields, dep):
            reqs, bufs = [], []
            for k in range(8):
                if nbr[k] < 0 or (k >= 4 and dep < 2):
                    continue
                out = np.concatenate([f[sl(*send_box(k, dep))].ravel() for f in fields])
                t = torch.from_numpy(out.copy())
                reqs.append(dist.isend(t, nbr[k]))
                inn = torch.empty(out.size, dtype=torch.float64)
                reqs.append(dist.irecv(inn, nbr[k]))
                bufs.append((k, inn))
            for q_ in reqs:
                q_.wait()
            for k, inn in bufs:
                v = inn.numpy()
                off = 0
                for f in fields:
                    box = recv_box(k, dep)
                    n = (box[1] - box[0]) * (box[3] - box[2])
                    f[sl(*box)] = v[off:off + n].reshape(box[3] - box[2], box[1] - box[0])
                    off += n

        def apply_A(X, R):
            j0, j1, k0, k1 = R
            c = sl(j0, j1, k0, k1)
            up, dn = sl(j0, j1, k0 + 1, k1 + 1), sl(j0, j1, k0 - 1, k1 - 1)
            rt, lf = sl(j0 + 1, j1 + 1, k0, k1), sl(j0 - 1, j1 - 1, k0, k1)
            kyu = Ky[up]
            kyd = Ky[c]
            kxr = Kx[rt]
            kxl = Kx[c]
            return ((1.0 + (kyu + kyd) + (kxr + kxl)) * X[c] - (kyu * X[up] + kyd * X[dn])
                    - (kxr * X[rt] + kxl * X[lf]))

        # eigen interval + coefficients (oracle's), folded as the kernels do
        lmin, lmax = 1.0, 1.05 * (1 + 4 * (Kx_g.max() + Ky_g.max()))
        theta, a, b = oracle.cheb_coeffs(lmin, lmax, s)
        co = folded_coeffs(theta, a, b)
        z = [field(), field(), field()]  # z_i in z[(i-1) % 3]
        ops = tea.cheb_schedule(s, d)
        step = 0
        for code, arg in ops:
            if code == 1:
                exchange([r], arg)
            elif code == 3:
                exchange([z[(step - 1) % 3], z[(step - 2) % 3] if step >= 2 else z[(step - 1) % 3]],
                         arg)
            elif code == 4:
                exchange([z[(s - 1) % 3]], arg)
            else:
                step += 1
                R = ext(arg)
                cx, cz, cr, ca = co[step - 1]
                X = r if step == 1 else z[(step - 2) % 3]
                AX = apply_A(X, R)
                c = sl(*R)
                zn = cx * X[c] - ca * AX
                if step >= 2:
                    zn = zn + cr * r[c]
                if step >= 3:
                    zn = zn + cz * z[(step - 3) % 3][c]
                z[(step - 1) % 3][c] = zn
        zs = z[(s - 1) % 3]
        # the final z must be valid on the 1-cell ring toward every neighbour
        ring = ext(1)
        own = zs[sl(0, bx, 0, by)]
        rz = torch.tensor([float(np.sum(r[sl(0, bx, 0, by)] * own))], dtype=torch.float64)
        dist.all_reduce(rz)
        q.put((rank, (x0, x1, y0, y1), own.copy(), zs[sl(*ring)].copy(), ring, float(rz.item()),
               (bx, by)))
        dist.barrier()
        dist.destroy_process_group()
    except Exception as e:  # surface worker failures in the parent
        import traceback
        q.put(("error", rank, traceback.format_exc()))
        raise


def run_cluster(cfg, world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, cfg, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=300) for _ in range(world)]
    for p in procs:
        p.join(timeout=120)
    for r in res:
        if r[0] == "error":
            raise AssertionError(f"rank {r[1]} failed:\n{r[2]}")
    return res


@pytest.mark.parametrize("world,px,py,d,s", [
    (2, 2, 1, 1, 1), (2, 2, 1, 1, 4), (2, 1, 2, 2, 10), (2, 2, 1, 3, 5), (2, 1, 2, 5, 10),
    (4, 2, 2, 2, 10), (4, 2, 2, 4, 7), (4, 4, 1, 1, 3),
])
def test_distributed_chebyshev_matches_oracle(ora, world, px, py, d, s):
    from paper_conf_cluster_mcintosh_smithm17_b200 import inputs
    nx, ny = 41, 36
    res = run_cluster((nx, ny, px, py, d, s), world)
    deck = inputs.crooked_pipe(nx, ny)
    rx, ry = ora.mesh_r(deck)
    Kx, Ky = ora.face_coefficients(nx, ny, rx, ry, deck.density)
    r_g = np.random.default_rng(7).standard_normal((ny, nx))
    lmin, lmax = 1.0, 1.05 * (1 + 4 * (Kx.max() + Ky.max()))
    theta, a, b = ora.cheb_coeffs(lmin, lmax, s)
    z_ref = ora.cheb_apply(Kx, Ky, s, theta, a, b, r_g)
    z = np.full((ny, nx), np.nan)
    for rank, (x0, x1, y0, y1), own, ringvals, ring, rz, (bx, by) in res:
        z[y0:y1, x0:x1] = own
        # ring values (toward neighbours) equal the neighbours' owned values
        j0, j1, k0, k1 = ring
        gx0, gy0 = x0 + j0, y0 + k0
        ref_ring = z_ref[gy0:gy0 + (k1 - k0), gx0:gx0 + (j1 - j0)]
        np.testing.assert_allclose(ringvals, ref_ring, rtol=1e-11,
                                   atol=1e-12 * np.abs(z_ref).max())
    assert not np.isnan(z).any()
    np.testing.assert_allclose(z, z_ref, rtol=1e-11, atol=1e-12 * np.abs(z_ref).max())
    rz_ref = float(np.sum(r_g * z_ref))
    for r_ in res:
        assert r_[5] == pytest.approx(rz_ref, rel=1e-12)


def _id_worker(rank, world, port, q):
    sys.path.insert(0, ROOT)
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    import torch
    import torch.distributed as dist
    dist.init_process_group("gloo", rank=rank, world_size=world)
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    buf = torch.zeros(128, dtype=torch.uint8)
    if rank == 0:
        buf.copy_(torch.frombuffer(bytearray(tea.get_nccl_id()), dtype=torch.uint8))
    dist.broadcast(buf, 0)
    q.put((rank, bytes(buf.numpy().tobytes())))
    dist.barrier()
    dist.destroy_process_group()


def test_nccl_id_broadcast_over_process_group():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = free_port()
    procs = [ctx.Process(target=_id_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    got = dict(q.get(timeout=120) for _ in range(2))
    for p in procs:
        p.join(timeout=60)
    assert len(got[0]) == 128 and got[0] == got[1] and any(got[0])


# ---------------------------------------------------------------- halo message order
# NCCL (like gloo) matches the point-to-point calls between two ranks in posting order. With
# several blocks per rank a rank pair carries several messages, some of equal size; the
# library posts them in one canonical order (tea_halo_order). Each rank replays the LIBRARY's
# order over gloo isend/irecv (one tag, FIFO per pair) with payloads that name the message;
# every receive must get exactly the message it was posted for.
HALO_CASES = [  # (nx, ny, px, py, nranks, depth, corners)
    (64, 48, 2, 2, 2, 3, True),    # a face and an equal-sized corner cross between 2 ranks
    (64, 48, 4, 2, 2, 4, True),
    (96, 64, 2, 4, 4, 11, True),
    (90, 60, 3, 2, 2, 2, True),    # 3 blocks per rank, ragged extents
    (80, 80, 4, 4, 2, 1, False),   # depth 1, faces only
    (80, 80, 4, 4, 4, 5, True),
]


def _code(src, dst, d):
    return float((src * 64 + dst) * 8 + d)


def _halo_worker(rank, world, port, cases, q):
    import torch
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    sys.path.insert(0, ROOT)
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    dist.init_process_group("gloo", rank=rank, world_size=world)
    res = []
    for (nx, ny, px, py, nranks, depth, corners) in cases:
        if nranks != world:
            continue
        msgs = tea.halo_order(tea.make_mesh(nx, ny), px, py, nranks, rank, depth, corners)
        reqs, recv = [], []
        for op, peer, src, dst, d, n in msgs:
            if op == 0:
                t = torch.full((n,), _code(src, dst, d), dtype=torch.float64)
                reqs.append(dist.isend(t, int(peer), tag=7))
        for op, peer, src, dst, d, n in msgs:
            if op == 1:
                t = torch.zeros(n, dtype=torch.float64)
                reqs.append(dist.irecv(t, int(peer), tag=7))
                recv.append((src, dst, d, t))
        for r in reqs:
            r.wait()
        ok = all(bool(torch.all(t == _code(s, dd, d))) for s, dd, d, t in recv)
        res.append(((nx, ny, px, py, nranks, depth, corners), ok, len(msgs)))
    dist.barrier()
    dist.destroy_process_group()
    q.put((rank, res))


@pytest.mark.parametrize("world", [2, 4])
def test_halo_message_order_over_gloo(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = free_port()
    procs = [ctx.Process(target=_halo_worker, args=(r, world, port, HALO_CASES, q))
             for r in range(world)]
    for p in procs:
        p.start()
    got = dict(q.get(timeout=180) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
    for r in range(world):
        assert got[r], "no case ran"
        for case, ok, n in got[r]:
            assert n > 0 and ok, (r, case)


def test_halo_message_order_pairs_agree():
    """Host-only: for every rank pair, A's sends to B equal B's receives from A, in order and
    length -- and the per-rank block x direction order of round 1 would cross-match the 2 x 2
    grid on 2 ranks (a corner received into a face's buffer of the same size)."""
    sys.path.insert(0, ROOT)
    import paper_conf_cluster_mcintosh_smithm17_b200 as tea
    for (nx, ny, px, py, nranks, depth, corners) in HALO_CASES:
        m = tea.make_mesh(nx, ny)
        per = {r: tea.halo_order(m, px, py, nranks, r, depth, corners) for r in range(nranks)}
        for a in range(nranks):
            for b in range(nranks):
                if a == b:
                    continue
                s = [(src, dst, d, n) for op, p, src, dst, d, n in per[a] if op == 0 and p == b]
                r = [(src, dst, d, n) for op, p, src, dst, d, n in per[b] if op == 1 and p == a]
                assert s == r, (nx, ny, px, py, nranks, a, b)
    # round 1: each rank posted (block, direction) pairs in its own loop order
    m = tea.make_mesh(64, 48)
    DXY = list(zip(DX, DY))

    def natural(rank, op):
        out = []
        for i in range(2):
            g = rank * 2 + i
            bi, bj = g % 2, g // 2
            for d, (dx, dy) in enumerate(DXY):
                ni, nj = bi + dx, bj + dy
                if 0 <= ni < 2 and 0 <= nj < 2 and (nj * 2 + ni) // 2 != rank:
                    nb = nj * 2 + ni
                    out.append((g, nb, d) if op == 0 else (nb, g, [1, 0, 3, 2, 7, 6, 5, 4][d]))
        return out
    assert natural(0, 0) != natural(1, 1)  # the crossing the canonical order removes
    canon = [(s, t, d) for op, p, s, t, d, n in tea.halo_order(m, 2, 2, 2, 0, 3, True) if op == 0]
    assert canon == [(s, t, d) for op, p, s, t, d, n in tea.halo_order(m, 2, 2, 2, 1, 3, True)
                     if op == 1]
