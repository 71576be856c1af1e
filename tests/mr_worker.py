"""One rank of a multi-process (NCCL) solve, for tests/test_gpu_multirank.py (launched with
torch.distributed.run, one process per GPU). Writes this rank's owned cells of u (zeros
elsewhere) and the solve statistics to OUT/u_<rank>.npy and OUT/stats_<rank>.json.

python -m torch.distributed.run --nproc-per-node N --master-addr 127.0.0.1 --master-port P \
    tests/mr_worker.py OUT NX NY METHOD HALO_DEPTH EPS MAX_ITERS INNER
"""
import json
import os
import sys

import numpy as np
import torch
import torch.distributed as dist

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import paper_conf_cluster_mcintosh_smithm17_b200 as tea  # noqa: E402
from paper_conf_cluster_mcintosh_smithm17_b200 import inputs  # noqa: E402


def factor(n):
    best = (1, n)
    for px in range(1, n + 1):
        if n % px == 0 and abs(px - n // px) < abs(best[0] - best[1]):
            best = (px, n // px)
    return best


def main():
    out, nx, ny, method, d, eps, its, s = sys.argv[1:9]
    nx, ny, method, d, its, s, eps = int(nx), int(ny), int(method), int(d), int(its), int(s), float(eps)
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    local = int(os.environ.get("LOCAL_RANK", rank))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    dist.init_process_group("nccl", device_id=dev)
    nid = torch.zeros(128, dtype=torch.uint8, device=dev)
    if rank == 0:
        nid.copy_(torch.frombuffer(bytearray(tea.get_nccl_id()), dtype=torch.uint8))
    dist.broadcast(nid, 0)
    px, py = factor(world)
    deck = inputs.crooked_pipe(nx, ny)
    t = tea.Tea(tea.mesh_of(deck), deck.density, deck.energy, deck.dt,
                dist=dict(rank=rank, nranks=world, px=px, py=py, halo_depth=d,
                          nccl_id=bytes(nid.cpu().numpy().tobytes())))
    r = t.solve(method=method, eps=eps, max_iters=its, inner_steps=s)
    u = np.zeros((ny, nx))
    t.fetch(u)
    t.close()
    np.save(os.path.join(out, f"u_{rank}.npy"), u)
    json.dump(dict(r.stats, ret=r.status, px=px, py=py), open(os.path.join(out, f"stats_{rank}.json"), "w"))
    dist.barrier()
    dist.destroy_process_group()


if __name__ == "__main__":
    main()
