"""Can NCCL run two ranks on one GPU here? (expected: no -- duplicate GPU)"""
import os, sys
import torch, torch.distributed as dist
dist.init_process_group("nccl")
torch.cuda.set_device(0)
x = torch.ones(4, device="cuda:0") * (dist.get_rank() + 1)
try:
    dist.all_reduce(x)
    torch.cuda.synchronize()
    print("rank", dist.get_rank(), "allreduce ok", x.tolist(), flush=True)
except Exception as e:
    print("rank", dist.get_rank(), "failed:", repr(e)[:300], flush=True)
dist.destroy_process_group()
