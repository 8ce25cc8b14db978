# can two NCCL ranks share one GPU? (used to decide whether real multi-rank NCCL paths can be
# exercised on a single-GPU box)
import os, sys, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch, torch.distributed as dist
dist.init_process_group("gloo")
r, n = dist.get_rank(), dist.get_world_size()
torch.cuda.set_device(0)
from paper_1011_0024_b200 import qudax
obj = [qudax.nccl_unique_id() if r == 0 else None]
dist.broadcast_object_list(obj, src=0)
try:
    ctx = qudax.Context((8, 4, 6, 16), nranks=n, rank=r, device=0, comm=qudax.COMM_NCCL, nccl_id=obj[0])
    print(r, "NCCL init ok", flush=True)
    ctx.close()
except Exception as e:
    print(r, "NCCL init failed:", e, flush=True)
dist.barrier()
os._exit(0)
