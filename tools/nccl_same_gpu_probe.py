"""Can two NCCL ranks share one GPU on this box?  (Probe for exercising the band exchange's NCCL
transport with one GPU; not the product.)  Run: torchrun --nproc-per-node 2 ... this file."""
import os

import torch
import torch.distributed as dist

rank = int(os.environ["RANK"])
torch.cuda.set_device(0)
try:
    dist.init_process_group("nccl", device_id=torch.device("cuda", 0))
    t = torch.full((4,), float(rank), device="cuda")
    if rank == 0:
        dist.send(t, 1)
    else:
        dist.recv(t, 0)
    torch.cuda.synchronize()
    print("rank", rank, "ok", t.tolist(), flush=True)
    dist.destroy_process_group()
except Exception as e:  # noqa: BLE001
    print("rank", rank, "failed:", type(e).__name__, str(e).splitlines()[0][:300], flush=True)
