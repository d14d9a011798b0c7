import os, torch, torch.distributed as dist
from torch.multiprocessing.reductions import reduce_tensor
dist.init_process_group("gloo")
r = dist.get_rank()
torch.cuda.set_device(0)
if r == 0:
    full = torch.zeros(8, dtype=torch.int32, device="cuda")
    obj = [reduce_tensor(full)]
else:
    obj = [None]
dist.broadcast_object_list(obj, src=0)
if r != 0:
    fn, args = obj[0]
    view = fn(*args)
    view[4:] = 7
    torch.cuda.synchronize()
dist.barrier()
if r == 0:
    full[:4] = 1
    torch.cuda.synchronize()
    print("rank0 sees", full.tolist(), flush=True)
dist.barrier()
