"""One process per GPU (torch.distributed plumbing for sg_run_rank).

    import torch.distributed as dist
    from paper_conf_cgo_nguyenl16_b200 import dist as sgdist
    plan = sgdist.pipeline_plan(program)          # same plan on every rank, n_gpus = world size
    plan.run_rank(x_or_None, n, y_or_None)        # boundary streams: NCCL send/recv over NVLink

torch.distributed only carries the NCCL unique id (a 128-byte broadcast) and the
barriers / max-over-ranks timing of the benchmark; every boundary-stream byte
moves through the native library's ncclSend/ncclRecv.  Also: the replica helpers
used by bench.py (`replica_shard`, `max_over_ranks`).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

from . import sg


def pipeline_plan(program, **plan_kw):
    world, rank = dist.get_world_size(), dist.get_rank()
    plan = sg.plan(program, world, **plan_kw)
    uid = [sg.comm_unique_id() if rank == 0 else None]
    dist.broadcast_object_list(uid, src=0)
    device = torch.cuda.current_device()
    plan.comm_init(world, rank, uid[0], device)
    return plan


def replica_shard(n_total: int, rank: int, world: int):
    """Contiguous iteration range [k0, k1) of rank `rank` when n_total iterations are split."""
    per = n_total // world
    extra = n_total % world
    k0 = rank * per + min(rank, extra)
    return k0, k0 + per + (1 if rank < extra else 0)


def max_over_ranks(value: float, device=None) -> float:
    if not dist.is_initialized() or dist.get_world_size() == 1:
        return value
    t = torch.tensor([value], dtype=torch.float64, device=device)
    dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return float(t.item())
