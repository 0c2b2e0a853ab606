"""world_size-2 tests of the multi-GPU host logic on CPU (gloo).

* The per-rank schedule that sg_run_rank issues (kernel launches, NCCL sends and
  receives of boundary-stream fragments) is replayed with real gloo point-to-point
  messages: every message must match (same edge, fragment and size on both
  sides, in the same order -- NCCL P2P matches by order), nothing may deadlock,
  and every partition of a rank must be launched for every fragment.
* The replica helpers bench.py uses under torchrun (iteration sharding, max over
  ranks).
"""
import os
import socket

import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    return port


def _worker(rank, world, port, name, n, frag, q, replicas=1, extra=None):
    import sys
    sys.path.insert(0, ROOT)
    try:
        dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
        from workloads import apps
        from paper_conf_cgo_nguyenl16_b200 import sg
        from paper_conf_cgo_nguyenl16_b200.dist import max_over_ranks, replica_shard
        prog = {"filterbank8": lambda: apps.filterbank(8), "fmradio4": lambda: apps.fmradio(5),
                "beamformer": lambda: apps.beamformer(channels=3, beams=2, frame=64, taps=8, mf_taps=16)}[name]()
        with sg.plan(prog, world, iters_per_fragment=frag, replicas=replicas, plan_only=1, **(extra or {})) as p:
            info = p.info()
            R = info["replicas"]
            Gs = world // R
            grp = rank // Gs
            ops = p.rank_schedule(rank, n)
            mine = [q_ for q_, g in enumerate(info["partition_gpu"]) if g == rank % Gs]
            for o in ops:                                            # peers stay inside the replica group
                assert o["peer"] // Gs == grp
            launched = {}
            sent = recv = 0
            for o in ops:
                if o["op"] == sg.SG_OP_LAUNCH:
                    assert o["part"] in mine
                    launched.setdefault(o["part"], []).append((o["k_begin"], o["k_end"]))
                    continue
                tag = o["edge"] * 100003 + o["fragment"]
                if o["op"] == sg.SG_OP_SEND:
                    t = torch.full((o["items"] + 2,), tag, dtype=torch.int64)
                    t[-1] = o["items"]
                    dist.send(t, dst=o["peer"])
                    sent += 1
                else:
                    t = torch.empty(o["items"] + 2, dtype=torch.int64)
                    dist.recv(t, src=o["peer"])
                    assert int(t[0]) == tag, (int(t[0]), tag)       # same edge and fragment
                    assert int(t[-1]) == o["items"]                  # same size on both sides
                    recv += 1
            nfrag = (n + frag - 1) // frag
            want = [(f * frag, min(n, (f + 1) * frag)) for f in range(grp, nfrag, R)]   # this group's fragments
            for part in mine:                                        # every fragment of every partition
                assert sorted(launched.get(part, [])) == want
            k0, k1 = replica_shard(1000, rank, world)
            tot = torch.tensor([k1 - k0])
            dist.all_reduce(tot)
            assert int(tot) == 1000
            assert max_over_ranks(float(rank + 1)) == float(world)
            q.put((rank, "ok", sent, recv, len(info["partition_gpu"])))
        dist.barrier()
        dist.destroy_process_group()
    except Exception as e:  # report to the parent
        import traceback
        q.put((rank, "fail", traceback.format_exc()))


CHAIN = dict(chain_groups=-2, partitioner="chain")   # chain_groups = world (filled in below)


@pytest.mark.parametrize("name,n,frag,world,replicas,extra", [
    ("filterbank8", 5000, 700, 2, 1, None), ("fmradio4", 3000, 512, 2, 1, None), ("beamformer", 40, 7, 2, 1, None),
    # hybrid replica x pipeline plans: two groups
    ("filterbank8", 5000, 300, 2, 2, None), ("fmradio4", 3000, 256, 4, 2, None),
    # chain fission: one group per rank, forward + accumulate streams hop rank to rank
    ("filterbank8", 5000, 700, 2, 1, CHAIN), ("fmradio4", 3000, 256, 4, 1, CHAIN)])
def test_rank_schedules_match_over_gloo(name, n, frag, world, replicas, extra):
    if extra is CHAIN:
        extra = dict(CHAIN, chain_groups=world)
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, name, n, frag, q, replicas, extra))
             for r in range(world)]
    for p in procs:
        p.start()
    results = [q.get(timeout=240) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
    for r in results:
        assert r[1] == "ok", r
    sent = sum(r[2] for r in results)
    recv = sum(r[3] for r in results)
    assert sent == recv


def test_replica_shard_covers_range():
    from paper_conf_cgo_nguyenl16_b200.dist import replica_shard
    for total in (0, 1, 7, 1000, 1 << 20):
        for world in (1, 2, 3, 8):
            spans = [replica_shard(total, r, world) for r in range(world)]
            assert spans[0][0] == 0 and spans[-1][1] == total
            assert all(spans[i][1] == spans[i + 1][0] for i in range(world - 1))
