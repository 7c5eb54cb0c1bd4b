"""Multi-process host logic of the N > 1 path, on CPU with the gloo backend (world_size 2).

What runs on each rank of a real 8-GPU job:
* rank r owns global ids [floor(rN/P), floor((r+1)N/P)) (workloads.shard); RNG keys use the
  global id, so per-particle results do not depend on P;
* rank 0's 128-byte NCCL unique id is broadcast with torch.distributed;
* the per-rank tallies are summed by an allreduce once per timestep and the step statistics
  are summed the same way; the timestep time is the max over ranks.
Here the per-rank tracker is the oracle (no GPU) and the collective is gloo's allreduce; the
result must equal the single-process run (tally within summation-order rounding).
"""
import os

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_conf_cluster_martineaum17_b200 import workloads as wl

WORLD = 2


def _worker(rank, world, port, cfgname, out_dir):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    import oracle
    cfg = wl.CONFIGS[cfgname]
    # unique-id broadcast, as bench.py does for the NCCL communicator
    obj = [os.urandom(128) if rank == 0 else None]
    dist.broadcast_object_list(obj, src=0)
    assert isinstance(obj[0], bytes) and len(obj[0]) == 128
    first, n = wl.shard(cfg.n_particles, rank, world)
    tally, parts, (st,) = oracle.run(cfg, first_id=first, n_local=n)
    t = torch.from_numpy(tally.ravel().copy())
    dist.all_reduce(t, op=dist.ReduceOp.SUM)
    keys = ["n_alive_start", "n_facets", "n_collisions", "n_census", "n_killed", "tally_total",
            "census_energy", "census_weight", "killed_energy", "killed_weight", "absorbed_weight"]
    s = torch.tensor([float(st[k]) for k in keys], dtype=torch.float64)
    dist.all_reduce(s, op=dist.ReduceOp.SUM)
    ms = torch.tensor([float(rank + 1)], dtype=torch.float64)
    dist.all_reduce(ms, op=dist.ReduceOp.MAX)
    np.save(os.path.join(out_dir, f"tally_{rank}.npy"), t.numpy())
    np.save(os.path.join(out_dir, f"stats_{rank}.npy"), s.numpy())
    np.savez(os.path.join(out_dir, f"parts_{rank}.npz"), **parts.as_dict())
    np.save(os.path.join(out_dir, f"ms_{rank}.npy"), ms.numpy())
    dist.barrier()
    dist.destroy_process_group()


@pytest.mark.parametrize("cfgname", ["tiny_csp", "tiny_split"])
def test_two_rank_shards_equal_single_run(orc, tmp_path, cfgname):
    import socket
    with socket.socket() as sk:
        sk.bind(("127.0.0.1", 0))
        port = sk.getsockname()[1]
    mp.start_processes(_worker, args=(WORLD, port, cfgname, str(tmp_path)), nprocs=WORLD,
                       join=True, start_method="spawn")
    cfg = wl.CONFIGS[cfgname]
    t_all, p_all, (s_all,) = orc.run(cfg)
    for r in range(WORLD):
        t = np.load(tmp_path / f"tally_{r}.npy")
        assert np.allclose(t, t_all.ravel(), rtol=1e-12, atol=0)          # allreduced tally
        s = np.load(tmp_path / f"stats_{r}.npy")
        assert s[0] == s_all["n_alive_start"] and s[1] == s_all["n_facets"]
        assert s[2] == s_all["n_collisions"] and s[3] == s_all["n_census"]
        assert abs(s[5] - s_all["tally_total"]) <= 1e-12 * s_all["tally_total"]
        assert np.load(tmp_path / f"ms_{r}.npy")[0] == WORLD                 # max over ranks
    parts = [np.load(tmp_path / f"parts_{r}.npz") for r in range(WORLD)]
    for name, _ in orc.Particles.FIELDS:
        cat = np.concatenate([p[name] for p in parts])
        assert np.array_equal(cat, getattr(p_all, name)), name


def test_shard_partition_covers_ids():
    for n in [0, 1, 7, 1000, 1 << 23, 10_000_000]:
        for world in [1, 2, 3, 4, 8]:
            spans = [wl.shard(n, r, world) for r in range(world)]
            assert spans[0][0] == 0
            for (a, na), (b, _) in zip(spans, spans[1:]):
                assert a + na == b
            assert spans[-1][0] + spans[-1][1] == n
            assert max(s[1] for s in spans) - min(s[1] for s in spans) <= 1
