"""The oracle over a whole paper-size workload, one process per host core (test helper).

Particle histories are independent given the mesh and tables, and the
RNG is keyed by the global id, so a workload's per-particle results and its
tally are the oracle's results over disjoint id ranges, and the tally is their sum (tallies
are additive over particles).  Each process runs the unmodified single-threaded oracle on
one contiguous id range and writes its particles and its partial tally into shared files;
the parent adds the partial tallies in rank order.

Used by tests/test_gpu_fullscale.py only (the oracle is test infrastructure).
"""
from __future__ import annotations

import multiprocessing as mp
import os
import tempfile
import time

import numpy as np

import oracle
from paper_conf_cluster_martineaum17_b200 import workloads as wl

_FIELDS = [(n, t) for n, t in oracle.Particles.FIELDS]


def _shm_dir() -> str:
    return "/dev/shm" if os.path.isdir("/dev/shm") and os.access("/dev/shm", os.W_OK) else tempfile.gettempdir()


def _worker(cfg, lo, n, tdir, r, steps):
    prob = oracle.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    p = oracle.inject(prob, lo, n)
    tally = np.memmap(os.path.join(tdir, f"tally_{r}.f64"), dtype=np.float64, mode="w+",
                      shape=(cfg.nx * cfg.ny,))
    st = None
    for _ in range(steps):
        tally[:] = 0.0
        st = oracle.step(prob, p, lo, tally)
    tally.flush()
    for name, dt in _FIELDS:
        a = np.memmap(os.path.join(tdir, f"{name}_{r}.bin"), dtype=dt, mode="w+", shape=(max(n, 1),))
        a[:n] = getattr(p, name)
        a.flush()
    np.save(os.path.join(tdir, f"stats_{r}.npy"), np.array([st[k] for k in sorted(st)], dtype=np.float64))


def run_full(cfg, procs: int | None = None, steps: int = 1):
    """(tally [ny][nx], particles dict, stats dict, info) of the oracle over all ids of cfg."""
    procs = procs or (len(os.sched_getaffinity(0)) if hasattr(os, "sched_getaffinity") else os.cpu_count())
    oracle.build()
    n_total = cfg.n_particles
    procs = max(1, min(procs, n_total))
    spans = [wl.shard(n_total, r, procs) for r in range(procs)]
    ctx = mp.get_context("fork")
    t0 = time.perf_counter()
    with tempfile.TemporaryDirectory(dir=_shm_dir()) as tdir:
        ps = [ctx.Process(target=_worker, args=(cfg, lo, n, tdir, r, steps)) for r, (lo, n) in enumerate(spans)]
        for q in ps:
            q.start()
        for q in ps:
            q.join()
            assert q.exitcode == 0, f"oracle worker failed ({q.exitcode})"
        wall = time.perf_counter() - t0
        tally = np.zeros(cfg.nx * cfg.ny)
        for r in range(procs):
            tally += np.memmap(os.path.join(tdir, f"tally_{r}.f64"), dtype=np.float64, mode="r",
                               shape=(cfg.nx * cfg.ny,))
        parts = {}
        for name, dt in _FIELDS:
            parts[name] = np.concatenate([
                np.array(np.memmap(os.path.join(tdir, f"{name}_{r}.bin"), dtype=dt, mode="r",
                                   shape=(max(n, 1),))[:n]) for r, (lo, n) in enumerate(spans)])
        keys = sorted(oracle.stats_dict(oracle._Stats()).keys())
        tot = np.sum([np.load(os.path.join(tdir, f"stats_{r}.npy")) for r in range(procs)], axis=0)
        stats = {k: (int(v) if k.startswith("n_") else float(v)) for k, v in zip(keys, tot)}
    return tally.reshape(cfg.ny, cfg.nx), parts, stats, {"procs": procs, "wall_s": wall}
