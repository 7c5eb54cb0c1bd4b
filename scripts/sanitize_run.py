#!/usr/bin/env python
"""One small run of every tracking path through the C ABI, for compute-sanitizer.

    compute-sanitizer --tool memcheck|racecheck|synccheck|initcheck \
        python scripts/sanitize_run.py [--config tiny_csp]

Runs history and event mode, deterministic and production tallies, the x-slab path and the
physics variants on tiny problems, and checks each against the oracle (so a sanitizer run
also shows the results are unchanged under instrumentation).
"""
import argparse
import sys
from pathlib import Path

ROOT = Path(__file__).resolve().parents[1]
sys.path.insert(0, str(ROOT))

import numpy as np  # noqa: E402

import oracle  # noqa: E402
from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl  # noqa: E402
from tests.parity import compare_particles, compare_tally  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--configs", default="tiny_csp,tiny_mid,tiny_analog_mid")
    a = ap.parse_args()
    n = 0
    for name in a.configs.split(","):
        cfg = wl.CONFIGS[name].with_(n_particles=min(400, wl.CONFIGS[name].n_particles))
        ot, op, _ = oracle.run(cfg)
        for mode in ("history", "event"):
            for det in (False, True):
                t = binding.setup(cfg, mode=mode, deterministic=det)
                t.run_timestep(cfg.dt)
                compare_particles(t.read_particles(), op)
                compare_tally(t.read_tally(), ot, rtol=1e-9 if det else 1e-6, floor=1e-9 if det else 1e-12)
                t.close()
                n += 1
                print(f"{name} {mode} det={det}: ok", flush=True)
        # fused phases (one launch, cross-CTA hand-over of parked particles)
        for fused in (1, 2):
            t = binding.setup(cfg, mode="history", fused_consumers=fused, defer_below=33)
            t.run_timestep(cfg.dt)
            compare_particles(t.read_particles(), op)
            compare_tally(t.read_tally(), ot, rtol=1e-6, floor=1e-12)
            t.close()
            n += 1
            print(f"{name} history fused={fused}: ok", flush=True)
        # resume ring (cp.async into shared memory) and the bucket-index-only XS search
        for opts in ({"resume_prefetch": 1, "defer_below": 33}, {"xs_search": 3}, {"xs_search": 1}):
            t = binding.setup(cfg, mode="history", **opts)
            t.run_timestep(cfg.dt)
            compare_particles(t.read_particles(), op)
            compare_tally(t.read_tally(), ot, rtol=1e-6, floor=1e-12)
            t.close()
            n += 1
            print(f"{name} history {opts}: ok", flush=True)
    # x-slabs (caller-driven exchange, 2 contexts)
    cfg = wl.CONFIGS["tiny_csp"].with_(n_particles=300)
    ts = [binding.setup(cfg, first_id=lo, n_local=k, rank=r, nranks=2, decomposition=1)
          for r, (lo, k) in enumerate(wl.shard(cfg.n_particles, r, 2) for r in range(2))]
    for t in ts:
        t.slab_begin(cfg.dt)
    while True:
        outs = [t.slab_round() for t in ts]
        if sum(outs) == 0:
            break
        ex = [t.slab_export(k) for t, k in zip(ts, outs)]
        if ex[0][2]:
            ts[1].slab_import(ex[0][0][ex[0][1]:])
        if ex[1][1]:
            ts[0].slab_import(ex[1][0][:ex[1][1]])
    for t in ts:
        t.slab_end()
    tally = sum(t.read_tally(reduced=False) for t in ts)
    ot, _, _ = oracle.run(cfg)
    compare_tally(tally, ot, rtol=1e-6, floor=1e-12)
    for t in ts:
        t.close()
    print(f"slabs: ok; {n + 1} runs clean", flush=True)


if __name__ == "__main__":
    main()
