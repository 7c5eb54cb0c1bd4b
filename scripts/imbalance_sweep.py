#!/usr/bin/env python
"""Load-imbalance sweep of SURVEY §8(e) on one GPU: the per-rank tracking work of a P-rank run.

    python scripts/imbalance_sweep.py [--config split] [--ranks 2 4 8] [--out gpurun_out/imb.json]

For each P, every rank r's shard is tracked on this GPU in turn (the library is the same one
a P-process run uses; only the shards differ) and its tracking time is recorded:
  * "ids":     rank r owns global ids [rN/P, (r+1)N/P) of the config's source (births iid);
  * "spatial": rank r injects its N/P particles from the source strip x in [r/P, (r+1)/P)
               (a spatial decomposition of the source: ranks owning the dense half of split
               finish early).
Reported per P and partition: per-rank track ms, max/mean, and the scaling efficiency the
slowest rank allows, (sum of rank times) / (P * max rank time).  The NCCL tally allreduce
(~0.3 ms at 4000^2) is not included.
"""
from __future__ import annotations

import argparse
import json
import statistics
import sys
from pathlib import Path

ROOT = Path(__file__).resolve().parents[1]
sys.path.insert(0, str(ROOT))

from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="split")
    ap.add_argument("--ranks", type=int, nargs="+", default=[2, 4, 8])
    ap.add_argument("--reps", type=int, default=2)
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    cfg = wl.CONFIGS[a.config]
    N = cfg.n_particles
    t = binding.Tracker()
    t.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, wl.density(cfg))
    t.load_cross_sections(*wl.tables(cfg))
    sx, sy, sw, sh = cfg.source
    out = {"config": cfg.name, "particles": N, "results": []}
    for P in a.ranks:
        for part in ("ids", "spatial"):
            ms, ev = [], []
            for r in range(P):
                lo, hi = r * N // P, (r + 1) * N // P
                src = cfg.source if part == "ids" else (sx + sw * r / P, sy, sw / P, sh)
                best = None
                for _ in range(a.reps):
                    t.inject_particles(N, lo, hi - lo, src, cfg.e0, cfg.seed)
                    s = t.run_timestep(cfg.dt)
                    best = s if best is None or s["track_ms"] < best["track_ms"] else best
                ms.append(best["track_ms"])
                ev.append(best["events"])
            m, mx = statistics.mean(ms), max(ms)
            row = {"P": P, "partition": part, "track_ms": ms, "events": ev,
                   "max_over_mean": mx / m, "efficiency": sum(ms) / (P * mx),
                   "events_per_s_at_P": sum(ev) / (mx / 1e3)}
            out["results"].append(row)
            print(f"P={P} {part:8s} max/mean={mx / m:.3f} eff={row['efficiency']:.3f} "
                  f"ms=[{', '.join(f'{x:.1f}' for x in ms)}]", flush=True)
    t.close()
    if a.out:
        Path(a.out).parent.mkdir(parents=True, exist_ok=True)
        Path(a.out).write_text(json.dumps(out, indent=1) + "\n")


if __name__ == "__main__":
    main()
