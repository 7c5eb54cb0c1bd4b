"""Near-tie flip rate of a library variant against the oracle (run with NT_LIB_VARIANT=...):
the fraction of particles whose integer results (facet / collision / census counts, RNG
counter, status, cell) differ, and the max relative difference of E, w and the tally."""
import json
import sys

import numpy as np

sys.path.insert(0, ".")
import oracle  # noqa: E402
from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl  # noqa: E402

out = {}
for name in ["tiny_csp", "small_csp", "small_scatter", "tiny_mid", "tiny_split", "small_mosaic"]:
    cfg = wl.CONFIGS[name]
    ot, op, _ = oracle.run(cfg)
    for mode in ("history", "event"):
        t = binding.setup(cfg, mode=mode)
        t.run_timestep(cfg.dt)
        g = t.read_particles()
        gt = t.read_tally()
        t.close()
        bad = np.zeros(cfg.n_particles, dtype=bool)
        for f in ["nfac", "ncol", "ncen", "ctr", "status", "cx", "cy"]:
            bad |= g[f] != getattr(op, f)
        ok = ~bad
        rel = lambda a, b: float(np.max(np.abs(a - b) / np.maximum(np.abs(b), 1e-300))) if a.size else 0.0  # noqa: E731
        scale = max(np.max(np.abs(ot)), 1e-300)
        out[f"{name}/{mode}"] = {
            "particles": int(cfg.n_particles), "flipped": int(bad.sum()),
            "flip_rate": float(bad.mean()),
            "e_max_rel_unflipped": rel(g["e"][ok], op.e[ok]), "w_max_rel_unflipped": rel(g["w"][ok], op.w[ok]),
            "tally_max_rel": float(np.max(np.where(np.abs(ot) > 1e-12 * scale, np.abs(gt - ot) / np.maximum(np.abs(ot), 1e-300), 0))),
        }
        print(name, mode, out[f"{name}/{mode}"], flush=True)
print(json.dumps(out))
