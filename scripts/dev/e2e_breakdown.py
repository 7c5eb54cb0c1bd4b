"""Where the e2e step's time goes: each C-ABI call of bench.py's e2e loop timed
alone with a device synchronize on both sides, pinned host buffers, csp workload."""
import json
import sys
import time

import numpy as np
import torch

sys.path.insert(0, ".")
from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl  # noqa: E402

cfg = wl.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "csp"]
stream = torch.cuda.current_stream()
tr = binding.Tracker(device=0, stream=stream.cuda_stream, mode="history", A=cfg.A,
                     molar_mass=cfg.molar_mass, e_min=cfg.e_min, w_min=cfg.w_min)
pin_d = torch.from_numpy(wl.density(cfg)).pin_memory()
pin_t = [torch.from_numpy(np.ascontiguousarray(x)).pin_memory() for x in wl.tables(cfg)]
out = torch.empty((cfg.ny, cfg.nx), dtype=torch.float64).pin_memory()
calls = {
    "init_mesh": lambda: tr.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, pin_d),
    "load_cross_sections": lambda: tr.load_cross_sections(*pin_t),
    "inject_particles": lambda: tr.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source,
                                                    cfg.e0, cfg.seed),
    "run_timestep": lambda: tr.run_timestep(cfg.dt),
    "read_tally": lambda: tr.read_tally(out),
}
ms = {k: [] for k in calls}
for rep in range(6):
    for k, f in calls.items():
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        f()
        torch.cuda.synchronize()
        if rep > 0:
            ms[k].append((time.perf_counter() - t0) * 1e3)
res = {k: float(np.median(v)) for k, v in ms.items()}
res["sum"] = sum(res.values())
res["h2d_MB"] = (pin_d.numel() + sum(x.numel() for x in pin_t)) * 8 / 1e6
res["d2h_MB"] = out.numel() * 8 / 1e6
print(json.dumps({"config": cfg.name, "median_ms": res}))
