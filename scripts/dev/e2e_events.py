"""bench.py's e2e loop with a CUDA event after every C-ABI call (no extra synchronisation):
where the e2e step's time goes when the calls run back to back."""
import json
import sys

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
names = ["init_mesh", "load_cross_sections", "inject_particles", "run_timestep", "read_tally"]
calls = [lambda: tr.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, pin_d),
         lambda: tr.load_cross_sections(*pin_t),
         lambda: tr.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed),
         lambda: tr.run_timestep(cfg.dt),
         lambda: tr.read_tally(out)]
acc = {k: [] for k in names}
tot = []
for rep in range(8):
    ev = [torch.cuda.Event(enable_timing=True) for _ in range(len(calls) + 1)]
    ev[0].record(stream)
    for k, f in enumerate(calls):
        f()
        ev[k + 1].record(stream)
    torch.cuda.synchronize()
    if rep >= 2:
        for k, n in enumerate(names):
            acc[n].append(ev[k].elapsed_time(ev[k + 1]))
        tot.append(ev[0].elapsed_time(ev[-1]))
res = {k: float(np.median(v)) for k, v in acc.items()}
res["step"] = float(np.median(tot))
print(json.dumps({"config": cfg.name, "median_ms_between_events": res}))
