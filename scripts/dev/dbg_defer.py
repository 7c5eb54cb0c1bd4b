import numpy as np, sys
sys.path.insert(0, '.')
from paper_conf_cluster_martineaum17_b200 import binding, workloads as wl
cfg = wl.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "tiny_csp"]
for det in (False, True):
    for db in (1, 8, 33):
        t = binding.setup(cfg, deterministic=det, defer_below=db)
        s = t.run_timestep(cfg.dt)
        g = t.read_particles()
        t.close()
        print(f"det={det} defer={db} status counts={np.bincount(g['status'], minlength=3)} "
              f"facets={s['n_facets']} coll={s['n_collisions']} census={s['n_census']} killed={s['n_killed']} launches={s['n_launches']}")
