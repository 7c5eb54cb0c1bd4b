import sys, numpy as np
sys.path.insert(0, '.')
from paper_conf_cluster_martineaum17_b200 import binding as nt, workloads as wl
cfg = wl.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "tiny_csp"]
P = 2
ranks = []
for r in range(P):
    lo, n = wl.shard(cfg.n_particles, r, P)
    ranks.append(nt.setup(cfg, first_id=lo, n_local=n, rank=r, nranks=P, decomposition=1))
for t in ranks: t.slab_begin(cfg.dt)
rnd = 0
while True:
    outs = [t.slab_round() for t in ranks]
    parts = [t.read_particles() for t in ranks]
    print("round", rnd, "outs", outs, "status counts", [np.bincount(p["status"], minlength=5).tolist() for p in parts], "n_local", [len(p["status"]) for p in parts])
    rnd += 1
    if sum(outs) == 0 or rnd > 50: break
    exp = [t.slab_export(n) for t, n in zip(ranks, outs)]
    print("   exports", [(nl, nr) for _, nl, nr in exp])
    for r, (recs, nl, nr) in enumerate(exp):
        if nl: ranks[r - 1].slab_import(recs[:nl])
        if nr: ranks[r + 1].slab_import(recs[nl:])
st = [t.slab_end() for t in ranks]
parts = [t.read_particles() for t in ranks]
for r, p in enumerate(parts):
    print("rank", r, "status", np.bincount(p["status"], minlength=5).tolist(), "gid range", p["gid"].min(), p["gid"].max())
seen = np.zeros(cfg.n_particles, int)
for p in parts:
    k = p["status"] <= 1
    seen[p["gid"][k]] += 1
miss = np.nonzero(seen != 1)[0]
print("missing/dup", len(miss), miss[:10])
for g in miss[:5]:
    for r, p in enumerate(parts):
        w = np.nonzero(p["gid"] == g)[0]
        print("  gid", g, "rank", r, "slots", w, "status", p["status"][w], "cx", p["cx"][w])
