"""Full paper-scale parity: every particle and every tally cell of the BASELINE.json
workloads (csp, stream, scatter, split at 4000^2, 1e6-1e7 particles), CUDA path vs the
oracle run over all ids on the host cores (tests/full_oracle.py).

North star bar (BASELINE.json): per-particle facet / collision / census counts, RNG counter
and status exact; E, w to 1e-9; the production (fp64 atomic) tally to 1e-6 per cell, the
deterministic tally to 1e-9.  The paper validates a run through its tally
(§VI-F); its test problems are P:197-218 §IV-B.  Set NT_PARITY_REPORT=<dir> to
write one JSON report per case.
"""
import json
import os

import numpy as np
import pytest

from paper_conf_cluster_martineaum17_b200 import workloads as wl
from tests.parity import compare_particles, compare_stats, compare_tally

pytestmark = pytest.mark.gpu

CASES = [
    ("csp", "history", {}), ("csp", "event", {}),
    ("csp", "history", {"density_format": 1}), ("csp", "event", {"density_format": 1}),
    ("csp", "history", {"layout": 1}), ("csp", "event", {"layout": 1}),
    ("csp", "history", {"deterministic": True}), ("csp", "event", {"deterministic": True}),
    ("csp", "history", {"fused_consumers": 1}),
    ("stream", "history", {}), ("stream", "event", {}), ("stream", "history", {"deterministic": True}),
    ("scatter", "history", {}), ("scatter", "event", {}), ("scatter", "history", {"deterministic": True}),
    ("split", "history", {}), ("split", "event", {}), ("split", "history", {"fused_consumers": 1}),
    ("split", "history", {"deterministic": True}),
]

_CACHE = {}


@pytest.fixture(scope="module")
def nt():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cluster_martineaum17_b200 import binding, build
    build.build()
    return binding


def _oracle_full(cfgname):
    if cfgname not in _CACHE:
        from tests.full_oracle import run_full
        _CACHE.clear()                       # one workload's results at a time (split: ~1 GB)
        _CACHE[cfgname] = run_full(wl.CONFIGS[cfgname])
    return _CACHE[cfgname]


@pytest.mark.parametrize("cfgname,mode,opts", CASES,
                         ids=[f"{c}-{m}-{'-'.join(f'{k}{v}' for k, v in o.items()) or 'default'}"
                              for c, m, o in CASES])
def test_fullscale_every_particle_and_cell(nt, cfgname, mode, opts):
    cfg = wl.CONFIGS[cfgname]
    ot, op, os_, info = _oracle_full(cfgname)
    t = nt.setup(cfg, mode=mode, **opts)
    gs = t.run_timestep(cfg.dt)
    gt = t.read_tally()
    gp = t.read_particles()
    t.close()
    assert gs["status"] == 0
    det = bool(opts.get("deterministic"))
    rep_p = compare_particles(gp, op)                       # every particle: counts exact
    rep_t = compare_tally(gt, ot, rtol=1e-9 if det else 1e-6, floor=1e-9 if det else 1e-12)
    compare_stats(gs, os_, rtol=1e-9)
    rep = {"config": cfgname, "mode": mode, "opts": opts, "particles": int(cfg.n_particles),
           "events": int(gs["events"]), "oracle_procs": info["procs"], "oracle_wall_s": info["wall_s"],
           "tally": rep_t, "particle_fields": rep_p, "gpu_track_ms": gs["track_ms"]}
    print(json.dumps(rep))
    out = os.environ.get("NT_PARITY_REPORT")
    if out:
        os.makedirs(out, exist_ok=True)
        name = f"{cfgname}_{mode}_{'_'.join(f'{k}{v}' for k, v in opts.items()) or 'default'}.json"
        with open(os.path.join(out, name), "w") as f:
            json.dump(rep, f, indent=1)
