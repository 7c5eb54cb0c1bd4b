"""Parity helpers: compare the CUDA path's outputs with the oracle's, element by element.

Tolerances (BASELINE.json north_star):
* integers (facet / collision / census counts, RNG counter, status, cell indices): exact;
* E, w: relative 1e-9 (expected bit-exact: no libm in their chain);
* x, y, directions, mean free paths, per-particle deposits, per-cell tally:
  relative 1e-9 in the deterministic build, with an absolute floor of 1e-9 x max for
  cells / values whose only contributions are sub-ulp grazes; the production (fp64
  atomic) tally: relative 1e-6.
"""
from __future__ import annotations

import numpy as np

INT_FIELDS = ["nfac", "ncol", "ncen", "ctr", "status", "cx", "cy"]
EXACT_FP = ["e", "w"]
FP_FIELDS = ["x", "y", "ox", "oy", "mfp", "dep"]


def _as_dict(p):
    return p if isinstance(p, dict) else p.as_dict()


def compare_particles(gpu, orc, rtol=1e-9, idx=None):
    """Return a report dict; raise AssertionError on any violation."""
    g, o = _as_dict(gpu), _as_dict(orc)
    rep = {}
    for f in INT_FIELDS:
        a, b = np.asarray(g[f]), np.asarray(o[f])
        bad = np.nonzero(a != b)[0]
        assert bad.size == 0, f"{f}: {bad.size} mismatches, first at {bad[:5]}: gpu {a[bad[:5]]} oracle {b[bad[:5]]}"
    for f in EXACT_FP:
        a, b = np.asarray(g[f]), np.asarray(o[f])
        rel = np.abs(a - b) / np.maximum(np.abs(b), 1e-300)
        assert np.all(rel <= rtol), f"{f}: max rel {rel.max()}"
        rep[f + "_bitexact_frac"] = float(np.mean(a == b))
    for f in FP_FIELDS:
        a, b = np.asarray(g[f]), np.asarray(o[f])
        scale = max(np.max(np.abs(b)), 1e-300)
        err = np.abs(a - b)
        ok = err <= rtol * np.abs(b) + rtol * scale
        bad = np.nonzero(~ok)[0]
        assert bad.size == 0, f"{f}: {bad.size} beyond tol, first {bad[:5]}: {a[bad[:5]]} vs {b[bad[:5]]}"
        rep[f + "_bitexact_frac"] = float(np.mean(a == b))
    return rep


def compare_tally(gpu, orc, rtol=1e-9, floor=1e-9):
    g, o = np.asarray(gpu).ravel(), np.asarray(orc).ravel()
    scale = max(np.max(np.abs(o)), 1e-300)
    err = np.abs(g - o)
    rel_ok = err <= rtol * np.abs(o)
    floor_ok = err <= floor * scale
    bad = np.nonzero(~(rel_ok | floor_ok))[0]
    assert bad.size == 0, (f"tally: {bad.size} cells beyond tol, first {bad[:5]}: "
                           f"{g[bad[:5]]} vs {o[bad[:5]]}")
    return {"cells": int(g.size), "floor_cells": int(np.sum(~rel_ok & floor_ok)),
            "bitexact_frac": float(np.mean(g == o)),
            "max_rel": float(np.max(np.where(np.abs(o) > 0, err / np.maximum(np.abs(o), 1e-300), 0)))}


def compare_stats(gs: dict, os_: dict, rtol=1e-9):
    for k in ["n_alive_start", "n_facets", "n_collisions", "n_census", "n_killed", "n_xs_range",
              "n_nonfinite", "n_event_cap", "n_escaped", "n_absorbed"]:
        assert gs[k] == os_[k], f"stat {k}: gpu {gs[k]} oracle {os_[k]}"
    for k in ["tally_total", "census_energy", "census_weight", "killed_energy", "killed_weight",
              "absorbed_weight", "escaped_energy", "escaped_weight", "absorbed_energy",
              "roulette_gain"]:
        a, b = gs[k], os_[k]
        assert abs(a - b) <= rtol * max(abs(b), 1e-300) + 1e-300, f"stat {k}: gpu {a} oracle {b}"
