"""CPU oracle for the neutral particle-history tracker -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package.  The product path
(``paper_conf_cluster_martineaum17_b200``) never imports it, and it never imports
the product path: the only shared module is the input generator
``paper_conf_cluster_martineaum17_b200.workloads``, which holds none of the method's
arithmetic.

The arithmetic lives in ``neutral_oracle.c`` (plain C, fp64, built with
``-O2 -ffp-contract=off -fno-fast-math``); this file is ctypes marshalling only.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess
from pathlib import Path

import numpy as np

_HERE = Path(__file__).resolve().parent
LIB_PATH = _HERE / "liboracle.so"
_SRC = _HERE / "neutral_oracle.c"
_HDR = _HERE / "neutral_oracle.h"

CFLAGS = ["-O2", "-std=c11", "-ffp-contract=off", "-fno-fast-math", "-fPIC", "-shared"]


def build(force: bool = False) -> Path:
    """Compile liboracle.so with gcc (no FMA contraction)."""
    if (not force and LIB_PATH.exists()
            and LIB_PATH.stat().st_mtime >= max(_SRC.stat().st_mtime, _HDR.stat().st_mtime)):
        return LIB_PATH
    tmp = LIB_PATH.with_suffix(f".so.tmp{os.getpid()}")
    subprocess.check_call(["gcc", *CFLAGS, "-o", str(tmp), str(_SRC), "-lm"])
    os.replace(tmp, LIB_PATH)
    return LIB_PATH


class _Problem(C.Structure):
    _fields_ = [("nx", C.c_int32), ("ny", C.c_int32), ("width", C.c_double),
                ("height", C.c_double), ("density", C.c_void_p),
                ("scatter_keys", C.c_void_p), ("scatter_vals", C.c_void_p),
                ("n_scatter", C.c_int64), ("capture_keys", C.c_void_p),
                ("capture_vals", C.c_void_p), ("n_capture", C.c_int64),
                ("A", C.c_double), ("molar_mass", C.c_double), ("e_min", C.c_double),
                ("w_min", C.c_double), ("max_events", C.c_int64), ("boundary", C.c_int32),
                ("analog", C.c_int32), ("roulette", C.c_int32), ("pad", C.c_int32),
                ("roulette_weight", C.c_double)]


_PFIELDS = [("x", np.float64), ("y", np.float64), ("ox", np.float64), ("oy", np.float64),
            ("e", np.float64), ("w", np.float64), ("mfp", np.float64), ("cx", np.int32),
            ("cy", np.int32), ("ctr", np.uint32), ("status", np.uint8), ("nfac", np.uint32),
            ("ncol", np.uint32), ("ncen", np.uint32), ("dep", np.float64),
            ("tfl", np.float64)]   # tfl: the oracle's flight-time ledger (no GPU counterpart)


class _Particles(C.Structure):
    _fields_ = [(n, C.c_void_p) for n, _ in _PFIELDS]


class _Stats(C.Structure):
    _fields_ = [("n_alive_start", C.c_uint64), ("n_facets", C.c_uint64),
                ("n_collisions", C.c_uint64), ("n_census", C.c_uint64),
                ("n_killed", C.c_uint64), ("tally_total", C.c_double),
                ("census_energy", C.c_double), ("census_weight", C.c_double),
                ("killed_energy", C.c_double), ("killed_weight", C.c_double),
                ("absorbed_weight", C.c_double), ("n_xs_range", C.c_uint64),
                ("n_nonfinite", C.c_uint64), ("n_event_cap", C.c_uint64),
                ("n_escaped", C.c_uint64), ("n_absorbed", C.c_uint64),
                ("escaped_energy", C.c_double), ("escaped_weight", C.c_double),
                ("absorbed_energy", C.c_double), ("roulette_gain", C.c_double)]


_lib_handle = None


def lib():
    global _lib_handle
    if _lib_handle is None:
        L = C.CDLL(str(build()))
        u64, d, i32, i64, vp = C.c_uint64, C.c_double, C.c_int32, C.c_int64, C.c_void_p
        L.or_threefry2x64_20.argtypes = [u64, u64, u64, u64, C.POINTER(u64)]
        L.or_threefry2x64_20.restype = None
        L.or_u01.argtypes = [u64]
        L.or_u01.restype = d
        L.or_edge.argtypes = [i32, d, i32]
        L.or_edge.restype = d
        L.or_cell_of.argtypes = [d, d, i32]
        L.or_cell_of.restype = i32
        L.or_xs_index.argtypes = [vp, i64, d]
        L.or_xs_index.restype = i64
        L.or_xs_lookup.argtypes = [vp, vp, i64, d]
        L.or_xs_lookup.restype = d
        L.or_inject.argtypes = [C.POINTER(_Problem), C.POINTER(_Particles), i64, i64,
                                d, d, d, d, d, u64]
        L.or_inject.restype = None
        L.or_step.argtypes = [C.POINTER(_Problem), C.POINTER(_Particles), i64, i64, u64, d,
                              vp, C.POINTER(_Stats)]
        L.or_step.restype = None
        _lib_handle = L
    return _lib_handle


def _ptr(a: np.ndarray) -> int:
    assert a.flags["C_CONTIGUOUS"]
    return a.ctypes.data


# ---- scalar primitives (for pins) ------------------------------------------------------
def threefry2x64_20(c0: int, c1: int, k0: int, k1: int) -> tuple[int, int]:
    out = (C.c_uint64 * 2)()
    lib().or_threefry2x64_20(c0, c1, k0, k1, out)
    return int(out[0]), int(out[1])


def u01(x: int) -> float:
    return lib().or_u01(x)


def edge(i: int, extent: float, n: int) -> float:
    return lib().or_edge(i, extent, n)


def cell_of(q: float, extent: float, n: int) -> int:
    return lib().or_cell_of(q, extent, n)


def xs_index(keys: np.ndarray, e: float) -> int:
    keys = np.ascontiguousarray(keys, dtype=np.float64)
    return lib().or_xs_index(_ptr(keys), len(keys), e)


def xs_lookup(keys: np.ndarray, vals: np.ndarray, e: float) -> float:
    keys = np.ascontiguousarray(keys, dtype=np.float64)
    vals = np.ascontiguousarray(vals, dtype=np.float64)
    return lib().or_xs_lookup(_ptr(keys), _ptr(vals), len(keys), e)


# ---- problem / particles / run -----------------------------------------------------------
class Problem:
    """Owns the numpy arrays an or_problem points at."""

    def __init__(self, cfg, density: np.ndarray, tables, max_events: int = 10**9):
        self.cfg = cfg
        self.density = np.ascontiguousarray(density, dtype=np.float64)
        self.tables = [np.ascontiguousarray(t, dtype=np.float64) for t in tables]
        sk, sv, ck, cv = self.tables
        self.c = _Problem(cfg.nx, cfg.ny, cfg.width, cfg.height, _ptr(self.density),
                          _ptr(sk), _ptr(sv), len(sk), _ptr(ck), _ptr(cv), len(ck),
                          cfg.A, cfg.molar_mass, cfg.e_min, cfg.w_min, max_events,
                          getattr(cfg, "boundary", 0), getattr(cfg, "analog", 0),
                          getattr(cfg, "roulette", 0), 0,
                          getattr(cfg, "roulette_weight", 0.0) or 2.0 * cfg.w_min)


class Particles:
    """SoA particle store (numpy), the oracle's or_particles."""

    FIELDS = _PFIELDS

    def __init__(self, n: int):
        self.n = n
        for name, dt in _PFIELDS:
            setattr(self, name, np.zeros(n, dtype=dt))

    def c(self) -> _Particles:
        return _Particles(*[_ptr(getattr(self, n)) for n, _ in _PFIELDS])

    def as_dict(self) -> dict:
        return {n: getattr(self, n) for n, _ in _PFIELDS}

    def copy(self) -> "Particles":
        p = Particles(self.n)
        for n, _ in _PFIELDS:
            getattr(p, n)[:] = getattr(self, n)
        return p


def stats_dict(s: _Stats) -> dict:
    return {n: getattr(s, n) for n, _ in _Stats._fields_}


def inject(prob: Problem, first_id: int, n_local: int, seed: int | None = None) -> Particles:
    cfg = prob.cfg
    p = Particles(n_local)
    sx, sy, sw, sh = cfg.source
    lib().or_inject(C.byref(prob.c), C.byref(p.c()), first_id, n_local, sx, sy, sw, sh,
                    cfg.e0, cfg.seed if seed is None else seed)
    return p


def step(prob: Problem, parts: Particles, first_id: int, tally: np.ndarray,
         seed: int | None = None, dt: float | None = None) -> dict:
    cfg = prob.cfg
    assert tally.dtype == np.float64 and tally.size == cfg.nx * cfg.ny
    st = _Stats()
    lib().or_step(C.byref(prob.c), C.byref(parts.c()), first_id, parts.n,
                  cfg.seed if seed is None else seed, cfg.dt if dt is None else dt,
                  _ptr(tally), C.byref(st))
    return stats_dict(st)


def run(cfg, first_id: int = 0, n_local: int | None = None, steps: int = 1,
        density: np.ndarray | None = None, tables=None, max_events: int = 10**9):
    """Inject ids [first_id, first_id+n_local) and run `steps` timesteps.

    Returns (tally of the last step [ny][nx], particles, list of per-step stats)."""
    from paper_conf_cluster_martineaum17_b200 import workloads as wl
    if n_local is None:
        n_local = cfg.n_particles - first_id
    prob = Problem(cfg, wl.density(cfg) if density is None else density,
                   wl.tables(cfg) if tables is None else tables, max_events)
    parts = inject(prob, first_id, n_local)
    all_stats = []
    tally = None
    for _ in range(steps):
        tally = np.zeros((cfg.ny, cfg.nx))
        all_stats.append(step(prob, parts, first_id, tally))
    return tally, parts, all_stats
