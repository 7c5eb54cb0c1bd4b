"""Seeded synthetic input generators shared by the CUDA path, the oracle tests and bench.py.

This module holds NO arithmetic of the method: only problem definitions (mesh sizes,
density maps, source rectangles, particle counts, seeds) and the synthetic
cross-section tables.  It imports neither ``oracle`` nor the CUDA binding.

Workload recipe, following the paper's test problems
(§IV-B):

* stream  -- rho = 1e-30 kg/m^3 everywhere, source in the centre,
  1e6 particles; ~7000 facets per particle.
* scatter -- rho = 1e3 kg/m^3 everywhere, 1e7 particles; most
  particles never leave their birth cell.
* csp     -- low density except a dense centre square, source bottom-left
  (P:208-211), 1e6 particles.
* split   -- BASELINE.json's two-region problem (not in the paper): dense for x < W/2.
* All use a 4000^2 mesh and dt = 1e-7 s.

Cross-section tables are "dummy data" mimicking capture and scatter:
scatter sigma_s(E) = 2000 (1 + 0.2 sin(3 ln E)) b on 65536 log-spaced keys, capture
sigma_a(E) = 200 E^-1/2 b (1/v law) on 49152 log-spaced keys over [1e-5, 2e7] eV.
"""
from __future__ import annotations

import dataclasses
from dataclasses import dataclass, field

import numpy as np

# Problem constants (DESIGN.md §4 readings).  Physical constants of the method live
# separately in oracle/ and csrc/; these are only the problem's inputs.
WIDTH = 1.0          # m  (reading R2: pins ~7000 facets/particle)
HEIGHT = 1.0
E0 = 1.0e6           # eV (reading R3)
DT = 1.0e-7          # s
RHO_LO = 1.0e-30     # kg/m^3
RHO_HI = 1.0e3       # kg/m^3
A_DEFAULT = 1.0
MOLAR_MASS = 1.0e-3  # kg/mol
E_MIN = 1.0          # eV (reading R6)
W_MIN = 1.0e-3       # (reading R7)
KEY_LO, KEY_HI = 1.0e-5, 2.0e7


@dataclass(frozen=True)
class Tables:
    kind: str = "paper"          # "paper" (log-spaced synthetic) or "1g" (single group)
    n_scatter: int = 65536
    n_capture: int = 49152
    sigma_s_1g: float = 2000.0   # barns, single-group tables only
    sigma_a_1g: float = 200.0


@dataclass(frozen=True)
class Config:
    name: str
    nx: int
    ny: int
    density: str                 # "csp" | "uniform_lo" | "uniform_hi" | "split" | "zero"
    source: tuple                # (x, y, w, h) in metres
    n_particles: int
    seed: int
    tables: Tables = field(default_factory=Tables)
    width: float = WIDTH
    height: float = HEIGHT
    dt: float = DT
    e0: float = E0
    A: float = A_DEFAULT
    molar_mass: float = MOLAR_MASS
    e_min: float = E_MIN
    w_min: float = W_MIN
    rho: float = RHO_HI          # density of the "uniform" map
    # physics variants (R30-R32)
    boundary: int = 0            # 0 reflective, 1 vacuum (escape)
    analog: int = 0              # 0 implicit capture, 1 sampled absorption
    roulette: int = 0            # 0 hard w_min kill, 1 Russian roulette
    roulette_weight: float = 0.0  # survivor weight (0 -> 2 w_min)

    def with_(self, **kw) -> "Config":
        return dataclasses.replace(self, **kw)


_SINGLE = Tables(kind="1g", n_scatter=2, n_capture=2)

CONFIGS: dict[str, Config] = {
    # BASELINE.json configs[0..4]
    "tiny_csp": Config("tiny_csp", 64, 64, "csp", (0.0, 0.0, 0.1, 0.1), 1000, 1, _SINGLE),
    "csp": Config("csp", 4000, 4000, "csp", (0.0, 0.0, 0.1, 0.1), 1_000_000, 11),
    "stream": Config("stream", 4000, 4000, "uniform_lo", (0.45, 0.45, 0.1, 0.1), 1_000_000, 21),
    "stream_8m": Config("stream_8m", 4000, 4000, "uniform_lo", (0.45, 0.45, 0.1, 0.1), 1 << 23, 21),
    "scatter": Config("scatter", 4000, 4000, "uniform_hi", (0.45, 0.45, 0.1, 0.1), 10_000_000, 31),
    # scatter's atomic-contention sweep: source side 0.5 / 0.01 m
    "scatter_src050": Config("scatter_src050", 4000, 4000, "uniform_hi", (0.25, 0.25, 0.5, 0.5), 10_000_000, 32),
    "scatter_src001": Config("scatter_src001", 4000, 4000, "uniform_hi", (0.495, 0.495, 0.01, 0.01), 10_000_000, 33),
    "split": Config("split", 4000, 4000, "split", (0.0, 0.0, 1.0, 1.0), 1 << 23, 41),
    # test-only problems
    "tiny_vacuum": Config("tiny_vacuum", 64, 64, "zero", (0.4, 0.4, 0.2, 0.2), 1000, 3, _SINGLE),
    "tiny_vacuum_lo": Config("tiny_vacuum_lo", 64, 64, "uniform_lo", (0.4, 0.4, 0.2, 0.2), 1000, 4, _SINGLE),
    "tiny_scatter_1g": Config("tiny_scatter_1g", 64, 64, "uniform_hi", (0.4, 0.4, 0.2, 0.2), 10_000, 5, _SINGLE),
    "tiny_wkill": Config("tiny_wkill", 64, 64, "uniform_hi", (0.4, 0.4, 0.2, 0.2), 4000, 6,
                         Tables(kind="1g", n_scatter=2, n_capture=2, sigma_a_1g=20000.0)),
    "tiny_A12": Config("tiny_A12", 64, 64, "uniform_hi", (0.4, 0.4, 0.2, 0.2), 10_000, 7, _SINGLE, A=12.0),
    # mean free path ~ 1 cell: many facets inside matter (pins facet-side bookkeeping)
    "tiny_mid": Config("tiny_mid", 64, 64, "uniform", (0.4, 0.4, 0.2, 0.2), 10_000, 13, _SINGLE, rho=0.5),
    # pure absorber (1 - p_a < w_min): every history ends at its first collision, mfp ~ 3 cells
    "tiny_absorber": Config("tiny_absorber", 64, 64, "uniform", (0.4, 0.4, 0.2, 0.2), 10_000, 14,
                            Tables(kind="1g", n_scatter=2, n_capture=2, sigma_s_1g=1.0,
                                   sigma_a_1g=20000.0), rho=0.0177),
    # thin medium: mfp ~ 0.3 m at E0, so census segments carry high-energy deposits
    "tiny_thin": Config("tiny_thin", 64, 64, "uniform", (0.4, 0.4, 0.2, 0.2), 10_000, 15, _SINGLE, rho=0.02),
    # heterogeneous maps exercising the u16 and f64 density layouts
    "tiny_levels": Config("tiny_levels", 64, 64, "levels", (0.3, 0.3, 0.4, 0.4), 3000, 16, _SINGLE, rho=2.0),
    "small_random": Config("small_random", 300, 300, "random", (0.3, 0.3, 0.4, 0.4), 3000, 17, rho=2.0),
    "tiny_stream": Config("tiny_stream", 64, 64, "uniform_lo", (0.45, 0.45, 0.1, 0.1), 2000, 8),
    "tiny_split": Config("tiny_split", 64, 64, "split", (0.0, 0.0, 1.0, 1.0), 2000, 9),
    # a few materials in random rectangles on ragged meshes: u8 codes whose block map holds
    # both uniform and mixed blocks (block sides 4 and 8)
    "tiny_mosaic": Config("tiny_mosaic", 70, 50, "mosaic", (0.1, 0.1, 0.8, 0.8), 2000, 18, _SINGLE, rho=2.0),
    "small_mosaic": Config("small_mosaic", 601, 590, "mosaic", (0.2, 0.2, 0.6, 0.6), 3000, 19, rho=0.5),
    # every particle born in one cell of a dense medium: maximal tally contention
    "tiny_hotspot": Config("tiny_hotspot", 64, 64, "uniform_hi", (0.5, 0.5, 0.01, 0.01), 10_000, 20, _SINGLE),
    # physics variants
    "tiny_vacuum_bc": Config("tiny_vacuum_bc", 64, 64, "zero", (0.4, 0.4, 0.2, 0.2), 1000, 21, _SINGLE,
                             boundary=1),
    "tiny_mid_bc": Config("tiny_mid_bc", 64, 64, "uniform", (0.0, 0.4, 0.2, 0.2), 10_000, 22, _SINGLE,
                          rho=0.1, boundary=1),
    "tiny_analog": Config("tiny_analog", 64, 64, "uniform_hi", (0.4, 0.4, 0.2, 0.2), 10_000, 23, _SINGLE,
                          analog=1),
    "tiny_analog_mid": Config("tiny_analog_mid", 64, 64, "uniform", (0.0, 0.4, 0.2, 0.2), 10_000, 24, _SINGLE,
                              rho=0.1, analog=1, boundary=1),
    "tiny_roulette": Config("tiny_roulette", 64, 64, "uniform_hi", (0.4, 0.4, 0.2, 0.2), 4000, 25,
                            Tables(kind="1g", n_scatter=2, n_capture=2, sigma_a_1g=20000.0),
                            w_min=0.05, roulette=1, roulette_weight=0.2),
    "small_csp_variants": Config("small_csp_variants", 256, 256, "csp", (0.0, 0.0, 0.1, 0.1), 4096, 26,
                                 boundary=1, analog=1),
    "small_csp": Config("small_csp", 256, 256, "csp", (0.0, 0.0, 0.1, 0.1), 4096, 10),
    "small_scatter": Config("small_scatter", 256, 256, "uniform_hi", (0.45, 0.45, 0.1, 0.1), 8192, 12),
}


def density(cfg: Config) -> np.ndarray:
    """Cell-centred mass densities, f64 [ny][nx] row-major."""
    ny, nx = cfg.ny, cfg.nx
    xc = (np.arange(nx) + 0.5) * (cfg.width / nx)
    yc = (np.arange(ny) + 0.5) * (cfg.height / ny)
    if cfg.density == "zero":
        return np.zeros((ny, nx))
    if cfg.density == "uniform_lo":
        return np.full((ny, nx), RHO_LO)
    if cfg.density == "uniform_hi":
        return np.full((ny, nx), RHO_HI)
    if cfg.density == "uniform":
        return np.full((ny, nx), cfg.rho)
    if cfg.density == "levels":      # 1000 distinct levels in [0, rho]: u16 material codes
        rng = np.random.default_rng(cfg.seed)
        return rng.integers(0, 1000, (ny, nx)) * (cfg.rho / 1000.0)
    if cfg.density == "random":      # continuous random densities: no lossless code fits
        rng = np.random.default_rng(cfg.seed)
        return rng.uniform(0.0, cfg.rho, (ny, nx))
    if cfg.density == "mosaic":      # 12 random rectangles of 5 materials over rho_lo
        rng = np.random.default_rng(cfg.seed)
        levels = np.array([0.0, RHO_LO, 0.05 * cfg.rho, cfg.rho, 20.0 * cfg.rho])
        rho = np.full((ny, nx), RHO_LO)
        for _ in range(12):
            x0, y0 = rng.integers(0, nx), rng.integers(0, ny)
            w, h = rng.integers(1, max(2, nx // 3)), rng.integers(1, max(2, ny // 3))
            rho[y0:y0 + h, x0:x0 + w] = levels[rng.integers(0, len(levels))]
        return rho
    if cfg.density == "csp":
        inx = (xc >= 0.25 * cfg.width) & (xc <= 0.75 * cfg.width)
        iny = (yc >= 0.25 * cfg.height) & (yc <= 0.75 * cfg.height)
        rho = np.full((ny, nx), RHO_LO)
        rho[np.ix_(iny, inx)] = RHO_HI
        return rho
    if cfg.density == "split":
        rho = np.full((ny, nx), RHO_LO)
        rho[:, xc < 0.5 * cfg.width] = RHO_HI
        return rho
    raise ValueError(cfg.density)


def _log_keys(n: int) -> np.ndarray:
    k = np.geomspace(KEY_LO, KEY_HI, n)
    k[0], k[-1] = KEY_LO, KEY_HI
    assert np.all(np.diff(k) > 0)
    return k


def tables(cfg: Config):
    """(scatter_keys, scatter_vals, capture_keys, capture_vals), f64, barns."""
    t = cfg.tables
    if t.kind == "1g":
        k = np.array([KEY_LO, KEY_HI])
        return k.copy(), np.full(2, t.sigma_s_1g), k.copy(), np.full(2, t.sigma_a_1g)
    ks = _log_keys(t.n_scatter)
    ka = _log_keys(t.n_capture)
    vs = 2000.0 * (1.0 + 0.2 * np.sin(3.0 * np.log(ks)))
    va = 200.0 / np.sqrt(ka)
    return ks, vs, ka, va


def shard(n_total: int, rank: int, world: int) -> tuple[int, int]:
    """Rank r owns global ids [floor(rN/P), floor((r+1)N/P)) -> (first_id, n_local)."""
    lo = (rank * n_total) // world
    hi = ((rank + 1) * n_total) // world
    return lo, hi - lo


def random_tables(rng: np.random.Generator, n: int):
    """Random tiny strictly-increasing tables for lookup tests."""
    k = np.sort(rng.uniform(0.0, 10.0, n))
    while np.any(np.diff(k) <= 0):
        k = np.sort(rng.uniform(0.0, 10.0, n))
    v = rng.uniform(0.0, 5.0, n)
    return k, v
