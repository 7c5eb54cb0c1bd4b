"""Pin P18 for the oracle: the per-cell tally of streaming particles is the track-length
estimator of the paper, cell by cell.

Between two events a particle deposits w * d * Sigma_t * H into the cell it crosses and
flushes the deposit when it leaves the cell (§IV-A P:159-166 and §V-D P:429-439,
"energy deposition ... tallied at each facet").  In a homogeneous, almost empty medium
(rho = 1e-30, tiny_vacuum_lo) no particle collides, so E, w, Sigma_t and H stay constant
and every cell's tally must equal one constant times the total length of the straight,
wall-reflected paths inside that cell (reflective boundaries).  The path
lengths per cell are computed here by plain geometry, independently of the oracle: each
path is unfolded into a straight segment of length L = v dt in the mirrored plane
 and cut at every grid line.  A deposit flushed into the wrong cell, a
dropped or doubled segment, a wrong segment length or a lost census deposit breaks the
proportionality in some cells.
"""
import math

import numpy as np

from paper_conf_cluster_martineaum17_b200 import workloads as wl

EV_J = 1.602176634e-19      # SI 2019
M_N = 1.67492749804e-27     # CODATA 2018


def _chords(x0, y0, ox, oy, L, nx, ny, W, H):
    """Per-cell path length [ny][nx] of the reflected straight path of length L."""
    dx, dy = W / nx, H / ny
    ts = [0.0, L]
    if ox != 0.0:
        xe = x0 + L * ox
        lo, hi = sorted((x0, xe))
        ts += [(i * dx - x0) / ox for i in range(math.floor(lo / dx) + 1, math.ceil(hi / dx))]
    if oy != 0.0:
        ye = y0 + L * oy
        lo, hi = sorted((y0, ye))
        ts += [(j * dy - y0) / oy for j in range(math.floor(lo / dy) + 1, math.ceil(hi / dy))]
    ts = np.unique(np.clip(np.array(ts), 0.0, L))
    mid = 0.5 * (ts[1:] + ts[:-1])
    seg = ts[1:] - ts[:-1]
    ux, uy = x0 + mid * ox, y0 + mid * oy                  # unfolded midpoints
    iu, ju = np.floor(ux / dx).astype(np.int64), np.floor(uy / dy).astype(np.int64)
    kx, rx = np.divmod(iu, nx)
    ky, ry = np.divmod(ju, ny)
    cx = np.where(kx % 2 == 0, rx, nx - 1 - rx)            # fold the mirrored copies back
    cy = np.where(ky % 2 == 0, ry, ny - 1 - ry)
    out = np.zeros((ny, nx))
    np.add.at(out, (cy, cx), seg)
    return out


def test_streaming_tally_is_track_length_per_cell(orc):
    cfg = wl.CONFIGS["tiny_vacuum_lo"].with_(n_particles=400)
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    p0 = orc.inject(prob, 0, cfg.n_particles)
    p = p0.copy()
    tally = np.zeros((cfg.ny, cfg.nx))
    st = orc.step(prob, p, 0, tally)
    assert st["n_collisions"] == 0 and st["n_census"] == cfg.n_particles
    L = math.sqrt(2.0 * cfg.e0 * EV_J / M_N) * cfg.dt
    chord = np.zeros_like(tally)
    for k in range(cfg.n_particles):
        chord += _chords(p0.x[k], p0.y[k], p0.ox[k], p0.oy[k], L, cfg.nx, cfg.ny, cfg.width, cfg.height)
    assert abs(chord.sum() - cfg.n_particles * L) <= 1e-9 * cfg.n_particles * L
    hit = chord > 0
    assert hit.mean() > 0.5                                 # the paths cover most of the mesh
    assert np.all(tally[~hit] == 0.0)                       # no deposit where no path runs
    c = tally.sum() / chord.sum()                           # Sigma_t * H * w, one constant
    assert c > 0
    rel = np.abs(tally[hit] - c * chord[hit]) / (c * chord[hit])
    assert rel.max() < 1e-9, rel.max()
    # the particles' own deposit ledgers add up to the tally
    assert abs(p.dep.sum() - tally.sum()) <= 1e-12 * tally.sum()
