"""Pins P3 (injection), P4 (vacuum closed form), P5 (population) for the oracle.

P4 (§IV-C; reflective boundaries P:240-242): with density 0 a
particle flies a straight line of length L = v dt in the "unfolded" plane; the number
of facets it crosses is |floor(X/dx) - floor(x0/dx)| + |floor(Y/dy) - floor(y0/dy)| and
its final position is the unfolded end point folded back into [0, W] by reflection.
"""
import math

import numpy as np
import pytest
from scipy import stats

from paper_conf_cluster_martineaum17_b200 import workloads as wl

# Physical constants written independently of the oracle (SI 2019 / CODATA 2018).
EV_J = 1.602176634e-19
M_N = 1.67492749804e-27


def _speed(e_ev):
    return math.sqrt(2.0 * e_ev * EV_J / M_N)


def test_edges_and_cell_of_brute_force(orc):
    rng = np.random.default_rng(1)
    for n, ext in [(1, 1.0), (7, 1.0), (64, 1.0), (4000, 1.0), (13, 2.5)]:
        edges = [(i * ext) / n for i in range(n + 1)]
        assert edges[0] == 0.0 and edges[-1] == ext
        for i in range(n + 1):
            assert orc.edge(i, ext, n) == edges[i]
        qs = list(rng.uniform(0, ext, 300)) + edges + [np.nextafter(e, 0) for e in edges[1:]]
        for q in qs:
            brute = [i for i in range(n) if edges[i] <= q < edges[i + 1]]
            want = brute[0] if brute else n - 1          # q == W -> last cell
            assert orc.cell_of(q, ext, n) == want


def test_injection_geometry(orc):
    cfg = wl.CONFIGS["tiny_csp"].with_(n_particles=20000)
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    p = orc.inject(prob, 0, cfg.n_particles)
    sx, sy, sw, sh = cfg.source
    assert np.all((p.x >= sx) & (p.x <= sx + sw) & (p.y >= sy) & (p.y <= sy + sh))
    ex = np.array([(i * cfg.width) / cfg.nx for i in range(cfg.nx + 1)])
    assert np.all(ex[p.cx] <= p.x) and np.all(p.x < ex[p.cx + 1])
    ey = np.array([(i * cfg.height) / cfg.ny for i in range(cfg.ny + 1)])
    assert np.all(ey[p.cy] <= p.y) and np.all(p.y < ey[p.cy + 1])
    assert np.max(np.abs(np.hypot(p.ox, p.oy) - 1.0)) <= 4 * 2.0**-52
    # uniform position, uniform angle, Exp(1) mean free paths
    assert stats.kstest((p.x - sx) / sw, "uniform").pvalue > 1e-4
    assert stats.kstest((p.y - sy) / sh, "uniform").pvalue > 1e-4
    th = np.mod(np.arctan2(p.oy, p.ox), 2 * np.pi) / (2 * np.pi)
    assert stats.kstest(th, "uniform").pvalue > 1e-4
    assert stats.kstest(p.mfp, "expon").pvalue > 1e-4
    assert np.all(p.e == cfg.e0) and np.all(p.w == 1.0) and np.all(p.ctr == 2)
    assert np.all(p.status == 1)
    # the same id gives the same particle regardless of the range it is injected in
    q = orc.inject(prob, 777, 50)
    assert np.array_equal(q.x, p.x[777:827]) and np.array_equal(q.oy, p.oy[777:827])


def _fold(u, ext):
    m = np.mod(u, 2 * ext)
    return np.where(m <= ext, m, 2 * ext - m)


@pytest.mark.parametrize("name", ["tiny_vacuum", "tiny_vacuum_lo"])
def test_vacuum_closed_form(orc, name):
    cfg = wl.CONFIGS[name]
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    p0 = orc.inject(prob, 0, cfg.n_particles)
    p = p0.copy()
    tally = np.zeros((cfg.ny, cfg.nx))
    st = orc.step(prob, p, 0, tally)
    L = _speed(cfg.e0) * cfg.dt
    dx, dy = cfg.width / cfg.nx, cfg.height / cfg.ny
    X = p0.x + L * p0.ox
    Y = p0.y + L * p0.oy
    fx = np.abs(np.floor(X / dx) - np.floor(p0.x / dx))
    fy = np.abs(np.floor(Y / dy) - np.floor(p0.y / dy))
    # exclude near-ties: end point within 1e-9 cell of a grid line
    ok = ((np.abs(X / dx - np.round(X / dx)) > 1e-9) & (np.abs(Y / dy - np.round(Y / dy)) > 1e-9))
    assert ok.mean() > 0.99
    assert np.array_equal(p.nfac[ok], (fx + fy)[ok].astype(np.uint32))
    assert np.all(p.ncol == 0) and np.all(p.ncen == 1) and np.all(p.status == 1)
    assert np.max(np.abs(p.x - _fold(X, cfg.width))[ok]) < 1e-12
    assert np.max(np.abs(p.y - _fold(Y, cfg.height))[ok]) < 1e-12
    assert np.array_equal(np.abs(p.ox), np.abs(p0.ox)) and np.array_equal(np.abs(p.oy), np.abs(p0.oy))
    # direction sign flips once per reflection: parity of wall hits
    nrefx = np.abs(np.floor(X / cfg.width))
    assert np.array_equal(np.sign(p.ox)[ok], (np.sign(p0.ox) * (-1.0) ** nrefx)[ok])
    assert st["n_census"] == cfg.n_particles and st["n_killed"] == 0
    assert st["n_facets"] == int(p.nfac.sum())
    # mean facets per particle = L (4/pi) nx / W for isotropic 2D directions
    assert abs(p.nfac.mean() - L * 4 / np.pi * cfg.nx / cfg.width) < 5 * p.nfac.std() / np.sqrt(cfg.n_particles)
    if cfg.density == "zero":
        assert np.all(tally == 0.0) and np.all(p.dep == 0.0)
    else:
        assert np.all(tally >= 0.0)


def test_population_and_counters(orc):
    """P5: reflective boundaries conserve the population."""
    for name in ["tiny_csp", "tiny_split", "tiny_stream"]:
        cfg = wl.CONFIGS[name]
        tally, p, sts = orc.run(cfg, steps=2)
        s0, s1 = sts
        assert s0["n_alive_start"] == cfg.n_particles
        assert s0["n_census"] + s0["n_killed"] == s0["n_alive_start"]
        assert s1["n_alive_start"] == s0["n_census"]
        assert s1["n_census"] + s1["n_killed"] == s1["n_alive_start"]
        assert int(p.ncen.sum()) == s0["n_census"] + s1["n_census"]
        assert int(p.ncol.sum()) == s0["n_collisions"] + s1["n_collisions"]
        assert int(p.nfac.sum()) == s0["n_facets"] + s1["n_facets"]
        assert np.array_equal(p.ctr.astype(np.int64), 2 + p.ncol.astype(np.int64))  # R11
        assert np.all((p.status == 1) == (p.ncen == 2))
        assert s0["n_nonfinite"] == 0 and s0["n_xs_range"] == 0 and s0["n_event_cap"] == 0
        assert np.all((p.x >= 0) & (p.x <= cfg.width) & (p.y >= 0) & (p.y <= cfg.height))


def test_sharding_invariance(orc):
    """Per-particle results depend only on the global id; tallies add."""
    cfg = wl.CONFIGS["tiny_csp"]
    t_all, p_all, _ = orc.run(cfg)
    parts, tallies = [], []
    for r in range(3):
        lo, n = wl.shard(cfg.n_particles, r, 3)
        t, p, _ = orc.run(cfg, first_id=lo, n_local=n)
        parts.append(p)
        tallies.append(t)
    for name, _ in orc.Particles.FIELDS:
        cat = np.concatenate([getattr(p, name) for p in parts])
        assert np.array_equal(cat, getattr(p_all, name)), name
    tsum = tallies[0] + tallies[1] + tallies[2]
    assert np.allclose(tsum, t_all, rtol=1e-12, atol=0)


def test_facet_axis_tie_goes_to_y(orc):
    """Reading R16 (Listing 1 order; X-facet iff tx < ty): a particle
    whose two facet distances are exactly equal crosses Y first, then X at distance ~0 (a
    corner is two facets, R17).  Constructed input: a cell centre, direction (s, s)."""
    cfg = wl.CONFIGS["tiny_vacuum"]
    dx = cfg.width / cfg.nx
    s = math.sqrt(0.5)
    for cap, want in [(1, (3, 4, 1)), (2, (4, 4, 2))]:
        prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg), max_events=cap)
        p = orc.Particles(4)
        for k, (c0, ox, oy) in enumerate([(3, s, s), (3, -s, -s), (3, s, -s), (3, -s, s)]):
            p.x[k] = p.y[k] = (c0 + 0.5) * dx
            p.cx[k] = p.cy[k] = c0
            p.ox[k], p.oy[k] = ox, oy
            p.e[k], p.w[k], p.mfp[k], p.ctr[k], p.status[k] = cfg.e0, 1.0, 1.0, 2, 1
        orc.step(prob, p, 0, np.zeros(cfg.nx * cfg.ny))
        assert np.all(p.nfac == want[2])
        # k = 0 moves +x +y: after the tie the first crossing is Y
        assert (p.cx[0], p.cy[0]) == (want[0], want[1])
        if cap == 1:
            assert np.array_equal(p.cx, [3, 3, 3, 3])
            assert np.array_equal(p.cy, [4, 2, 2, 4])
