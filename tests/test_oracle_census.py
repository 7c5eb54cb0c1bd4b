"""Pins for the oracle's census clock and census carry-over (R21, R23).

A timestep ends for a particle at census, when its elapsed flight time reaches dt
(§IV-A: "the particle will be stored until the next timestep"); the event timers
are "updated … to account for the distance travelled".  The oracle keeps the
census timer as a distance (R21) and converts it through time at every collision, where the
speed changes; a census particle keeps its remaining number of mean free paths into the
next timestep (R23).  Three facts fix these steps independently of how the oracle writes
them:

* flight-time ledger: the sum over a history's segments of length / speed -- the oracle's
  instrument ``tfl``, fed back into nothing -- equals k*dt at the k-th census, and is below
  it for a particle that died;
* first flight across a census: in a homogeneous pure absorber (every particle dies at its
  first collision) the path length to that collision is Exp(Sigma_t) (P6) whether or not the
  particle waited at a census on the way -- the memoryless flight law holds only
  if the census carries the n_mfp left over;
* splitting a timestep: census is a pause, not an event of the physics, so two steps of dt
  and one step of 2*dt give the same histories (same collisions, energies, weights and
  facets; positions to rounding) and the same deposited energy per cell.

Mutations that these catch (each checked while writing them): dropping the census-timer
conversion at a collision (``dcen = tcen * v``), dropping the census n_mfp update, and
computing the census timer from the pre-collision speed.
"""
import math

import numpy as np
import pytest
from scipy import stats

from paper_conf_cluster_martineaum17_b200 import workloads as wl

N_A = 6.02214076e23
BARN = 1e-28
EV_J = 1.602176634e-19
M_N = 1.67492749804e-27


def _speed(e_ev):
    return math.sqrt(2.0 * e_ev * EV_J / M_N)


def _run(orc, cfg, dts, seed=None):
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    p = orc.inject(prob, 0, cfg.n_particles, seed=seed)
    tallies, sts = [], []
    for dt in dts:
        t = np.zeros(cfg.nx * cfg.ny)
        sts.append(orc.step(prob, p, 0, t, seed=seed, dt=dt))
        tallies.append(t)
    return p, tallies, sts


@pytest.mark.parametrize("cfgname", ["tiny_mid", "tiny_thin", "tiny_mid_bc", "tiny_csp", "small_csp"])
def test_census_flight_time_ledger(orc, cfgname):
    cfg = wl.CONFIGS[cfgname]
    if cfgname == "small_csp":
        cfg = cfg.with_(n_particles=800)
    for k in (1, 2, 3):
        p, _, _ = _run(orc, cfg, [cfg.dt] * k)
        alive = p.status == 1
        assert alive.sum() > 50
        # the conversion through a collision is exercised: census particles that collided
        assert (p.ncol[alive] > 0).sum() > 50
        err = np.abs(p.tfl[alive] - k * cfg.dt)
        assert err.max() <= 1e-12 * k * cfg.dt, (cfgname, k, err.max() / cfg.dt)
        # a particle that died stopped before the end of the step it died in
        assert np.all(p.tfl[~alive] <= k * cfg.dt * (1 + 1e-12))
        assert np.all(p.tfl[~alive] >= 0.0)


def test_census_flight_time_single_group_speed_law(orc):
    """The ledger itself, on vacuum: no collisions, so tfl * v0 is the straight-line path
    length v0 * dt, which the vacuum closed form (P4) also fixes."""
    cfg = wl.CONFIGS["tiny_vacuum"]
    p, _, _ = _run(orc, cfg, [cfg.dt, cfg.dt])
    assert np.all(p.status == 1) and np.all(p.ncol == 0)
    assert np.max(np.abs(p.tfl * _speed(cfg.e0) - 2 * cfg.dt * _speed(cfg.e0))) <= 1e-12


# pure absorber (1 - p_a < w_min: the first collision kills), Sigma_t * v0 * dt ~ 1, so
# about e^-1 of the particles wait at the first census before colliding
_ABS = wl.CONFIGS["tiny_absorber"].with_(name="census_absorber", rho=6.0e-4, n_particles=20000)


def _sigma_t(cfg):
    t = cfg.tables
    return cfg.rho * N_A / cfg.molar_mass * (t.sigma_s_1g + t.sigma_a_1g) * BARN


@pytest.mark.parametrize("seed", [51, 52])
def test_first_flight_exponential_across_census(orc, seed):
    cfg = _ABS
    sig = _sigma_t(cfg)
    L = _speed(cfg.e0) * cfg.dt
    assert 0.7 < sig * L < 1.5
    p, _, sts = _run(orc, cfg, [cfg.dt] * 8, seed=seed)
    waited = sts[0]["n_census"] / cfg.n_particles
    assert abs(waited - math.exp(-sig * L)) < 0.02          # first census reached
    assert sts[1]["n_alive_start"] == sts[0]["n_census"] > 0.3 * cfg.n_particles
    dead = p.status == 0
    assert dead.mean() > 0.995 and np.all(p.ncol[dead] == 1)
    # path to the (only) collision: speed is E0's until then
    ell = p.tfl[dead] * _speed(cfg.e0)
    assert stats.kstest(ell * sig, "expon").pvalue > 1e-3
    # the conditional law past the first census: memoryless
    late = ell > L
    assert late.mean() > 0.3
    assert stats.kstest((ell[late] - L) * sig, "expon").pvalue > 1e-3


@pytest.mark.parametrize("cfgname", ["tiny_mid", "tiny_thin", "tiny_csp", "tiny_split", "tiny_mid_bc"])
def test_split_timestep_invariance(orc, cfgname):
    cfg = wl.CONFIGS[cfgname]
    a, ta, sa = _run(orc, cfg, [cfg.dt, cfg.dt])
    b, tb, sb = _run(orc, cfg, [2 * cfg.dt])
    assert sa[0]["n_census"] > 50 and (a.ncol[a.ncen > 0] > 0).sum() > 20
    same = (a.ncol == b.ncol) & (a.nfac == b.nfac) & (a.status == b.status)
    # histories equal up to near-ties decided by rounding at the split point
    assert same.mean() >= 0.995, same.mean()
    assert np.array_equal(a.ctr[same], b.ctr[same])
    assert np.array_equal(a.e[same], b.e[same])
    assert np.array_equal(a.w[same], b.w[same])
    live = same & (a.status == 1)
    assert np.max(np.abs(a.x[live] - b.x[live])) <= 1e-9
    assert np.max(np.abs(a.y[live] - b.y[live])) <= 1e-9
    assert np.max(np.abs(a.tfl[same] - b.tfl[same])) <= 1e-12 * 2 * cfg.dt
    # a census costs one census event; nothing else
    na, nb = a.ncen[same].astype(np.int64), b.ncen[same].astype(np.int64)
    assert np.array_equal(na - nb, (na >= 1).astype(np.int64))
    # deposited energy: the two step tallies add up to the single-step tally
    ta2 = ta[0] + ta[1]
    assert abs(ta2.sum() - tb[0].sum()) <= 1e-6 * abs(tb[0].sum())
    dep_rel = np.abs(a.dep[same] - b.dep[same]) / np.maximum(np.abs(b.dep[same]), 1e-300)
    assert np.quantile(dep_rel, 0.99) <= 1e-9
