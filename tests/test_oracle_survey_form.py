"""The oracle's timer readings (R21, R22) against SURVEY §8(c)'s literal form.

SURVEY §8(c) writes the census timer as a remaining time t_rem (d_census = v * t_rem,
t_rem -= d / v after every segment) and the facet distance as a division
((edge - x) / omega).  The oracle keeps the census timer as a distance,
converted through time only at a collision (R21: "individual timers for each
event ... updated ... to account for the distance travelled"), and multiplies by a cached
1/omega (R22).  The two forms are the same real-number algorithm; they differ only in
rounding.  This test runs §8(c) as written -- a small pure-Python tracker that shares no
arithmetic with the oracle; it calls the oracle only for Threefry, whose words are pinned
by published KATs (test_oracle_rng) -- and requires the same histories: identical event
counts, energies and weights for all but near-tie particles, positions to rounding.
"""
import math

import numpy as np
import pytest

from paper_conf_cluster_martineaum17_b200 import workloads as wl

N_A = 6.02214076e23
EV = 1.602176634e-19
M_N = 1.67492749804e-27
BARN = 1.0e-28


def _u(x):
    return float((x >> 11) | 1) * 2.0 ** -53


def _track_survey(orc, cfg, p0, i, pid, dens):
    """SURVEY §8(c) STEP(p, dt) for one particle, single-group tables (sigma constant)."""
    nx, ny, W, H = cfg.nx, cfg.ny, cfg.width, cfg.height
    t = cfg.tables
    A = cfg.A
    x, y, ox, oy = p0.x[i], p0.y[i], p0.ox[i], p0.oy[i]
    E, w, mfp = p0.e[i], p0.w[i], p0.mfp[i]
    cx, cy, c = int(p0.cx[i]), int(p0.cy[i]), int(p0.ctr[i])
    ex = lambda k: (k * W) / nx  # noqa: E731
    ey = lambda k: (k * H) / ny  # noqa: E731
    cn = N_A / cfg.molar_mass
    sig_t = t.sigma_s_1g + t.sigma_a_1g
    p_a = t.sigma_a_1g / sig_t
    speed = lambda e: math.sqrt(((2.0 * e) * EV) / M_N)  # noqa: E731
    n = dens[cy, cx] * cn
    St = (n * sig_t) * BARN
    v = speed(E)
    t_rem = cfg.dt
    nf = nc = 0
    while True:
        tx = (ex(cx + 1) - x) / ox if ox > 0 else ((ex(cx) - x) / ox if ox < 0 else math.inf)
        tx = max(tx, 0.0)
        ty = (ey(cy + 1) - y) / oy if oy > 0 else ((ey(cy) - y) / oy if oy < 0 else math.inf)
        ty = max(ty, 0.0)
        axis_x = tx < ty
        d_f = tx if axis_x else ty
        d_c = mfp / St if St > 0 else math.inf
        d_s = v * t_rem
        if d_c < d_f and d_c < d_s:
            x = x + d_c * ox
            y = y + d_c * oy
            t_rem = max(0.0, t_rem - d_c / v)
            a, b = orc.threefry2x64_20(c, 0, pid, cfg.seed)
            c += 1
            nc += 1
            w = w * (1.0 - p_a)
            mu = 1.0 - 2.0 * _u(a)
            E2 = E * (((A * A + (2.0 * A) * mu) + 1.0) / ((A + 1.0) * (A + 1.0)))
            ct = 0.5 * ((A + 1.0) * math.sqrt(E2 / E) - (A - 1.0) * math.sqrt(E / E2))
            st = (-1.0 if a & 1 else 1.0) * math.sqrt(max(0.0, 1.0 - ct * ct))
            ox, oy = ox * ct - oy * st, ox * st + oy * ct
            E = E2
            if E < cfg.e_min or w < cfg.w_min:
                return dict(nfac=nf, ncol=nc, ctr=c, status=0, e=E, w=w, x=x, y=y, cx=cx, cy=cy)
            v = speed(E)
            mfp = -math.log(_u(b))
        elif d_f < d_s:
            mfp = max(0.0, mfp - d_f * St)
            t_rem = max(0.0, t_rem - d_f / v)
            if axis_x:
                y = y + d_f * oy
                x = ex(cx + 1) if ox > 0 else ex(cx)
                if ox > 0:
                    if cx == nx - 1:
                        ox = -ox
                    else:
                        cx += 1
                else:
                    if cx == 0:
                        ox = -ox
                    else:
                        cx -= 1
            else:
                x = x + d_f * ox
                y = ey(cy + 1) if oy > 0 else ey(cy)
                if oy > 0:
                    if cy == ny - 1:
                        oy = -oy
                    else:
                        cy += 1
                else:
                    if cy == 0:
                        oy = -oy
                    else:
                        cy -= 1
            nf += 1
            n = dens[cy, cx] * cn
            St = (n * sig_t) * BARN
        else:
            x = x + d_s * ox
            y = y + d_s * oy
            return dict(nfac=nf, ncol=nc, ctr=c, status=1, e=E, w=w, x=x, y=y, cx=cx, cy=cy)


@pytest.mark.parametrize("cfgname,n", [("tiny_mid", 1000), ("tiny_thin", 1000), ("tiny_csp", 1000),
                                       ("tiny_split", 1000)])
def test_oracle_matches_survey_literal_form(orc, cfgname, n):
    cfg = wl.CONFIGS[cfgname]
    if cfg.tables.kind != "1g":
        cfg = cfg.with_(tables=wl.Tables(kind="1g", n_scatter=2, n_capture=2))
    dens = wl.density(cfg)
    prob = orc.Problem(cfg, dens, wl.tables(cfg))
    p0 = orc.inject(prob, 0, n)
    p = p0.copy()
    orc.step(prob, p, 0, np.zeros(cfg.nx * cfg.ny))
    same = 0
    for i in range(n):
        r = _track_survey(orc, cfg, p0, i, i, dens)
        ok = (r["nfac"] == p.nfac[i] and r["ncol"] == p.ncol[i] and r["ctr"] == p.ctr[i]
              and r["status"] == p.status[i] and r["cx"] == p.cx[i] and r["cy"] == p.cy[i])
        if ok:
            same += 1
            assert r["e"] == p.e[i] and r["w"] == p.w[i]
            assert abs(r["x"] - p.x[i]) <= 1e-9 and abs(r["y"] - p.y[i]) <= 1e-9
    assert same >= n - 2, (same, n)                     # near-ties only (none seen)
