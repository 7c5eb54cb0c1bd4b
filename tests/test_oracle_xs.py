"""Pin P9: microscopic cross-section lookup (§IV-D).

"a search is performed to find the energy bin for the particle's continuous energy,
and a linear interpolation gives an accurate approximation" -- checked against a
brute-force linear scan for the bin on random tiny tables, at keys, at the end points,
and on linear data (where interpolation must reproduce the line).
"""
import numpy as np
from hypothesis import given, settings, strategies as st

from paper_conf_cluster_martineaum17_b200 import workloads as wl


def _brute_bin(keys, e):
    n = len(keys)
    cand = [i for i in range(n - 1) if keys[i] <= e]
    return max(cand) if cand else 0


@settings(max_examples=200, deadline=None)
@given(st.integers(2, 64), st.integers(0, 2**32 - 1))
def test_bin_matches_brute_force(orc, n, seed):
    rng = np.random.default_rng(seed)
    keys, vals = wl.random_tables(rng, n)
    es = list(rng.uniform(keys[0], keys[-1], 20)) + list(keys)
    for e in es:
        i = orc.xs_index(keys, e)
        assert i == _brute_bin(keys, e)
        assert keys[i] <= e and (e < keys[i + 1] or (i == n - 2 and e == keys[-1]))


def test_values_at_keys_and_linear_data(orc):
    rng = np.random.default_rng(5)
    keys, vals = wl.random_tables(rng, 40)
    for k, v in zip(keys[:-1], vals[:-1]):
        assert orc.xs_lookup(keys, vals, k) == v            # t = 0: sigma(k[i]) = v[i] exactly
    # top key lands in the last bin with t = 1: v[N-2] + (v[N-1] - v[N-2]) rounds within ulps
    assert abs(orc.xs_lookup(keys, vals, keys[-1]) - vals[-1]) <= 4 * np.spacing(max(vals[-2:]))
    a, b = 3.0, -0.25
    lin = a + b * keys
    for e in rng.uniform(keys[0], keys[-1], 200):
        assert abs(orc.xs_lookup(keys, lin, e) - (a + b * e)) < 1e-12
    # interpolated value lies between neighbouring table values
    for e in rng.uniform(keys[0], keys[-1], 200):
        i = orc.xs_index(keys, e)
        s = orc.xs_lookup(keys, vals, e)
        assert min(vals[i], vals[i + 1]) - 1e-12 <= s <= max(vals[i], vals[i + 1]) + 1e-12


def test_paper_tables_shape():
    cfg = wl.CONFIGS["csp"]
    sk, sv, ck, cv = wl.tables(cfg)
    assert len(sk) == 65536 and len(ck) == 49152          # two tables, different grids
    assert np.all(np.diff(sk) > 0) and np.all(np.diff(ck) > 0)
    assert sk[0] <= cfg.e_min and sk[-1] >= cfg.e0 and ck[0] <= cfg.e_min and ck[-1] >= cfg.e0
    assert np.all(sv > 0) and np.all(cv > 0)
