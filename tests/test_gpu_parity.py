"""GPU parity: the CUDA path (through the C ABI) against the oracle, element by element.

Runs on a B200 (`pytest -m gpu` via gpurun).  Sizes: tiny/small problems the oracle
finishes in well under a second (several CTAs of particles, ragged tails), then the
BASELINE.json full-size configs in the launch configuration bench.py times, checked on
sampled particles the oracle recomputes one by one and by properties that hold at any
size.
"""
import math

import numpy as np
import pytest

from paper_conf_cluster_martineaum17_b200 import workloads as wl
from tests.parity import compare_particles, compare_stats, compare_tally

pytestmark = pytest.mark.gpu

MODES = ["history", "event"]


@pytest.fixture(scope="module")
def nt():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cluster_martineaum17_b200 import binding, build
    build.build()
    return binding


def _gpu_run(nt, cfg, steps=1, first_id=0, n_local=None, **opts):
    t = nt.setup(cfg, first_id=first_id, n_local=n_local, **opts)
    stats = [t.run_timestep(cfg.dt) for _ in range(steps)]
    tally = t.read_tally()
    parts = t.read_particles()
    t.close()
    return tally, parts, stats


# ---------------------------------------------------------------------------------------------
def test_threefry_words_bit_exact(nt, orc):
    rng = np.random.default_rng(0)
    grid = [(c, 0, p, s) for c in range(0, 40) for p in (0, 1, 2, 999, 2**40 + 3) for s in (0, 11, 2**63)]
    rand = [tuple(int(v) for v in rng.integers(0, 2**64, 4, dtype=np.uint64)) for _ in range(2000)]
    inp = np.array(grid + rand, dtype=np.uint64)
    t = nt.Tracker()
    out = t.debug_threefry(inp)
    t.close()
    assert tuple(int(v) for v in out[0 * 0]) == orc.threefry2x64_20(*[int(v) for v in inp[0]])
    for row, o in zip(inp, out):
        assert tuple(int(v) for v in o) == orc.threefry2x64_20(*[int(v) for v in row])


@pytest.mark.parametrize("xs_search", [0, 1, 3, 4])
@pytest.mark.parametrize("cfgname", ["csp", "tiny_csp"])
def test_xs_lookup_matches_oracle(nt, orc, cfgname, xs_search):
    cfg = wl.CONFIGS[cfgname]
    sk, sv, ck, cv = wl.tables(cfg)
    t = nt.Tracker(xs_search=xs_search)
    t.init_mesh(4, 4, 1.0, 1.0, np.ones(16))
    t.load_cross_sections(sk, sv, ck, cv)
    rng = np.random.default_rng(3)
    es = np.concatenate([np.exp(rng.uniform(np.log(1e-5), np.log(2e7), 3000)), sk[:50], sk[-50:],
                         ck[::997], [sk[0], sk[-1], 1.0, 1e6]])
    gs, ga = t.debug_xs(es)
    if xs_search in (0, 4) and cfgname == "csp":
        assert t.xs_rows() == 7            # the paper tables get direct rows and the union grid
    t.close()
    for e, a, b in zip(es, gs, ga):
        assert a == orc.xs_lookup(sk, sv, e)
        assert b == orc.xs_lookup(ck, cv, e)


@pytest.mark.parametrize("xs_search", [0, 3, 4])
def test_xs_random_tables(nt, orc, xs_search):
    rng = np.random.default_rng(9)
    for n in [2, 3, 5, 17, 64, 1000]:
        k, v = wl.random_tables(rng, n)
        t = nt.Tracker(xs_search=xs_search)
        t.init_mesh(4, 4, 1.0, 1.0, np.ones(16))
        t.load_cross_sections(k, v, k, v[::-1].copy())
        es = np.concatenate([rng.uniform(k[0], k[-1], 300), k])
        gs, ga = t.debug_xs(es)
        t.close()
        for e, a, b in zip(es, gs, ga):
            assert a == orc.xs_lookup(k, v, e)
            assert b == orc.xs_lookup(k, v[::-1].copy(), e)


@pytest.mark.parametrize("xs_search", [0, 4])
def test_xs_tables_with_different_ranges(nt, orc, xs_search):
    """The unionised grid (0) over two tables with different, partly overlapping key ranges
    and densities: energies inside both ranges use the union rows, energies clamped by one
    table fall back to the per-table rows -- every lookup equals the oracle's binary search
    (P:252-265)."""
    rng = np.random.default_rng(21)
    ks = np.geomspace(1e-3, 1e3, 700)
    kc = np.geomspace(1e-1, 1e5, 3000)
    vs = rng.uniform(1.0, 3.0, ks.size)
    vc = rng.uniform(0.1, 9.0, kc.size)
    t = nt.Tracker(xs_search=xs_search)
    t.init_mesh(4, 4, 1.0, 1.0, np.ones(16))
    t.load_cross_sections(ks, vs, kc, vc)
    es = np.concatenate([np.exp(rng.uniform(np.log(1e-4), np.log(1e6), 4000)), ks, kc[::7],
                         [1e-3, 1e-1, 1e3, 1e5, np.nextafter(1e3, 0), np.nextafter(1e-1, 1)]])
    gs, ga = t.debug_xs(es)
    assert t.xs_rows() & 4                      # the union grid was built
    t.close()
    for e, a, b in zip(es, gs, ga):        # each table clamps the energy into its own range
        assert a == orc.xs_lookup(ks, vs, min(max(e, ks[0]), ks[-1]))
        assert b == orc.xs_lookup(kc, vc, min(max(e, kc[0]), kc[-1]))


@pytest.mark.parametrize("cfgname", ["tiny_csp", "csp", "split"])
def test_inject_matches_oracle(nt, orc, cfgname):
    cfg = wl.CONFIGS[cfgname].with_(n_particles=5000)
    t = nt.setup(cfg)
    g = t.read_particles()
    t.close()
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    o = orc.inject(prob, 0, cfg.n_particles)
    for f in ["x", "y", "e", "w"]:
        assert np.array_equal(g[f], getattr(o, f)), f
    for f in ["cx", "cy", "ctr", "status", "nfac", "ncol", "ncen"]:
        assert np.array_equal(g[f], getattr(o, f)), f
    for f in ["ox", "oy", "mfp"]:          # libdevice vs libm: <= 2 ulp
        a, b = g[f], getattr(o, f)
        assert np.all(np.abs(a - b) <= 2 * np.spacing(np.abs(b)) + 1e-300), f


# ---------------------------------------------------------------------------------------------
TINY = ["tiny_csp", "tiny_stream", "tiny_split", "tiny_vacuum", "tiny_vacuum_lo", "tiny_scatter_1g",
        "tiny_wkill", "tiny_A12", "tiny_mid", "tiny_thin", "tiny_absorber", "small_csp", "small_scatter",
        "tiny_levels", "small_random", "tiny_mosaic", "small_mosaic", "tiny_hotspot",
        # physics variants (R30-R32)
        "tiny_vacuum_bc", "tiny_mid_bc", "tiny_analog", "tiny_analog_mid", "tiny_roulette",
        "small_csp_variants"]


@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("cfgname", TINY)
def test_parity_deterministic(nt, orc, cfgname, mode):
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=True, mode=mode)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    rep = compare_tally(gt, ot)
    compare_stats(gs, os_)
    assert gs["status"] == 0
    print(cfgname, mode, rep)


@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("layout", [0, 1])
@pytest.mark.parametrize("density_format", [0, 1, 2])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "tiny_split", "tiny_mid", "small_scatter", "tiny_levels",
                                     "tiny_mosaic", "tiny_analog_mid", "tiny_roulette"])
def test_parity_production_atomic(nt, orc, cfgname, mode, density_format, layout):
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=False, mode=mode, density_format=density_format,
                             layout=layout)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)                  # per-particle results do not depend on the tally
    compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
    compare_stats(gs, os_, rtol=1e-9)


@pytest.mark.parametrize("fused", [1, 2])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "small_csp", "small_scatter", "tiny_split", "tiny_mosaic",
                                     "tiny_mid", "tiny_hotspot"])
def test_parity_fused_phases(nt, orc, cfgname, fused):
    """fused_consumers k: one launch in which k CTAs per SM resume the parked collisions
    while the others run phase 1 (hand-over through a published queue): same per-particle
    results, tally within the production bar, every particle tracked once."""
    cfg = wl.CONFIGS[cfgname]
    for defer_below in (8, 33):                     # 33: every collision is parked
        gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=False, fused_consumers=fused,
                                 defer_below=defer_below)
        ot, op, (os_,) = orc.run(cfg)
        compare_particles(gp, op)
        compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
        compare_stats(gs, os_, rtol=1e-9)
        assert np.all(gp["status"] <= 1)


@pytest.mark.parametrize("resume_prefetch", [0, 1])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "small_csp", "small_scatter", "tiny_split", "tiny_mosaic",
                                     "tiny_mid", "tiny_hotspot"])
def test_parity_resume_prefetch(nt, orc, cfgname, resume_prefetch):
    """Production history mode with parked particles as queue-ordered records streamed by a
    cp.async ring (1) or the particle store + index queue (0): same per-particle results,
    tally within the production bar, every parked particle resumed once (batches of 12
    records, ragged last batch; defer_below 33 parks every collision)."""
    cfg = wl.CONFIGS[cfgname]
    for defer_below in (8, 33):
        gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=False, resume_prefetch=resume_prefetch,
                                 defer_below=defer_below)
        ot, op, (os_,) = orc.run(cfg)
        compare_particles(gp, op)
        compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
        compare_stats(gs, os_, rtol=1e-9)
        assert np.all(gp["status"] <= 1)


@pytest.mark.parametrize("cfgname", ["tiny_csp", "small_csp", "small_scatter", "tiny_split", "tiny_mosaic"])
def test_parity_aos_particle_layout(nt, orc, cfgname):
    """particle_layout 1 (AoS records while the history kernel runs): same
    per-particle results, tally within the production bar."""
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=False, particle_layout=1)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
    compare_stats(gs, os_, rtol=1e-9)


def hot_window(cfg, margin=2, cells=2048):
    """The cells around the source rectangle (tally_mode 3's privatised window)."""
    sx, sy, sw, sh = cfg.source
    x0 = max(0, int(sx / cfg.width * cfg.nx) - margin)
    y0 = max(0, int(sy / cfg.height * cfg.ny) - margin)
    nx = min(cfg.nx - x0, int(math.ceil(sw / cfg.width * cfg.nx)) + 2 * margin)
    ny = min(cfg.ny - y0, max(1, min(int(math.ceil(sh / cfg.height * cfg.ny)) + 2 * margin, cells // max(nx, 1))))
    return (x0, y0, max(1, min(nx, cells)), ny)


@pytest.mark.parametrize("tally_mode", [1, 2, 3])
@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("cfgname", ["tiny_hotspot", "tiny_scatter_1g", "tiny_mosaic", "tiny_csp"])
def test_parity_tally_modes(nt, orc, cfgname, mode, tally_mode):
    """Production tally ablations (history mode; event mode uses one RED per flush):
    1 same-cell flushes of a warp summed with shuffles, one atomic per cell; 2 fp64 add by
    compare-and-swap; 3 shared-memory privatised hot window."""
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=False, mode=mode, tally_mode=tally_mode,
                             hot_window=hot_window(cfg))
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
    compare_stats(gs, os_, rtol=1e-9)


@pytest.mark.parametrize("defer_below", [1, 4, 33])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "tiny_split", "tiny_mid", "small_csp", "tiny_mosaic"])
def test_parity_collision_deferral(nt, orc, cfgname, defer_below):
    """History mode with collision deferral off (1), at 4, and parking every collision (33):
    per-particle results and the deterministic tally are unchanged."""
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=True, defer_below=defer_below)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    compare_tally(gt, ot)
    compare_stats(gs, os_)
    assert np.all(gp["status"] <= 1)


@pytest.mark.parametrize("xs_search", [1, 2, 3, 4])
@pytest.mark.parametrize("cfgname", ["small_scatter", "small_csp", "tiny_split", "small_mosaic", "tiny_A12"])
def test_parity_xs_search_strategies(nt, orc, cfgname, xs_search):
    """Plain binary search (1), the paper's cached-index linear walk (2) and the
    bucket index alone (3) give the same bins as the default direct bucket rows, hence the
    oracle's results."""
    cfg = wl.CONFIGS[cfgname]
    gt, gp, (gs,) = _gpu_run(nt, cfg, deterministic=True, xs_search=xs_search)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    compare_tally(gt, ot)
    compare_stats(gs, os_)


@pytest.mark.parametrize("mode", MODES)
def test_parity_two_steps_and_shard(nt, orc, mode):
    cfg = wl.CONFIGS["tiny_split"]
    lo, n = 317, 1203                          # ragged shard of the id space
    gt, gp, gs = _gpu_run(nt, cfg, steps=2, first_id=lo, n_local=n, deterministic=True, mode=mode)
    ot, op, os_ = orc.run(cfg, first_id=lo, n_local=n, steps=2)
    compare_particles(gp, op)
    compare_tally(gt, ot)
    for a, b in zip(gs, os_):
        compare_stats(a, b)
    assert gs[1]["n_alive_start"] == gs[0]["n_census"]


def test_checkpoint_resume_bit_exact(nt):
    """Census is a restart point; counter-based RNG makes resume exact."""
    cfg = wl.CONFIGS["tiny_mid"]
    t = nt.setup(cfg, deterministic=True)
    t.run_timestep(cfg.dt)
    snap = t.read_particles()
    t.run_timestep(cfg.dt)
    want = t.read_particles()
    want_tally = t.read_tally()
    t.write_particles(0, snap)
    t.run_timestep(cfg.dt)
    got = t.read_particles()
    for k in want:
        assert np.array_equal(want[k], got[k]), k
    assert np.array_equal(want_tally, t.read_tally())
    t.close()


def test_edge_cases(nt, orc):
    # empty particle set
    cfg = wl.CONFIGS["tiny_csp"]
    t = nt.setup(cfg, n_local=0, first_id=0)
    s = t.run_timestep(cfg.dt)
    assert s["events"] == 0 and s["status"] == 0
    assert np.all(t.read_tally() == 0)
    t.close()
    # 1 x 1 mesh: every facet is a reflection
    c1 = wl.CONFIGS["tiny_stream"].with_(nx=1, ny=1, n_particles=300, source=(0.0, 0.0, 1.0, 1.0))
    gt, gp, (gs,) = _gpu_run(nt, c1, deterministic=True)
    ot, op, (os_,) = orc.run(c1)
    compare_particles(gp, op)
    compare_stats(gs, os_)
    # non-square mesh, non-unit extents
    c2 = wl.CONFIGS["tiny_mid"].with_(nx=37, ny=91, width=2.5, height=0.7, source=(1.0, 0.1, 0.5, 0.3),
                                       n_particles=999)
    gt, gp, (gs,) = _gpu_run(nt, c2, deterministic=True)
    ot, op, (os_,) = orc.run(c2)
    compare_particles(gp, op)
    compare_tally(gt, ot)
    # event cap
    c3 = wl.CONFIGS["tiny_stream"]
    gt, gp, (gs,) = _gpu_run(nt, c3, deterministic=True, max_events=50)
    prob = orc.Problem(c3, wl.density(c3), wl.tables(c3), max_events=50)
    op = orc.inject(prob, 0, c3.n_particles)
    ot = np.zeros((c3.ny, c3.nx))
    os_ = orc.step(prob, op, 0, ot)
    assert gs["status"] == 8 and gs["n_event_cap"] == os_["n_event_cap"] > 0
    compare_particles(gp, op)
    compare_tally(gt, ot)
    # energy above the table: counted and clamped (NT_ERR_XS_RANGE)
    c4 = wl.CONFIGS["tiny_scatter_1g"].with_(e0=5e7, n_particles=200)
    gt, gp, (gs,) = _gpu_run(nt, c4, deterministic=True)
    ot, op, (os_,) = orc.run(c4)
    assert gs["status"] == 6 and gs["n_xs_range"] == os_["n_xs_range"] > 0
    compare_particles(gp, op)


def test_api_errors(nt):
    t = nt.Tracker()
    with pytest.raises(nt.NeutralError) as e:
        t.run_timestep(1e-7)
    assert e.value.status == 2
    with pytest.raises(nt.NeutralError) as e:
        t.init_mesh(0, 4, 1.0, 1.0, np.ones(4))
    assert e.value.status == 1
    with pytest.raises(nt.NeutralError):
        t.init_mesh(2, 2, 1.0, 1.0, np.array([1.0, -1.0, 0.0, 0.0]))
    t.init_mesh(2, 2, 1.0, 1.0, np.ones(4))
    with pytest.raises(nt.NeutralError):
        t.load_cross_sections([1.0, 1.0], [1.0, 1.0], [1.0, 2.0], [1.0, 1.0])   # not increasing
    t.load_cross_sections([1.0, 2.0], [1.0, 1.0], [1.0, 2.0], [1.0, 1.0])
    with pytest.raises(nt.NeutralError):
        t.inject_particles(10, 5, 6, (0, 0, 0.5, 0.5), 1.5, 1)                    # past n_total
    with pytest.raises(nt.NeutralError):
        t.inject_particles(10, 0, 10, (0.8, 0, 0.5, 0.5), 1.5, 1)                 # outside mesh
    t.inject_particles(10, 0, 10, (0, 0, 0.5, 0.5), 1.5, 1)
    with pytest.raises(nt.NeutralError):
        t.run_timestep(-1.0)
    t.close()


def test_device_pointer_inputs_and_outputs(nt, orc):
    import torch
    cfg = wl.CONFIGS["tiny_csp"]
    dens = torch.as_tensor(wl.density(cfg), device="cuda")
    tabs = [torch.as_tensor(a, device="cuda") for a in wl.tables(cfg)]
    t = nt.Tracker(deterministic=True)
    t.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, dens)
    t.load_cross_sections(*tabs)
    t.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed)
    t.run_timestep(cfg.dt)
    out = torch.empty((cfg.ny, cfg.nx), dtype=torch.float64, device="cuda")
    t.read_tally(out)
    ot, _, _ = orc.run(cfg)
    compare_tally(out.cpu().numpy(), ot)
    t.close()


# ---------------------------------------------------------------------------------------------
# Full BASELINE.json sizes, production launch configuration (what bench.py times).
SCALE = ["csp", "stream", "scatter", "split"]


def _sample_ids(n, k=48):
    ids = np.unique(np.concatenate([np.arange(8), np.linspace(0, n - 1, k).astype(np.int64), [n - 1]]))
    return ids


@pytest.mark.parametrize("mode", MODES)
@pytest.mark.parametrize("cfgname", SCALE)
def test_scale_sampled_parity_and_properties(nt, orc, cfgname, mode):
    cfg = wl.CONFIGS[cfgname]
    t = nt.setup(cfg, mode=mode)      # bench.py's launch configuration (defaults)
    s = t.run_timestep(cfg.dt)
    tally = t.read_tally()
    g = t.read_particles()
    t.close()
    assert s["status"] == 0
    n = cfg.n_particles
    # properties at any size
    assert s["n_alive_start"] == n and s["n_census"] + s["n_killed"] == n          # P5
    assert s["n_facets"] == int(g["nfac"].astype(np.int64).sum())
    assert s["n_collisions"] == int(g["ncol"].astype(np.int64).sum())
    assert np.array_equal(g["ctr"].astype(np.int64), 2 + g["ncol"].astype(np.int64))
    tot = tally.sum()
    assert abs(tot - s["tally_total"]) <= 1e-9 * abs(tot)
    assert abs(tot - g["dep"].sum()) <= 1e-9 * abs(tot)
    r = g["dep"] + g["w"] * g["e"] - cfg.e0                                       # P10
    assert abs(r.mean()) < 5 * r.std() / math.sqrt(n) + 1e-9 * cfg.e0
    wl_ = s["census_weight"] + s["killed_weight"] + s["absorbed_weight"]
    assert abs(wl_ - n) <= 1e-9 * n
    # sampled per-particle parity: the oracle recomputes these ids one by one
    prob = orc.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    ids = _sample_ids(n)
    for pid in ids:
        op = orc.inject(prob, int(pid), 1)
        orc.step(prob, op, int(pid), np.zeros(cfg.nx * cfg.ny))
        gp = {k: v[pid:pid + 1] for k, v in g.items()}
        compare_particles(gp, op)


@pytest.mark.parametrize("mode", MODES)
def test_scale_deterministic_subrange(nt, orc, mode):
    """Paper-size mesh, id subrange [0, K): the deterministic tally equals the oracle's."""
    cfg = wl.CONFIGS["csp"]
    K = 6000
    gt, gp, (gs,) = _gpu_run(nt, cfg, n_local=K, deterministic=True, mode=mode)
    ot, op, (os_,) = orc.run(cfg, n_local=K)
    compare_particles(gp, op)
    rep = compare_tally(gt, ot)
    compare_stats(gs, os_)
    print(rep)


@pytest.mark.parametrize("mode", MODES)
def test_nccl_allreduce_path_single_rank(nt, orc, mode):
    """The NCCL tally/stats allreduce path (nranks > 1 in production), on a 1-rank
    communicator: the reduced tally equals the local tally and the oracle's."""
    cfg = wl.CONFIGS["tiny_csp"]
    uid = nt.get_unique_id()
    t = nt.setup(cfg, mode=mode, deterministic=True, rank=0, nranks=1, unique_id=uid)
    s = t.run_timestep(cfg.dt)
    red = t.read_tally(reduced=True)
    loc = t.read_tally(reduced=False)
    t.close()
    ot, _, (os_,) = orc.run(cfg)
    assert np.array_equal(red, loc)
    compare_tally(red, ot)
    compare_stats(s, os_)
    assert s["reduce_ms"] > 0.0


# ---------------------------------------------------------------------------------------------
# x-slab decomposition: several contexts on this GPU, one per slab,
# exchanging emigrants through the caller-driven nt_slab_* calls.
def _run_slabs(nt, cfg, nslabs, **opts):
    ranks = []
    for r in range(nslabs):
        lo, n = wl.shard(cfg.n_particles, r, nslabs)
        ranks.append(nt.setup(cfg, first_id=lo, n_local=n, rank=r, nranks=nslabs, decomposition=1,
                              **opts))
    for t in ranks:
        t.slab_begin(cfg.dt)
    rounds = 0
    while True:
        outs = [t.slab_round() for t in ranks]
        rounds += 1
        if sum(outs) == 0:
            break
        exp = [t.slab_export(n) for t, n in zip(ranks, outs)]
        for r, (recs, nl, nr) in enumerate(exp):
            assert nl == 0 or r > 0, "emigrant left of slab 0"
            assert nr == 0 or r < nslabs - 1, "emigrant right of the last slab"
            if nl:
                ranks[r - 1].slab_import(recs[:nl])
            if nr:
                ranks[r + 1].slab_import(recs[nl:])
    stats = [t.slab_end() for t in ranks]
    tally = sum(t.read_tally(reduced=False) for t in ranks)
    parts = [t.read_particles() for t in ranks]
    for t in ranks:
        t.close()
    # gather the particles by global id (slots of emigrants keep status 4)
    n = cfg.n_particles
    out = {k: np.zeros(n, dtype=v.dtype) for k, v in parts[0].items()}
    seen = np.zeros(n, dtype=np.int64)
    for p in parts:
        keep = p["status"] <= 1
        g = p["gid"][keep]
        seen[g] += 1
        for k in out:
            out[k][g] = p[k][keep]
    assert np.all(seen == 1), "every particle ends on exactly one slab"
    tot = {k: sum(s[k] for s in stats) for k in stats[0] if k not in ("status",)}
    return tally, out, tot, rounds


@pytest.mark.parametrize("nslabs", [2, 3])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "tiny_stream", "tiny_split", "tiny_mid_bc", "small_csp"])
def test_slab_decomposition_matches_oracle(nt, orc, cfgname, nslabs):
    cfg = wl.CONFIGS[cfgname]
    gt, gp, gs, rounds = _run_slabs(nt, cfg, nslabs)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)                  # per-particle results: identical to replicated
    compare_tally(gt, ot, rtol=1e-6, floor=1e-12)
    compare_stats(gs, os_, rtol=1e-9)
    assert rounds >= 2 if cfg.density != "uniform_hi" else True


def test_slab_storage_scales_with_ranks(nt, orc):
    """x-slab ranks store only their columns plus a one-column halo (§IX: a
    decomposition is what lets a mesh exceed one node's memory): the mesh bytes of a
    4-slab rank are about a quarter of the replicated context's, and the slabs' tallies
    still add up to the oracle's."""
    cfg = wl.CONFIGS["tiny_csp"].with_(nx=1024, ny=1024, n_particles=2000, name="slab_mem")
    rep = nt.setup(cfg)
    full = rep.mesh_bytes()
    rep.close()
    ranks = [nt.setup(cfg, first_id=lo, n_local=n, rank=r, nranks=4, decomposition=1)
             for r, (lo, n) in enumerate(wl.shard(cfg.n_particles, r, 4) for r in range(4))]
    for t in ranks:
        assert t.mesh_bytes() <= 0.27 * full, (t.mesh_bytes(), full)
    for t in ranks:
        t.close()
    gt, gp, gs, rounds = _run_slabs(nt, cfg, 4)
    ot, op, (os_,) = orc.run(cfg)
    compare_particles(gp, op)
    compare_tally(gt, ot, rtol=1e-6, floor=1e-12)


@pytest.mark.parametrize("mode", ["history", "event"])
@pytest.mark.parametrize("cap", [1, 255, 256, 257, 300, 600])
@pytest.mark.parametrize("det", [True, False])
def test_event_cap_across_vote_rounds(nt, orc, mode, cap, det):
    """The event cap (R27) at, below and above the history kernel's 256-event bound between
    warp votes: the bound that ends a lane's round also enforces the cap."""
    c = wl.CONFIGS["tiny_stream"].with_(nx=256, ny=256, n_particles=400)   # ~450 facets each
    gt, gp, (gs,) = _gpu_run(nt, c, deterministic=det, mode=mode, max_events=cap)
    prob = orc.Problem(c, wl.density(c), wl.tables(c), max_events=cap)
    op = orc.inject(prob, 0, c.n_particles)
    ot = np.zeros((c.ny, c.nx))
    os_ = orc.step(prob, op, 0, ot)
    assert os_["n_event_cap"] > 0 if cap < 400 else True
    assert gs["n_event_cap"] == os_["n_event_cap"]
    compare_particles(gp, op)
    compare_stats(gs, os_)
    compare_tally(gt, ot, rtol=1e-9 if det else 1e-6, floor=1e-9 if det else 1e-12)
