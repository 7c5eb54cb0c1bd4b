"""GPU runtime tests of the C ABI: allocation-free timesteps, the NCCL step path, input
pointer kinds and stream ordering, and (on a box with >= 2 GPUs) two real ranks.

The per-step cross-rank reduction is the paper's privatised-tally merge at GPU
granularity (§VI-F); the ABI is DESIGN.md §1 / include/neutral_b200.h.
"""
import os

import numpy as np
import pytest

from paper_conf_cluster_martineaum17_b200 import workloads as wl
from tests.parity import compare_particles, compare_stats, compare_tally

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def nt():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cluster_martineaum17_b200 import binding, build
    build.build()
    return binding


@pytest.mark.parametrize("mode", ["history", "event"])
@pytest.mark.parametrize("det", [False, True])
@pytest.mark.parametrize("nccl", [False, True])
def test_timestep_allocates_nothing(nt, mode, det, nccl):
    """After the first step sized the context's buffers, further steps (and re-injections
    of the same particle count) make no device allocation: no cudaMalloc/cudaFree (which
    would synchronise the device) inside nt_run_timestep."""
    cfg = wl.CONFIGS["small_csp"]
    extra = dict(rank=0, nranks=1, unique_id=nt.get_unique_id()) if nccl else {}
    t = nt.setup(cfg, mode=mode, deterministic=det, **extra)
    t.run_timestep(cfg.dt)
    a0 = nt.alloc_count()
    for _ in range(3):
        t.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed)
        s = t.run_timestep(cfg.dt)
        assert s["status"] == 0
    assert nt.alloc_count() == a0
    if nccl:
        assert np.array_equal(t.read_tally(reduced=True), t.read_tally(reduced=False))
    t.close()


def test_tables_and_density_from_pinned_and_cuda_tensors(nt, orc):
    """Host (pageable, pinned) and device inputs give the same result; CUDA tensors made on
    torch's stream are ordered before the library reads them (binding.Tracker._order)."""
    import torch
    cfg = wl.CONFIGS["tiny_mid"]
    dens = wl.density(cfg)
    tabs = wl.tables(cfg)
    ot, op, (os_,) = orc.run(cfg)
    kinds = {
        "numpy": (dens, tabs),
        "pinned": (torch.from_numpy(dens).pin_memory(), [torch.from_numpy(a).pin_memory() for a in tabs]),
        # produced by a kernel on torch's current stream just before the call
        "cuda": (torch.as_tensor(dens, device="cuda") * 1.0, [torch.as_tensor(a, device="cuda") + 0.0 for a in tabs]),
    }
    for k, (d, tb) in kinds.items():
        t = nt.Tracker(deterministic=True)
        t.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, d)
        t.load_cross_sections(*tb)
        t.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed)
        s = t.run_timestep(cfg.dt)
        out = torch.empty((cfg.ny, cfg.nx), dtype=torch.float64, device="cuda") if k == "cuda" else None
        gt = t.read_tally(out)
        gt = gt.cpu().numpy() if k == "cuda" else gt
        compare_particles(t.read_particles(), op)
        compare_tally(gt, ot)
        compare_stats(s, os_)
        t.close()


def test_failed_reload_leaves_no_dangling_stage(nt):
    """A rejected nt_load_cross_sections / nt_inject_particles lowers the stage, so a later
    nt_run_timestep is refused instead of running on replaced buffers."""
    cfg = wl.CONFIGS["tiny_csp"]
    t = nt.setup(cfg)
    t.run_timestep(cfg.dt)
    with pytest.raises(nt.NeutralError):
        t.load_cross_sections([1.0, 1.0], [1.0, 1.0], [1.0, 2.0], [1.0, 1.0])
    with pytest.raises(nt.NeutralError) as e:
        t.run_timestep(cfg.dt)
    assert e.value.status == 2
    t.load_cross_sections(*wl.tables(cfg))
    with pytest.raises(nt.NeutralError):
        t.inject_particles(10, 5, 6, cfg.source, cfg.e0, 1)
    t.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed)
    assert t.run_timestep(cfg.dt)["status"] == 0
    t.close()


# ---------------------------------------------------------------------------------------------
# Two real ranks (one process per GPU, NCCL over NVLink): skipped on a one-GPU box.
def _two_rank_worker(rank, uid, cfgname, decomposition, out_dir):
    import torch
    from paper_conf_cluster_martineaum17_b200 import binding
    torch.cuda.set_device(rank)
    cfg = wl.CONFIGS[cfgname]
    lo, n = wl.shard(cfg.n_particles, rank, 2)
    t = binding.setup(cfg, device=rank, first_id=lo, n_local=n, rank=rank, nranks=2, unique_id=uid,
                      decomposition=decomposition)
    s = t.run_timestep(cfg.dt)
    np.save(os.path.join(out_dir, f"tally_{rank}.npy"), t.read_tally(reduced=True))
    np.save(os.path.join(out_dir, f"local_{rank}.npy"), t.read_tally(reduced=False))
    p = t.read_particles()
    np.savez(os.path.join(out_dir, f"parts_{rank}.npz"), **p)
    np.save(os.path.join(out_dir, f"stats_{rank}.npy"),
            np.array([s["n_alive_start"], s["n_facets"], s["n_collisions"], s["n_census"], s["n_killed"],
                      s["tally_total"]], dtype=np.float64))
    t.close()


@pytest.mark.parametrize("decomposition", [0, 1])
@pytest.mark.parametrize("cfgname", ["tiny_csp", "small_csp"])
def test_two_ranks_nccl(nt, orc, tmp_path, cfgname, decomposition):
    import torch
    import torch.multiprocessing as mp
    if torch.cuda.device_count() < 2:
        pytest.skip("needs 2 GPUs")
    uid = nt.get_unique_id()
    mp.start_processes(_two_rank_worker, args=(uid, cfgname, decomposition, str(tmp_path)), nprocs=2,
                       start_method="spawn")
    cfg = wl.CONFIGS[cfgname]
    ot, op, (os_,) = orc.run(cfg)
    loc = [np.load(tmp_path / f"local_{r}.npy") for r in range(2)]
    for r in range(2):
        compare_tally(np.load(tmp_path / f"tally_{r}.npy"), ot, rtol=1e-6, floor=1e-12)
        s = np.load(tmp_path / f"stats_{r}.npy")
        assert s[0] == os_["n_alive_start"] and s[1] == os_["n_facets"] and s[2] == os_["n_collisions"]
    compare_tally(loc[0] + loc[1], ot, rtol=1e-6, floor=1e-12)
    parts = [dict(np.load(tmp_path / f"parts_{r}.npz")) for r in range(2)]
    n = cfg.n_particles
    out = {k: np.zeros(n, dtype=v.dtype) for k, v in parts[0].items()}
    seen = np.zeros(n, dtype=np.int64)
    for p in parts:
        keep = p["status"] <= 1
        g = p["gid"][keep]
        seen[g] += 1
        for k in out:
            out[k][g] = p[k][keep]
    assert np.all(seen == 1)
    compare_particles(out, op)


@pytest.mark.parametrize("n_distinct", [1, 2, 255, 256, 257, 2047, 2048, 5000, 70000])
def test_density_distinct_values_and_format(nt, n_distinct):
    """nt_init_mesh counts the distinct density values while the upload runs (a hashed set,
    falling back to sorting every cell's bit pattern past 2047 values) and picks the lossless
    u8 (<= 256) / u16 (<= 65536) material codes or the f64 map.  (That the codes
    reproduce the density exactly is covered by the parity tests on tiny_levels, u16, and
    small_random, f64.)"""
    rng = np.random.default_rng(n_distinct)
    nx, ny = 301, 297                            # ragged, several upload chunks
    levels = np.unique(rng.uniform(1e-3, 5.0, n_distinct * 2))[:n_distinct]
    assert len(levels) == n_distinct
    rho = levels[rng.integers(0, n_distinct, nx * ny)]
    rho[:n_distinct] = levels[: min(n_distinct, nx * ny)]   # every level present
    t = nt.Tracker(density_format=0)
    t.init_mesh(nx, ny, 1.0, 1.0, rho)
    fmt, nd = t.density_format()
    t.close()
    want = "u8" if n_distinct <= 256 else ("u16" if n_distinct <= 65536 else "f64")
    assert fmt == want and nd == n_distinct
