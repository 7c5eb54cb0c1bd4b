#!/usr/bin/env python
"""Benchmark: particle events/s per timestep of the B200 neutral tracker (BASELINE.json metric).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config csp] [--mode history]
    python -m torch.distributed.run --nproc-per-node N --master-addr 127.0.0.1 bench.py --gpus N
    python bench.py --impl reference ...      # the oracle on the host cores (reference arm)

A step is one pass of the whole hot path over one batch of synthetic input:
nt_inject_particles + nt_run_timestep (tally zero, tracking kernel, statistics, and the NCCL
tally allreduce when N > 1).  Inputs (mesh, tables) are resident in HBM; the working set
(128 MB density + 128 MB tally + particle store) exceeds the 126 MB L2, so no explicit L2
flush is needed.  Weak scaling: every rank tracks the config's full particle count with
its own global id range.  Rank 0 prints one JSON line.
"""
from __future__ import annotations

import argparse
import json
import math
import os
import statistics
import subprocess
import sys
import time
from pathlib import Path

import numpy as np

ROOT = Path(__file__).resolve().parent
sys.path.insert(0, str(ROOT))

from paper_conf_cluster_martineaum17_b200 import workloads as wl  # noqa: E402

METRIC = "particle events/sec per timestep at 1/2/4/8 B200; % of HBM roofline"
UNIT = "events/s"

# Algorithmic HBM bytes of the method: a facet reads the
# entered cell's density (8 B) and read-modify-writes the exited cell's tally (16 B); a
# census or kill flush is one tally RMW (16 B); every particle's state (x, y, ωx, ωy, E, w,
# n_mfp, cx, cy, ctr, status = 69 B) is read and written once per step.
B_FACET, B_FLUSH, B_PARTICLE = 24, 16, 138


def algorithmic_bytes(s: dict) -> int:
    return (B_FACET * s["n_facets"] + B_FLUSH * (s["n_census"] + s["n_killed"])
            + B_PARTICLE * s["n_alive_start"])


def measured_peaks() -> dict:
    p = ROOT / "MEASURED_PEAKS.json"
    if p.exists():
        d = json.loads(p.read_text())
        return {"hbm_gbs": d["hbm_gbs"], "source": "measured (MEASURED_PEAKS.json)"}
    return {"hbm_gbs": 6650.0, "source": "fallback (B200_PROFILING.md)"}


def l2_red_peak():
    """Scattered fp64 RED throughput of the L2 (REDs/s), measured by scripts/dev/red_microbench.cu
    on a B200 (profiles/r01_v16_red_microbench.json): the best L2-resident footprint."""
    p = ROOT / "profiles" / "r01_v16_red_microbench.json"
    if not p.exists():
        return None
    d = json.loads(p.read_text())
    return max(r["reds_per_s"] for r in d["results"] if r["footprint_MB"] < 100)


def ncu_traffic(config: str, mode: str):
    """Per-launch DRAM bytes of the tracking kernel from a committed ncu --set full capture."""
    p = ROOT / "profiles" / "ncu_traffic.json"
    if not p.exists():
        return None
    d = json.loads(p.read_text())
    return d.get(f"{config}/{mode}")


def ncu_inst(config: str, mode: str):
    """Warp instructions of the tracking kernel(s) per step from a committed ncu capture."""
    p = ROOT / "profiles" / "ncu_inst.json"
    if not p.exists():
        return None
    return json.loads(p.read_text()).get(f"{config}/{mode}")


def issue_roofline(config: str, mode: str, kernel_ms: float, sm_mhz: float, sms: int):
    """Instruction-issue bound: warp instructions per step (ncu, same workload) over the
    kernel's live time, against 4 warp schedulers x 1 instruction per clock per SM at the
    measured SM clock -- the ceiling of a collision-dominated (ALU) kernel."""
    inst = ncu_inst(config, mode)
    if not inst or not kernel_ms or not sm_mhz:
        return None
    achieved = inst / (kernel_ms / 1e3)
    peak = sms * 4 * sm_mhz * 1e6
    return {"bound": "alu", "achieved": achieved, "peak": peak, "unit": "warp inst/s", "frac": achieved / peak,
            "inst_per_step": inst, "peak_source": f"{sms} SMs x 4 schedulers x {sm_mhz:.0f} MHz (measured clock)",
            "inst_source": "smsp__inst_executed.sum, profiles/ncu_inst.json"}


# ---- clocks sampled during the timed region ------------------------------------------------
class ClockSampler:
    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu_index: int):
        self.idx = gpu_index
        self.proc = None

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(
                ["nvidia-smi", f"--query-gpu={self.FIELDS}", "--format=csv,noheader,nounits",
                 "-i", str(self.idx), "-lms", "200"],
                stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
        except Exception:
            self.proc = None
        time.sleep(0.3)
        return self

    def __exit__(self, *a):
        self.out = ""
        if self.proc:
            time.sleep(0.25)
            self.proc.terminate()
            try:
                self.out, _ = self.proc.communicate(timeout=5)
            except Exception:
                self.proc.kill()

    def summary(self) -> dict:
        rows = []
        for line in (getattr(self, "out", "") or "").splitlines():
            f = [x.strip() for x in line.split(",")]
            if len(f) < 9:
                continue
            try:
                rows.append((float(f[1]), float(f[2]), f[5:9]))
            except ValueError:
                continue
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unavailable"], "samples": 0}
        smax = max(r[1] for r in rows)
        loaded = [r for r in rows if r[0] > 0.5 * smax] or rows
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in loaded for i, v in enumerate(r[2]) if v.lower() == "active"})
        return {"sm_mhz": statistics.median(r[0] for r in loaded), "sm_max_mhz": smax,
                "reasons": reasons, "samples": len(rows)}


# ---- the oracle on the host cores (cpu_baseline leg and --impl reference) ----------------------
_ORC_STATE = {}


def _oracle_worker(args):
    lo, n = args
    import oracle
    prob = _ORC_STATE["prob"]
    t0 = time.perf_counter()
    p = oracle.inject(prob, lo, n)
    tally = np.zeros(prob.cfg.nx * prob.cfg.ny)
    st = oracle.step(prob, p, lo, tally)
    dt = time.perf_counter() - t0
    return st["n_facets"] + st["n_collisions"] + st["n_census"], dt


def oracle_host_rate(cfg, budget_s: float = 12.0, max_procs: int | None = None) -> dict:
    """Events/s of the unmodified oracle on the host's cores: one process per core, each on
    a disjoint id range of the workload (ids are iid, so events/s is intensive)."""
    import multiprocessing as mp

    import oracle
    oracle.build()
    prob = oracle.Problem(cfg, wl.density(cfg), wl.tables(cfg))
    _ORC_STATE["prob"] = prob
    cores = len(os.sched_getaffinity(0)) if hasattr(os, "sched_getaffinity") else os.cpu_count()
    procs = max(1, min(cores, max_procs or cores))
    # calibrate on one core
    ev, dt = _oracle_worker((0, 64))
    per_particle = max(dt / 64, 1e-7)
    n_per = max(1, int(budget_s / per_particle))
    n_per = min(n_per, max(1, cfg.n_particles // procs))
    ranges = [(r * n_per, n_per) for r in range(procs)]
    ctx = mp.get_context("fork")
    t0 = time.perf_counter()
    with ctx.Pool(procs) as pool:
        res = pool.map(_oracle_worker, ranges)
    wall = time.perf_counter() - t0
    events = sum(r[0] for r in res)
    slowest = max(r[1] for r in res)
    return {"value": events / slowest, "unit": UNIT, "cores": procs, "kind": "oracle",
            "sample": f"{cfg.name}: ids [0, {procs * n_per}) as {procs} processes x {n_per} particles "
                      f"(1 step each, {events} events, slowest process {slowest:.2f} s, wall {wall:.2f} s)"}


# ---- main --------------------------------------------------------------------------------------
def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--config", default="csp", choices=sorted(wl.CONFIGS))
    ap.add_argument("--mode", default="history", choices=["history", "event"])
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--ctas-per-sm", type=int, default=0)
    ap.add_argument("--refill-min", type=int, default=0)
    ap.add_argument("--layout", type=int, default=0, help="0 tiled 4x4 (default), 1 row-major")
    ap.add_argument("--density-format", type=int, default=0,
                    help="0 u8/u16 codes + block map (default), 1 f64 map, 2 codes without block map")
    ap.add_argument("--tally-mode", type=int, default=0,
                    help="0 one RED per flush, 1 warp-aggregated, 2 CAS-emulated fp64 add, "
                         "3 shared-memory hot window around the source")
    ap.add_argument("--defer-below", type=int, default=0,
                    help="collision deferral threshold (0 default 8, 1 off, 33 park every collision)")
    ap.add_argument("--xs-search", type=int, default=0,
                    help="0 unionised grid (one index and one 96 B row for both tables) + direct rows, "
                         "1 plain binary search, 2 cached-bin linear walk, 3 bucket index alone (two "
                         "dependent loads), 4 direct bucket rows per table (one dependent load per lookup)")
    ap.add_argument("--resume-prefetch", type=int, default=-1,
                    help="history mode: 1 parked records + cp.async resume ring, 0 particle store + "
                         "index queue, -1 the library default")
    ap.add_argument("--xs-l2-persist", type=int, default=0,
                    help="1: L2 persisting access-policy window over the XS tables while tracking")
    ap.add_argument("--table-size", type=int, default=0,
                    help="experiment: scatter table keys (capture = 3/4 of it); 0 = the config's")
    ap.add_argument("--fused-consumers", type=int, default=0,
                    help="history mode: fuse the parking phases (k > 0: k-1 dedicated consumer CTAs per SM, "
                         "the other warps resume parked particles once the range is exhausted; 0: two launches)")
    ap.add_argument("--particle-layout", type=int, default=0,
                    help="0 structure of arrays (default), 1 AoS records while tracking (ablation)")
    ap.add_argument("--json-out", default=None)
    ap.add_argument("--no-extras", action="store_true",
                    help="skip the short runs of the other configs / modes added to the JSON line")
    ap.add_argument("--mesh", type=int, default=0, help="experiment: override nx = ny")
    ap.add_argument("--particles", type=int, default=0, help="experiment: override the particle count")
    return ap.parse_args()


def hot_window(cfg, margin=2, cells=2048):
    """tally_mode 3's privatised window: the cells around the source rectangle (<= 2048)."""
    sx, sy, sw, sh = cfg.source
    x0 = max(0, int(sx / cfg.width * cfg.nx) - margin)
    y0 = max(0, int(sy / cfg.height * cfg.ny) - margin)
    nx = max(1, min(cfg.nx - x0, int(math.ceil(sw / cfg.width * cfg.nx)) + 2 * margin, cells))
    ny = max(1, min(cfg.ny - y0, int(math.ceil(sh / cfg.height * cfg.ny)) + 2 * margin, cells // nx))
    return (x0, y0, nx, ny)


def dist_env():
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return rank, world, local


def emit(d: dict, path: str | None):
    line = json.dumps(d)
    print(line, flush=True)
    if path:
        Path(path).parent.mkdir(parents=True, exist_ok=True)
        Path(path).write_text(line + "\n")


def run_reference(a):
    rank, world, _ = dist_env()
    if rank != 0:
        return
    cfg = wl.CONFIGS[a.config]
    n_gpus = max(a.gpus, world)
    budget = max(3.0, min(20.0, 120.0 / max(1, a.steps + a.warmup)))
    vals = []
    last = None
    for k in range(a.warmup + a.steps):
        r = oracle_host_rate(cfg, budget_s=budget)
        if k >= a.warmup:
            vals.append(r["value"])
            last = r
    v = statistics.median(vals)
    cpu = dict(last)
    cpu["value"] = v
    emit({"impl": "reference", "metric": METRIC, "value": v, "unit": UNIT, "n_gpus": n_gpus,
          "steps": a.steps, "warmup": a.warmup, "ms_per_step": None, "higher_is_better": True,
          "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
          "config": {"workload": cfg.name, "mode": "oracle (Listing 1, single-threaded per process)",
                     "nx": cfg.nx, "ny": cfg.ny, "particles_per_gpu": cfg.n_particles},
          "cpu_baseline": cpu,
          "e2e": {"value": v, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}},
         a.json_out)


# Short runs of the other BASELINE.json workloads and variants, reported next to the headline
# in the same JSON line (extra keys; the headline value stays csp / history mode).
EXTRAS = [
    ("stream", "history", {}), ("scatter", "history", {}), ("split", "history", {}),
    ("csp", "event", {}), ("stream", "event", {}), ("scatter", "event", {}), ("split", "event", {}),
    ("csp", "history", {"density_format": 1}),
]


def measure_extra(binding, torch, cfgname, mode, opts, local, steps=3, warmup=2):
    cfg = wl.CONFIGS[cfgname]
    stream = torch.cuda.current_stream()
    tr = binding.Tracker(device=local, stream=stream.cuda_stream, mode=mode, A=cfg.A,
                         molar_mass=cfg.molar_mass, e_min=cfg.e_min, w_min=cfg.w_min, **opts)
    tr.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, wl.density(cfg))
    tr.load_cross_sections(*wl.tables(cfg))

    def step():
        tr.inject_particles(cfg.n_particles, 0, cfg.n_particles, cfg.source, cfg.e0, cfg.seed)
        return tr.run_timestep(cfg.dt)

    for _ in range(warmup):
        step()
    torch.cuda.synchronize()
    e0 = torch.cuda.Event(enable_timing=True)
    e1 = torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    stats = [step() for _ in range(steps)]
    e1.record(stream)
    torch.cuda.synchronize()
    tr.close()
    ms = e0.elapsed_time(e1) / steps
    events = statistics.mean(s["events"] for s in stats)
    track_ms = statistics.mean(s["track_ms"] for s in stats)
    ab = statistics.mean(algorithmic_bytes(s) for s in stats)
    reds = statistics.mean(s["n_facets"] + s["n_census"] + s["n_killed"] for s in stats)
    red_peak = l2_red_peak()
    return {"workload": cfgname, "mode": mode, "opts": opts, "value": events / (ms / 1e3), "unit": UNIT,
            "ms_per_step": ms, "steps": steps, "warmup": warmup, "events_per_step": events,
            "kernel_ms": track_ms,
            "hbm_roofline_frac": ab / (track_ms / 1e3) / 1e9 / measured_peaks()["hbm_gbs"],
            "l2_red_frac": None if red_peak is None else reds / (track_ms / 1e3) / red_peak,
            "grind_ns_per_event": track_ms * 1e6 / max(1.0, events),
            "status": sorted({s["status"] for s in stats})}


def main():
    a = parse()
    if a.impl == "reference":
        return run_reference(a)
    import torch
    import torch.distributed as dist

    from paper_conf_cluster_martineaum17_b200 import binding

    rank, world, local = dist_env()
    if world > 1 and not dist.is_initialized():
        torch.cuda.set_device(local)
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    torch.cuda.set_device(local)
    cfg = wl.CONFIGS[a.config]
    if a.mesh:
        cfg = cfg.with_(nx=a.mesh, ny=a.mesh, name=f"{cfg.name}@{a.mesh}")
    if a.particles:
        cfg = cfg.with_(n_particles=a.particles, name=f"{cfg.name}@{a.particles}p")
    if a.table_size:
        cfg = cfg.with_(tables=wl.Tables(n_scatter=a.table_size, n_capture=max(2, 3 * a.table_size // 4)),
                        name=f"{cfg.name}@xs{a.table_size}")
    n_per = cfg.n_particles
    n_total = n_per * world
    first_id = rank * n_per
    uid = None
    if world > 1:
        obj = [binding.get_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        uid = obj[0]
    stream = torch.cuda.current_stream()
    tr = binding.Tracker(device=local, stream=stream.cuda_stream, mode=a.mode, rank=rank,
                         nranks=world, unique_id=uid, A=cfg.A, molar_mass=cfg.molar_mass,
                         e_min=cfg.e_min, w_min=cfg.w_min, ctas_per_sm=a.ctas_per_sm,
                         refill_min=a.refill_min, layout=a.layout, density_format=a.density_format,
                         tally_mode=a.tally_mode, defer_below=a.defer_below,
                         xs_search=a.xs_search, hot_window=hot_window(cfg),
                         particle_layout=a.particle_layout, fused_consumers=a.fused_consumers,
                         xs_l2_persist=a.xs_l2_persist,
                         resume_prefetch=None if a.resume_prefetch < 0 else a.resume_prefetch)
    density = wl.density(cfg)
    tables = wl.tables(cfg)
    tr.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, density)
    tr.load_cross_sections(*tables)

    def step():
        tr.inject_particles(n_total, first_id, n_per, cfg.source, cfg.e0, cfg.seed)
        return tr.run_timestep(cfg.dt)

    def barrier():
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()

    for _ in range(a.warmup):
        step()
    barrier()
    vis = os.environ.get("CUDA_VISIBLE_DEVICES", "").split(",")
    gidx = int(vis[local]) if len(vis) > local and vis[local].strip().isdigit() else local
    stats = []
    with ClockSampler(gidx) as clk:
        barrier()
        e0 = torch.cuda.Event(enable_timing=True)
        e1 = torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(a.steps):
            stats.append(step())
        e1.record(stream)
        barrier()
    ms = e0.elapsed_time(e1)
    t = torch.tensor([ms], dtype=torch.float64, device="cuda")
    if world > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    ms = float(t.item())
    # events: the step statistics are already summed over ranks when world > 1
    events = sum(s["events"] for s in stats)
    value = events / (ms / 1e3)
    track_ms = statistics.mean(s["track_ms"] for s in stats)
    ab = statistics.mean(algorithmic_bytes(s) for s in stats) / world   # per rank launch
    peaks = measured_peaks()
    achieved = ab / (track_ms / 1e3) / 1e9
    traffic = ncu_traffic(cfg.name, a.mode)
    # one fp64 tally RED per flush: every facet, census and kill
    reds = statistics.mean(s["n_facets"] + s["n_census"] + s["n_killed"] for s in stats) / world
    red_peak = l2_red_peak()
    red_rate = reds / (track_ms / 1e3)
    status = {s["status"] for s in stats}
    launches = sum(s["n_launches"] + 1 for s in stats)          # + inject kernel per step

    e2e = None
    if not a.no_e2e:
        pin_d = torch.from_numpy(density).pin_memory()
        pin_t = [torch.from_numpy(np.ascontiguousarray(x)).pin_memory() for x in tables]
        out = torch.empty((cfg.ny, cfg.nx), dtype=torch.float64).pin_memory()
        h2d = pin_d.numel() * 8 + sum(x.numel() * 8 for x in pin_t)
        d2h = out.numel() * 8 + 160          # tally + step statistics
        def e2e_step():
            tr.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, pin_d)
            tr.load_cross_sections(*pin_t)
            s = step()
            tr.read_tally(out)
            return s

        for _ in range(min(a.warmup, 1)):          # one untimed e2e step (first-touch of the pinned buffers)
            e2e_step()
        barrier()
        f0 = torch.cuda.Event(enable_timing=True)
        f1 = torch.cuda.Event(enable_timing=True)
        ev_e2e = 0
        f0.record(stream)
        for _ in range(a.steps):
            s = e2e_step()
            ev_e2e += s["events"]
        f1.record(stream)
        barrier()
        ms2 = f0.elapsed_time(f1)
        t2 = torch.tensor([ms2], dtype=torch.float64, device="cuda")
        if world > 1:
            dist.all_reduce(t2, op=dist.ReduceOp.MAX)
        e2e = {"value": ev_e2e / (float(t2.item()) / 1e3), "unit": UNIT, "h2d_bytes_per_step": h2d,
               "d2h_bytes_per_step": d2h, "ms_per_step": float(t2.item()) / a.steps,
               "path": "C ABI with pinned host buffers: init_mesh + load_cross_sections + inject + "
                       "run_timestep + read_tally"}
    tr.close()

    clk_sum = clk.summary()
    sms = torch.cuda.get_device_properties(local).multi_processor_count
    extras = None
    if rank == 0 and world == 1 and not a.no_extras and a.config == "csp" and a.mode == "history":
        extras = {}
        for c, m, o in EXTRAS:
            key = f"{c}/{m}" + "".join(f"/{k}={v}" for k, v in o.items())
            try:
                extras[key] = measure_extra(binding, torch, c, m, o, local)
                if not o:                    # an ncu capture exists for the default options
                    ir = issue_roofline(c, m, extras[key]["kernel_ms"], clk_sum.get("sm_mhz"), sms)
                    if ir:
                        extras[key]["issue_frac"] = ir["frac"]
            except Exception as ex:          # reported, never fatal for the headline
                extras[key] = {"error": str(ex)[:200]}

    cpu = None
    if rank == 0 and world == 1 and not a.no_cpu_baseline:
        cpu = oracle_host_rate(cfg)
        one = oracle_host_rate(cfg, budget_s=8.0, max_procs=1)
        cpu["one_core"] = {"value": one["value"], "cores": 1, "sample": one["sample"]}
        cpu["gpu_over_oracle"] = {"all_cores": value / cpu["value"], "one_core": value / one["value"]}

    if rank == 0:
        s0 = stats[-1]
        emit({
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": a.steps,
            "warmup": a.warmup, "ms_per_step": ms / a.steps, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": cfg.name, "mode": a.mode, "nx": cfg.nx, "ny": cfg.ny,
                       "layout": "tiled4x4" if a.layout == 0 else "row-major",
                       "particle_store": ["SoA", "AoS (ablation)"][a.particle_layout],
                       "phases": (f"fused, {a.fused_consumers - 1} dedicated consumer CTA(s)/SM" if a.fused_consumers
                                  else "two launches (park, resume)"),
                       "density_format": ["codes+block map", "f64", "codes"][a.density_format],
                       "tally": ["fp64 RED per flush", "warp-aggregated fp64 RED", "CAS-emulated fp64 add",
                                 "shared-memory hot window %s + RED" % (hot_window(cfg),)][a.tally_mode],
                       "defer_below": a.defer_below or 8,
                       "xs_search": ["unionised grid + direct rows", "binary", "cached-bin walk",
                                     "bucket index", "direct bucket rows"][a.xs_search],
                       "xs_l2_persist": bool(a.xs_l2_persist),
                       "particles_per_gpu": n_per, "global_particles": n_total, "dt": cfg.dt,
                       "tables": [len(tables[0]), len(tables[2])],
                       "parallelism": f"dp{world} (particle id shards, tally NCCL allreduce)",
                       "l2": "no flush: working set (128 MB density + 128 MB tally + particles) > 126 MB L2",
                       "step": "inject_particles + run_timestep"},
            "events_per_step": events / a.steps,
            "event_mix": {"facets": s0["n_facets"], "collisions": s0["n_collisions"],
                          "census": s0["n_census"], "killed": s0["n_killed"]},
            "status": sorted(status),
            # per-event grind time (the paper's 3 ns/facet on stream, 18 ns/collision on
            # scatter, were measured on a Xeon): tracking time / events this rank
            "grind_ns": {"per_event": track_ms * 1e6 * world / max(1.0, events / a.steps),
                         "per_facet_if_all_facets": track_ms * 1e6 * world / max(1, s0["n_facets"]),
                         "per_collision_if_all_collisions": track_ms * 1e6 * world / max(1, s0["n_collisions"])},
            "roofline": {"bound": "hbm", "basis": "algorithmic bytes of the paper's fp64 format (SURVEY §8(d): "
                         "24 B/facet, 16 B/census or kill flush, 138 B/particle) / tracking-kernel time; the "
                         "kernel reads u8 codes and its tally REDs stay in L2, so this is an algorithmic-byte "
                         "rate, not DRAM utilisation (that is traffic / kernel time, dram_frac); the binding "
                         "ceiling is l2_red_roofline",
                         "dram_frac": None if not traffic else traffic / (track_ms / 1e3) / 1e9 / peaks["hbm_gbs"],
                         "kernel": f"history_kernel<false>" if a.mode == "history" else "ev_loop_kernel",
                         "achieved": achieved, "peak": peaks["hbm_gbs"], "unit": "GB/s",
                         "frac": achieved / peaks["hbm_gbs"], "traffic": traffic,
                         "algorithmic_bytes_per_launch": ab, "kernel_ms": track_ms,
                         "kernel_share_of_step": track_ms / (ms / a.steps),
                         "peak_source": peaks["source"]},
            "l2_red_roofline": None if red_peak is None else {
                "bound": "l2_red", "achieved": red_rate, "peak": red_peak, "unit": "RED/s",
                "frac": red_rate / red_peak, "reds_per_launch": reds,
                "peak_source": "measured: scripts/dev/red_microbench.cu (profiles/r01_v16_red_microbench.json)"},
            "issue_roofline": issue_roofline(cfg.name, a.mode, track_ms, clk_sum.get("sm_mhz"), sms),
            "cpu_baseline": cpu,
            "extra_configs": extras,
            "e2e": e2e,
            "gpu_launches": launches,
            "clocks": clk_sum,
        }, a.json_out)
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
