"""Thin ctypes binding of the C ABI in include/neutral_b200.h (argument marshalling only).

Every step of the method runs in the CUDA kernels of ``lib/libneutral_b200.so``; this
module only converts numpy arrays / torch tensors to pointers and status codes to
exceptions.  There is no CPU fallback: if the library is missing, loading fails loudly.
"""
from __future__ import annotations

import ctypes as C
import os
from pathlib import Path

import numpy as np

LIB_PATH = Path(__file__).resolve().parent / "lib" / "libneutral_b200.so"
# profiling aid: NT_LIB_VARIANT=name loads lib/variants/libneutral_b200_<name>.so (an A/B build
# of the same sources with different compile-time options, scripts/dev/build_variants.sh)
if os.environ.get("NT_LIB_VARIANT"):
    LIB_PATH = LIB_PATH.parent / "variants" / f"libneutral_b200_{os.environ['NT_LIB_VARIANT']}.so"

NT_OK = 0
STATUS = {0: "NT_OK", 1: "NT_ERR_ARG", 2: "NT_ERR_STATE", 3: "NT_ERR_OOM", 4: "NT_ERR_CUDA",
          5: "NT_ERR_NCCL", 6: "NT_ERR_XS_RANGE", 7: "NT_ERR_NONFINITE",
          8: "NT_ERR_EVENT_CAP", 9: "NT_ERR_UNSUPPORTED"}
STEP_ANOMALIES = {6, 7, 8}     # the step completed; stats are valid
MODES = {"history": 0, "event": 1}

# Every function the header declares (tests check the library exports all of them).
EXPORTS = ["nt_abi_version", "nt_build_info", "nt_status_string", "nt_options_default",
           "nt_get_unique_id", "nt_create", "nt_destroy", "nt_last_error", "nt_init_mesh",
           "nt_load_cross_sections", "nt_inject_particles", "nt_run_timestep", "nt_read_tally",
           "nt_read_particles", "nt_write_particles", "nt_slab_record_bytes", "nt_slab_begin",
           "nt_slab_round", "nt_slab_export", "nt_slab_import", "nt_slab_end", "nt_particle_slots",
           "nt_debug_threefry", "nt_debug_xs", "nt_debug_alloc_count",
           "nt_debug_mesh_bytes", "nt_debug_xs_rows", "nt_debug_density_format"]


class NeutralError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS.get(status, status)}: {msg}")
        self.status = status


class Options(C.Structure):
    _fields_ = [("device", C.c_int32), ("stream", C.c_void_p), ("mode", C.c_int32),
                ("deterministic", C.c_int32), ("rank", C.c_int32), ("nranks", C.c_int32),
                ("nccl_unique_id", C.c_void_p), ("A", C.c_double), ("molar_mass", C.c_double),
                ("e_min", C.c_double), ("w_min", C.c_double),
                ("max_events_per_history", C.c_int64), ("block_size", C.c_int32),
                ("ctas_per_sm", C.c_int32), ("det_batch", C.c_int64),
                ("refill_min", C.c_int32), ("density_format", C.c_int32),
                ("layout", C.c_int32), ("tally_mode", C.c_int32),
                ("defer_below", C.c_int32), ("xs_search", C.c_int32),
                ("boundary", C.c_int32), ("analog_absorption", C.c_int32),
                ("roulette", C.c_int32), ("decomposition", C.c_int32),
                ("roulette_weight", C.c_double), ("hot_x0", C.c_int32), ("hot_y0", C.c_int32),
                ("hot_nx", C.c_int32), ("hot_ny", C.c_int32), ("particle_layout", C.c_int32),
                ("fused_consumers", C.c_int32), ("xs_l2_persist", C.c_int32),
                ("resume_prefetch", C.c_int32)]


class StepStats(C.Structure):
    _fields_ = [("n_alive_start", C.c_uint64), ("n_facets", C.c_uint64),
                ("n_collisions", C.c_uint64), ("n_census", C.c_uint64), ("n_killed", C.c_uint64),
                ("tally_total", C.c_double), ("census_energy", C.c_double),
                ("census_weight", C.c_double), ("killed_energy", C.c_double),
                ("killed_weight", C.c_double), ("absorbed_weight", C.c_double),
                ("n_xs_range", C.c_uint64), ("n_nonfinite", C.c_uint64),
                ("n_event_cap", C.c_uint64), ("track_ms", C.c_float), ("reduce_ms", C.c_float),
                ("step_ms", C.c_float), ("n_launches", C.c_uint32),
                ("n_escaped", C.c_uint64), ("n_absorbed", C.c_uint64),
                ("escaped_energy", C.c_double), ("escaped_weight", C.c_double),
                ("absorbed_energy", C.c_double), ("roulette_gain", C.c_double)]


PARTICLE_FIELDS = [("x", np.float64), ("y", np.float64), ("ox", np.float64), ("oy", np.float64),
                   ("e", np.float64), ("w", np.float64), ("mfp", np.float64), ("cx", np.int32),
                   ("cy", np.int32), ("ctr", np.uint32), ("status", np.uint8),
                   ("nfac", np.uint32), ("ncol", np.uint32), ("ncen", np.uint32),
                   ("dep", np.float64), ("gid", np.int64)]


class ParticlesView(C.Structure):
    _fields_ = [(n, C.c_void_p) for n, _ in PARTICLE_FIELDS]


_lib = None


def lib():
    """Load the CUDA library (fails loudly when it has not been built)."""
    global _lib
    if _lib is None:
        if not LIB_PATH.exists():
            raise ImportError(f"{LIB_PATH} is missing: run `python -m "
                              "paper_conf_cluster_martineaum17_b200.build` (no CPU fallback)")
        L = C.CDLL(str(LIB_PATH))
        vp, i32, i64, u64, d = C.c_void_p, C.c_int32, C.c_int64, C.c_uint64, C.c_double
        sigs = {
            "nt_abi_version": ([], i32),
            "nt_build_info": ([], C.c_char_p),
            "nt_status_string": ([C.c_int], C.c_char_p),
            "nt_options_default": ([C.POINTER(Options)], C.c_int),
            "nt_get_unique_id": ([vp], C.c_int),
            "nt_create": ([C.POINTER(Options), C.POINTER(vp)], C.c_int),
            "nt_destroy": ([vp], C.c_int),
            "nt_last_error": ([vp], C.c_char_p),
            "nt_init_mesh": ([vp, i32, i32, d, d, vp], C.c_int),
            "nt_load_cross_sections": ([vp, vp, vp, i64, vp, vp, i64], C.c_int),
            "nt_inject_particles": ([vp, i64, i64, i64, d, d, d, d, d, u64], C.c_int),
            "nt_run_timestep": ([vp, d, C.POINTER(StepStats)], C.c_int),
            "nt_read_tally": ([vp, vp, i32], C.c_int),
            "nt_read_particles": ([vp, i64, i64, C.POINTER(ParticlesView)], C.c_int),
            "nt_write_particles": ([vp, i64, i64, C.POINTER(ParticlesView)], C.c_int),
            "nt_slab_record_bytes": ([], i64),
            "nt_slab_begin": ([vp, d], C.c_int),
            "nt_slab_round": ([vp, C.POINTER(i64)], C.c_int),
            "nt_slab_export": ([vp, vp, i64, C.POINTER(i64), C.POINTER(i64)], C.c_int),
            "nt_slab_import": ([vp, vp, i64], C.c_int),
            "nt_slab_end": ([vp, C.POINTER(StepStats)], C.c_int),
            "nt_particle_slots": ([vp, C.POINTER(i64)], C.c_int),
            "nt_debug_threefry": ([vp, vp, i64, vp], C.c_int),
            "nt_debug_xs": ([vp, vp, i64, vp, vp], C.c_int),
            "nt_debug_alloc_count": ([], i64),
            "nt_debug_mesh_bytes": ([vp], i64),
            "nt_debug_xs_rows": ([vp], C.c_int32),
            "nt_debug_density_format": ([vp, vp], C.c_int32),
        }
        for name, (args, res) in sigs.items():
            f = getattr(L, name)
            f.argtypes = args
            f.restype = res
        _lib = L
    return _lib


def alloc_count() -> int:
    """Device allocations the library has made so far (process-wide)."""
    return int(lib().nt_debug_alloc_count())


def get_unique_id() -> bytes:
    buf = C.create_string_buffer(128)
    st = lib().nt_get_unique_id(buf)
    if st != NT_OK:
        raise NeutralError(st, "ncclGetUniqueId failed")
    return buf.raw


def _ptr(a):
    """(pointer, keepalive) for a numpy array or torch tensor (host or CUDA)."""
    if a is None:
        return None, None
    if isinstance(a, np.ndarray):
        if not a.flags["C_CONTIGUOUS"]:
            a = np.ascontiguousarray(a)
        return a.ctypes.data, a
    if hasattr(a, "data_ptr"):
        assert a.is_contiguous(), "tensor must be contiguous"
        return a.data_ptr(), a
    raise TypeError(f"unsupported array type {type(a)}")


def _f64(a):
    if isinstance(a, np.ndarray):
        return np.ascontiguousarray(a, dtype=np.float64)
    import torch
    if isinstance(a, torch.Tensor):
        assert a.dtype == torch.float64
        return a.contiguous()
    return np.ascontiguousarray(np.asarray(a, dtype=np.float64))


class Tracker:
    """One nt_ctx: a 2D mesh, two XS tables, this rank's particles, and its tally.

    Streams: the context orders its work on ``stream`` (a cudaStream_t handle, e.g.
    ``torch.cuda.current_stream().cuda_stream``) or, when None, on a stream of its own.
    CUDA tensors passed in or out are produced / consumed on torch's current stream: when
    that is not the context's stream, the binding synchronises torch's current stream
    before handing the pointer over (so a tensor is never read before its producer wrote
    it, nor overwritten while a kernel still reads it); the library synchronises its own
    stream before returning from every call that reads or writes caller memory.
    """

    def __init__(self, device: int = 0, stream=None, mode: str = "history",
                 deterministic: bool = False, rank: int = 0, nranks: int = 1,
                 unique_id: bytes | None = None, A: float = 1.0, molar_mass: float = 1e-3,
                 e_min: float = 1.0, w_min: float = 1e-3, max_events: int = 0,
                 ctas_per_sm: int = 0, det_batch: int = 0, refill_min: int = 0,
                 density_format: int = 0, layout: int = 0, tally_mode: int = 0,
                 defer_below: int = 0, xs_search: int = 0, boundary: int = 0,
                 analog: int = 0, roulette: int = 0, roulette_weight: float = 0.0,
                 decomposition: int = 0, hot_window=(0, 0, 0, 0), particle_layout: int = 0,
                 fused_consumers: int = 0, xs_l2_persist: int = 0, resume_prefetch: int | None = None):
        L = lib()
        o = Options()
        L.nt_options_default(C.byref(o))
        o.device = device
        o.stream = stream
        o.mode = MODES[mode]
        o.deterministic = int(bool(deterministic))
        o.rank, o.nranks = rank, nranks
        self._uid = C.create_string_buffer(unique_id, 128) if unique_id else None
        o.nccl_unique_id = C.cast(self._uid, C.c_void_p) if self._uid else None
        o.A, o.molar_mass, o.e_min, o.w_min = A, molar_mass, e_min, w_min
        o.max_events_per_history = max_events
        o.ctas_per_sm = ctas_per_sm
        o.det_batch = det_batch
        o.refill_min = refill_min
        o.density_format = density_format
        o.layout = layout
        o.tally_mode = tally_mode
        o.defer_below = defer_below
        o.xs_search = xs_search
        o.boundary = boundary
        o.analog_absorption = analog
        o.roulette = roulette
        o.roulette_weight = roulette_weight
        o.decomposition = decomposition
        o.hot_x0, o.hot_y0, o.hot_nx, o.hot_ny = hot_window
        o.particle_layout = particle_layout
        o.fused_consumers = fused_consumers
        o.xs_l2_persist = xs_l2_persist
        if resume_prefetch is not None:          # None: the library default
            o.resume_prefetch = resume_prefetch
        h = C.c_void_p()
        st = L.nt_create(C.byref(o), C.byref(h))
        if st != NT_OK:
            raise NeutralError(st, "nt_create failed")
        self._h = h
        self._stream = stream or 0
        self.nx = self.ny = 0
        self.n_local = 0

    # -- helpers ---------------------------------------------------------------------------
    def _order(self, *arrays):
        """Synchronise torch's current stream for CUDA tensors not on the context stream."""
        for a in arrays:
            if getattr(a, "is_cuda", False):
                import torch
                cur = torch.cuda.current_stream(a.device)
                if self._stream == 0 or cur.cuda_stream != self._stream:
                    cur.synchronize()

    def _check(self, st: int, what: str, allow=()):
        if st != NT_OK and st not in allow:
            raise NeutralError(st, f"{what}: {lib().nt_last_error(self._h).decode()}")
        return st

    def close(self):
        if getattr(self, "_h", None):
            lib().nt_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    # -- the five calls of the boundary -------------------------------------------------------
    def init_mesh(self, nx: int, ny: int, width: float, height: float, density):
        dens = _f64(density)
        self._order(dens)
        p, keep = _ptr(dens)
        self._check(lib().nt_init_mesh(self._h, nx, ny, width, height, p), "nt_init_mesh")
        self.nx, self.ny = nx, ny

    def load_cross_sections(self, scatter_keys, scatter_vals, capture_keys, capture_vals):
        arrs = [_f64(a) for a in (scatter_keys, scatter_vals, capture_keys, capture_vals)]
        self._order(*arrs)
        ps = [_ptr(a)[0] for a in arrs]
        self._check(lib().nt_load_cross_sections(self._h, ps[0], ps[1], len(arrs[0]), ps[2], ps[3],
                                                 len(arrs[2])), "nt_load_cross_sections")

    def inject_particles(self, n_total: int, first_id: int, n_local: int, source, initial_energy: float,
                         seed: int):
        sx, sy, sw, sh = source
        self._check(lib().nt_inject_particles(self._h, n_total, first_id, n_local, sx, sy, sw, sh,
                                              initial_energy, seed), "nt_inject_particles")
        self.n_local = n_local

    def run_timestep(self, dt: float) -> dict:
        s = StepStats()
        st = self._check(lib().nt_run_timestep(self._h, dt, C.byref(s)), "nt_run_timestep",
                         allow=STEP_ANOMALIES)
        d = {n: getattr(s, n) for n, _ in StepStats._fields_}
        d["status"] = st
        d["events"] = d["n_facets"] + d["n_collisions"] + d["n_census"]
        return d

    # -- slab decomposition driven by the caller (decomposition = 1) ------------------------
    def slab_begin(self, dt: float):
        self._check(lib().nt_slab_begin(self._h, dt), "nt_slab_begin")

    def slab_round(self) -> int:
        n = C.c_int64()
        self._check(lib().nt_slab_round(self._h, C.byref(n)), "nt_slab_round")
        return n.value

    def slab_export(self, n_max: int):
        rb = lib().nt_slab_record_bytes()
        buf = np.empty(max(1, n_max) * rb, dtype=np.uint8)
        nl, nr = C.c_int64(), C.c_int64()
        self._check(lib().nt_slab_export(self._h, buf.ctypes.data, n_max, C.byref(nl), C.byref(nr)),
                    "nt_slab_export")
        return buf[: (nl.value + nr.value) * rb].reshape(-1, rb), nl.value, nr.value

    def slab_import(self, recs: np.ndarray):
        recs = np.ascontiguousarray(recs, dtype=np.uint8)
        self._check(lib().nt_slab_import(self._h, recs.ctypes.data, recs.shape[0] if recs.ndim == 2 else 0),
                    "nt_slab_import")

    def slab_end(self) -> dict:
        s = StepStats()
        st = self._check(lib().nt_slab_end(self._h, C.byref(s)), "nt_slab_end", allow=STEP_ANOMALIES)
        d = {n: getattr(s, n) for n, _ in StepStats._fields_}
        d["status"] = st
        d["events"] = d["n_facets"] + d["n_collisions"] + d["n_census"]
        return d

    def read_tally(self, out=None, reduced: bool = True):
        if out is None:
            out = np.empty((self.ny, self.nx), dtype=np.float64)
        self._order(out)
        p, _ = _ptr(out)
        self._check(lib().nt_read_tally(self._h, p, int(reduced)), "nt_read_tally")
        return out

    # -- verification / checkpoint ------------------------------------------------------------
    def particle_slots(self) -> int:
        n = C.c_int64()
        self._check(lib().nt_particle_slots(self._h, C.byref(n)), "nt_particle_slots")
        return n.value

    def read_particles(self, first: int = 0, count: int | None = None) -> dict:
        if count is None:
            count = self.particle_slots() - first
        out = {n: np.empty(count, dtype=t) for n, t in PARTICLE_FIELDS}
        v = ParticlesView(*[out[n].ctypes.data for n, _ in PARTICLE_FIELDS])
        self._check(lib().nt_read_particles(self._h, first, count, C.byref(v)), "nt_read_particles")
        return out

    def write_particles(self, first: int, fields: dict):
        count = len(next(iter(fields.values())))
        keep = {n: np.ascontiguousarray(fields[n], dtype=t) for n, t in PARTICLE_FIELDS if n in fields}
        v = ParticlesView(*[keep[n].ctypes.data if n in keep else None for n, _ in PARTICLE_FIELDS])
        self._check(lib().nt_write_particles(self._h, first, count, C.byref(v)), "nt_write_particles")

    def mesh_bytes(self) -> int:
        """Device bytes held for the mesh (density + tally buffers)."""
        return int(lib().nt_debug_mesh_bytes(self._h))

    def density_format(self) -> tuple[str, int]:
        """(storage nt_init_mesh chose: "u8" / "u16" / "f64", distinct density values found)."""
        n = C.c_int32(0)
        f = int(lib().nt_debug_density_format(self._h, C.byref(n)))
        return {2: "u8", 1: "u16", 0: "f64"}.get(f, str(f)), int(n.value)

    def xs_rows(self) -> int:
        """Bit mask of the loaded tables with direct bucket rows (1 scatter, 2 capture)."""
        return int(lib().nt_debug_xs_rows(self._h))

    def debug_threefry(self, inputs: np.ndarray) -> np.ndarray:
        inp = np.ascontiguousarray(inputs, dtype=np.uint64).reshape(-1, 4)
        out = np.empty((len(inp), 2), dtype=np.uint64)
        self._check(lib().nt_debug_threefry(self._h, inp.ctypes.data, len(inp), out.ctypes.data),
                    "nt_debug_threefry")
        return out

    def debug_xs(self, energies: np.ndarray):
        e = np.ascontiguousarray(energies, dtype=np.float64)
        os_, oa = np.empty_like(e), np.empty_like(e)
        self._check(lib().nt_debug_xs(self._h, e.ctypes.data, len(e), os_.ctypes.data, oa.ctypes.data),
                    "nt_debug_xs")
        return os_, oa


def setup(cfg, *, density=None, tables=None, first_id: int = 0, n_local: int | None = None,
          **opts) -> Tracker:
    """Create a Tracker for a workloads.Config: mesh, tables and injected particles."""
    from . import workloads as wl
    phys = dict(boundary=cfg.boundary, analog=cfg.analog, roulette=cfg.roulette,
                roulette_weight=cfg.roulette_weight)
    phys.update({k: opts.pop(k) for k in list(opts) if k in phys})
    t = Tracker(A=cfg.A, molar_mass=cfg.molar_mass, e_min=cfg.e_min, w_min=cfg.w_min, **phys, **opts)
    t.init_mesh(cfg.nx, cfg.ny, cfg.width, cfg.height, wl.density(cfg) if density is None else density)
    t.load_cross_sections(*(wl.tables(cfg) if tables is None else tables))
    if n_local is None:
        n_local = cfg.n_particles - first_id
    t.inject_particles(cfg.n_particles, first_id, n_local, cfg.source, cfg.e0, cfg.seed)
    return t
