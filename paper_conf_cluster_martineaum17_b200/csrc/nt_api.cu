// nt_api.cu -- the C ABI (include/neutral_b200.h): context state machine, device
// allocations, argument validation, step orchestration, NCCL reduction.
//
// Host-side orchestration only; every step of the method runs in the kernels of
// nt_kernels.cu / nt_event.cu.
#include <nccl.h>

#include <atomic>
#include <cmath>
#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <string>
#include <vector>

#include <nvtx3/nvToolsExt.h>

#include "../../include/neutral_b200.h"
#include "nt_event.h"
#include "nt_internal.h"

using namespace nt;

namespace {

enum Stage { ST_CREATED = 0, ST_MESH = 1, ST_XS = 2, ST_PARTICLES = 3, ST_STEPPED = 4 };

// Device buffer that only grows.  ensure() frees the old allocation before it allocates
// the new one, so a caller whose state points into the buffer lowers its stage first
// (nt_load_cross_sections, nt_inject_particles): after a failed ensure nothing refers to
// freed memory.
struct DevBuf {
  void* p = nullptr;
  size_t bytes = 0;
  cudaError_t ensure(size_t b) {
    if (b <= bytes && p) return cudaSuccess;
    if (p) cudaFree(p);
    p = nullptr;
    bytes = 0;
    if (b == 0) return cudaSuccess;
    cudaError_t e = nt::device_malloc(&p, b);
    if (e == cudaSuccess) bytes = b;
    return e;
  }
  void release() {
    if (p) cudaFree(p);
    p = nullptr;
    bytes = 0;
  }
  template <class T> T* as() const { return static_cast<T*>(p); }
};

// NVTX range over a C-ABI call (nsys / ncu --nvtx show the library's phases by name; the
// header-only NVTX v3 costs nothing without a tool attached).
struct NvtxRange {
  explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
  ~NvtxRange() { nvtxRangePop(); }
};

}  // namespace

namespace nt {
static std::atomic<long long> g_device_allocs{0};
cudaError_t device_malloc(void** p, size_t bytes) {
  ++g_device_allocs;
  return cudaMalloc(p, bytes);
}
}  // namespace nt

struct nt_ctx {
  nt_options opt{};
  std::string err;
  int stage = ST_CREATED;
  int device = 0;
  int sm_count = 0;
  cudaStream_t stream = nullptr;
  bool own_stream = false;
  cudaEvent_t ev[6] = {};
  cudaStream_t aux = nullptr;            // nt_init_mesh: checks chunks while the next uploads
  cudaEvent_t chunk_ev[9] = {};
  DevBuf dset;                           // distinct-value set (kDistinctSlots u64)
  int32_t dens_distinct = 0;             // distinct density values found by nt_init_mesh
  ncclComm_t comm = nullptr;
  Phys ph{};
  // step statistics as doubles: [SU_COUNT u64 counts][SF_COUNT sums] (device, and a
  // pinned host copy read once per step)
  DevBuf stats_d;
  double* stats_h = nullptr;
  // mesh
  int32_t nx = 0, ny = 0;
  int32_t x0 = 0, nxs = 0;               // stored columns [x0, x0 + nxs) (x-slabs: own + halo)
  double W = 0, H = 0;
  DevBuf rho, tally, tally_red, ex, ey;  // tally_red: the cross-rank sum (comm only)
  DevBuf rho_code, nd_tab, enc_keys;     // lossless density encoding
  DevBuf blk;                            // block map of the u8 codes (Mesh::blk)
  int blk_shift = 0, blk_nbx = 0, blk_n = 0;   // blk_n = 0: no block map
  DevBuf rho_st, tally_rm;               // f64 density in storage layout; row-major staging
  DevBuf tally_full;                     // x-slabs: the whole-mesh tally assembled at read time
  int dens_fmt = kDensF64, dens_codes = 0;
  int tiled = 0, ntx = 0;                // storage layout of tally / density (cell_index)
  int64_t cells_st = 0;                  // cells in the storage layout (tiles padded)
  // tables
  DevBuf xs;
  size_t xs_bytes = 0;                   // bytes of xs in use (keys, values, indexes, pairs)
  size_t xs_persist_bytes = 0;           // xs_l2_persist: the device's persisting L2 carve-out
  Tables tables{};
  const double2* xs_row[2] = {nullptr, nullptr};   // direct bucket rows (xs_search 0, 4), if built
  const double2* xs_urow = nullptr;                 // unionised grid rows (xs_search 0), if built
  // particles
  int64_t n_total = 0, first_id = 0, n_local = 0;
  uint64_t seed = 0;
  DevBuf soa;
  DevBuf aos;                            // particle_layout 1: AoS records during the step
  Soa p{};
  int32_t* defer_q = nullptr;            // regime-parking queue (in soa)
  DevBuf park_rec;                       // resume_prefetch: queue-ordered parked records
  int64_t park_cap = 0;
  // x-slab decomposition (decomposition 1)
  int64_t n_cap = 0;                     // particle-store capacity (n_total with slabs)
  int32_t slab_lo = 0, slab_hi = 0;      // owned mesh columns
  int32_t* arr_q = nullptr;              // arrivals queued for the next round (in soa)
  int32_t* out_q = nullptr;              // emigrants of the running round (in soa)
  int64_t n_arr = 0;                     // arrivals waiting for the next round
  int32_t* free_q = nullptr;             // slots vacated by emigrants, reused by arrivals
  int64_t n_free = 0;
  int slab_round = 0;
  uint32_t slab_launches = 0;
  double slab_dt = 0.0;
  DevBuf slab_buf, slab_rbuf;            // packed emigrant / received records
  // step scratch: [counter][stats_u][stats_f]; per-thread f64 statistic slots
  DevBuf scratch, slots;
  // deterministic mode
  DevBuf rec_key, rec_val, rec_key2, rec_val2, sort_tmp, backup;
  unsigned long long rec_cap = 0;
  // event mode
  EventState* evs = nullptr;
};

namespace {

// The tables as the kernels see them under the xs_search option: 0 the unionised grid and
// the direct bucket rows where the loader could build them (else the bucket index), 1 no
// index (plain binary search), 2 and 3 the bucket index (2's walk is a kernel
// instantiation), 4 the direct bucket rows per table.
// xs_l2_persist: an L2 access-policy window marks the cross-section buffer persisting on the
// context stream while the step's tracking kernels run (cleared afterwards, also on error
// paths), so the table lines are not evicted by the tally and particle-store traffic.  The
// device-wide persisting carve-out is sized at nt_load_cross_sections.
struct XsWindow {
  nt_ctx* c;
  bool on = false;
  explicit XsWindow(nt_ctx* ctx);
  ~XsWindow();
};

static Tables xs_tables(const nt_ctx* c) {
  Tables t = c->tables;
  if (c->opt.xs_search == 1) {
    t.s.nb = 0;
    t.c.nb = 0;
  } else if (c->opt.xs_search == 4) {     // direct rows per table only
    t.s.row = c->xs_row[0];
    t.c.row = c->xs_row[1];
  } else if (c->opt.xs_search == 0) {     // unionised grid, the direct rows where it does not apply
    t.urow = c->xs_urow;
    t.s.row = c->xs_row[0];
    t.c.row = c->xs_row[1];
  }
  return t;
}

XsWindow::XsWindow(nt_ctx* ctx) : c(ctx) {
  if (!c->opt.xs_l2_persist || c->xs_bytes == 0 || c->xs_persist_bytes == 0) return;
  int maxwin = 0;
  cudaDeviceGetAttribute(&maxwin, cudaDevAttrMaxAccessPolicyWindowSize, c->device);
  cudaStreamAttrValue v{};
  v.accessPolicyWindow.base_ptr = c->xs.p;
  v.accessPolicyWindow.num_bytes = c->xs_bytes < (size_t)maxwin ? c->xs_bytes : (size_t)maxwin;
  const double r = (double)c->xs_persist_bytes / (double)v.accessPolicyWindow.num_bytes;
  v.accessPolicyWindow.hitRatio = (float)(r < 1.0 ? r : 1.0);
  v.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
  v.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
  on = cudaStreamSetAttribute(c->stream, cudaStreamAttributeAccessPolicyWindow, &v) == cudaSuccess;
  if (!on) cudaGetLastError();
}

XsWindow::~XsWindow() {
  if (!on) return;
  cudaStreamAttrValue v{};
  v.accessPolicyWindow.num_bytes = 0;     // no window: later work on the stream is unaffected
  cudaStreamSetAttribute(c->stream, cudaStreamAttributeAccessPolicyWindow, &v);
}

nt_status fail(nt_ctx* c, nt_status s, const char* fmt, ...) {
  if (c) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    c->err = buf;
  }
  return s;
}

#define NT_CUDA(c, call)                                                                \
  do {                                                                                  \
    cudaError_t e_ = (call);                                                            \
    if (e_ != cudaSuccess)                                                              \
      return fail((c), e_ == cudaErrorMemoryAllocation ? NT_ERR_OOM : NT_ERR_CUDA,      \
                  "%s: %s (%s:%d)", #call, cudaGetErrorString(e_), __FILE__, __LINE__); \
  } while (0)

#define NT_NCCL(c, call)                                                                \
  do {                                                                                  \
    ncclResult_t r_ = (call);                                                           \
    if (r_ != ncclSuccess)                                                              \
      return fail((c), NT_ERR_NCCL, "%s: %s", #call, ncclGetErrorString(r_));           \
  } while (0)

bool is_fin(double v) { return std::isfinite(v); }

// Copy n bytes from a host-or-device pointer into device memory.
cudaError_t copy_in(void* dst, const void* src, size_t n, cudaStream_t s) {
  if (n == 0) return cudaSuccess;
  return cudaMemcpyAsync(dst, src, n, cudaMemcpyDefault, s);
}

// Read a host-or-device array into a host vector (for validation).
template <class T>
cudaError_t fetch(std::vector<T>& out, const T* src, int64_t n, cudaStream_t s) {
  out.resize((size_t)n);
  cudaError_t e = cudaMemcpyAsync(out.data(), src, sizeof(T) * (size_t)n, cudaMemcpyDefault, s);
  if (e != cudaSuccess) return e;
  return cudaStreamSynchronize(s);
}

size_t align256(size_t b) { return (b + 255) & ~(size_t)255; }

void init_phys(nt_ctx* c) {
  const double A = c->opt.A;
  Phys& p = c->ph;
  p.A = A;
  p.AA = A * A;
  p.twoA = 2.0 * A;
  p.Ap1 = A + 1.0;
  p.Am1 = A - 1.0;
  p.Ap1sq = (A + 1.0) * (A + 1.0);
  p.f = (A * A + 1.0) / ((A + 1.0) * (A + 1.0));
  p.cn = kAvogadro / c->opt.molar_mass;
  p.kv = (2.0 * kEv) / kNeutronMass;
  p.e_min = c->opt.e_min;
  p.w_min = c->opt.w_min;
  p.w_roul = c->opt.roulette_weight;
  p.vacuum = c->opt.boundary;
  p.analog = c->opt.analog_absorption;
  p.roulette = c->opt.roulette;
}

}  // namespace

// =========================================================================================
extern "C" {

int32_t nt_abi_version(void) { return NT_ABI_VERSION; }

const char* nt_build_info(void) {
  return "neutral_b200 sm_100a; nvcc -fmad=false -O3; history+event tracking; "
         "fp64 RED tally / deterministic record-sort tally; NCCL allreduce";
}

const char* nt_status_string(nt_status s) {
  switch (s) {
    case NT_OK: return "NT_OK";
    case NT_ERR_ARG: return "NT_ERR_ARG";
    case NT_ERR_STATE: return "NT_ERR_STATE";
    case NT_ERR_OOM: return "NT_ERR_OOM";
    case NT_ERR_CUDA: return "NT_ERR_CUDA";
    case NT_ERR_NCCL: return "NT_ERR_NCCL";
    case NT_ERR_XS_RANGE: return "NT_ERR_XS_RANGE";
    case NT_ERR_NONFINITE: return "NT_ERR_NONFINITE";
    case NT_ERR_EVENT_CAP: return "NT_ERR_EVENT_CAP";
    case NT_ERR_UNSUPPORTED: return "NT_ERR_UNSUPPORTED";
  }
  return "NT_ERR_UNKNOWN";
}

nt_status nt_options_default(nt_options* opt) {
  if (!opt) return NT_ERR_ARG;
  std::memset(opt, 0, sizeof *opt);
  opt->nranks = 1;
  opt->A = 1.0;
  opt->molar_mass = 1.0e-3;
  opt->e_min = 1.0;
  opt->w_min = 1.0e-3;
  opt->max_events_per_history = 1000000000ll;
  opt->det_batch = 65536;
  opt->refill_min = 4;
  opt->defer_below = 8;
  return NT_OK;
}

nt_status nt_get_unique_id(void* out128) {
  if (!out128) return NT_ERR_ARG;
  ncclUniqueId id;
  if (ncclGetUniqueId(&id) != ncclSuccess) return NT_ERR_NCCL;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId size");
  std::memcpy(out128, &id, sizeof id);
  return NT_OK;
}

const char* nt_last_error(const nt_ctx* ctx) {
  if (!ctx) return "null context";
  return ctx->err.c_str();
}

nt_status nt_create(const nt_options* opt_in, nt_ctx** out) {
  if (!out) return NT_ERR_ARG;
  *out = nullptr;
  nt_options def;
  nt_options_default(&def);
  nt_options opt = opt_in ? *opt_in : def;
  if (opt.nranks <= 0) opt.nranks = 1;
  if (opt.A == 0.0) opt.A = def.A;
  if (opt.molar_mass == 0.0) opt.molar_mass = def.molar_mass;
  if (opt.e_min == 0.0) opt.e_min = def.e_min;
  if (opt.w_min == 0.0) opt.w_min = def.w_min;
  if (opt.max_events_per_history <= 0) opt.max_events_per_history = def.max_events_per_history;
  if (opt.det_batch <= 0) opt.det_batch = def.det_batch;
  if (opt.det_batch > 65536) opt.det_batch = 65536;
  if (opt.refill_min <= 0) opt.refill_min = def.refill_min;
  if (opt.refill_min > 32) opt.refill_min = 32;
  if (opt.defer_below == 0) opt.defer_below = def.defer_below;
  if (opt.defer_below < 0 || opt.defer_below > 33) return NT_ERR_ARG;
  if (opt.xs_search < 0 || opt.xs_search > 4) return NT_ERR_ARG;
  if (opt.boundary < 0 || opt.boundary > 1 || opt.analog_absorption < 0 ||
      opt.analog_absorption > 1 || opt.roulette < 0 || opt.roulette > 1)
    return NT_ERR_ARG;
  if (opt.roulette_weight == 0.0) opt.roulette_weight = 2.0 * opt.w_min;
  if (opt.roulette && !(opt.roulette_weight > opt.w_min) ) return NT_ERR_ARG;
  if (!(opt.A > 0.0) || !is_fin(opt.A) || !(opt.molar_mass > 0.0) || !is_fin(opt.molar_mass) ||
      !(opt.e_min > 0.0) || !(opt.w_min >= 0.0) || opt.mode < 0 || opt.mode > 1 ||
      opt.rank < 0 || opt.rank >= opt.nranks || opt.density_format < 0 ||
      opt.density_format > 2 || opt.layout < 0 || opt.layout > 1 || opt.tally_mode < 0 ||
      opt.tally_mode > 3)
    return NT_ERR_ARG;
  if (opt.particle_layout < 0 || opt.particle_layout > 1) return NT_ERR_ARG;
  if (opt.fused_consumers < 0 || opt.fused_consumers > 8) return NT_ERR_ARG;
  if (opt.xs_l2_persist < 0 || opt.xs_l2_persist > 1) return NT_ERR_ARG;
  if (opt.resume_prefetch < 0 || opt.resume_prefetch > 1) return NT_ERR_ARG;
  if (opt.tally_mode == 3 && (opt.hot_x0 < 0 || opt.hot_y0 < 0 || opt.hot_nx < 1 || opt.hot_ny < 1 ||
                              (int64_t)opt.hot_nx * opt.hot_ny > kHotCells))
    return NT_ERR_ARG;
  // nranks > 1 needs a communicator, except for x-slabs driven by the caller (nt_slab_*)
  if (opt.nranks > 1 && !opt.nccl_unique_id && opt.decomposition != 1) return NT_ERR_ARG;
  if (opt.decomposition < 0 || opt.decomposition > 1) return NT_ERR_ARG;

  nt_ctx* c = new nt_ctx();
  c->opt = opt;
  c->device = opt.device;
  cudaError_t e = cudaSetDevice(opt.device);
  if (e != cudaSuccess) {
    delete c;
    return NT_ERR_CUDA;
  }
  cudaDeviceGetAttribute(&c->sm_count, cudaDevAttrMultiProcessorCount, opt.device);
  if (opt.stream) {
    c->stream = static_cast<cudaStream_t>(opt.stream);
  } else {
    if (cudaStreamCreateWithFlags(&c->stream, cudaStreamNonBlocking) != cudaSuccess) {
      delete c;
      return NT_ERR_CUDA;
    }
    c->own_stream = true;
  }
  for (auto& ev : c->ev) cudaEventCreate(&ev);
  for (auto& ev : c->chunk_ev) cudaEventCreateWithFlags(&ev, cudaEventDisableTiming);
  if (cudaStreamCreateWithFlags(&c->aux, cudaStreamNonBlocking) != cudaSuccess) {
    nt_destroy(c);
    return NT_ERR_CUDA;
  }
  if (cudaHostAlloc(reinterpret_cast<void**>(&c->stats_h), (SU_COUNT + SF_COUNT) * sizeof(double),
                    cudaHostAllocDefault) != cudaSuccess ||
      c->stats_d.ensure((SU_COUNT + SF_COUNT) * sizeof(double)) != cudaSuccess) {
    nt_destroy(c);
    return NT_ERR_OOM;
  }
  init_phys(c);
  if (opt.nccl_unique_id) {
    ncclUniqueId id;
    std::memcpy(&id, opt.nccl_unique_id, sizeof id);
    ncclResult_t r = ncclCommInitRank(&c->comm, opt.nranks, id, opt.rank);
    if (r != ncclSuccess) {
      nt_destroy(c);
      return NT_ERR_NCCL;
    }
  }
  *out = c;
  return NT_OK;
}

nt_status nt_destroy(nt_ctx* c) {
  if (!c) return NT_OK;
  cudaSetDevice(c->device);
  if (c->stream) cudaStreamSynchronize(c->stream);
  if (c->evs) event_state_destroy(c->evs);
  if (c->xs_persist_bytes) {            // xs_l2_persist: release the persisting lines and carve-out
    cudaCtxResetPersistingL2Cache();
    cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, 0);
  }
  for (DevBuf* b : {&c->slab_buf, &c->slab_rbuf, &c->rho_code, &c->blk, &c->nd_tab, &c->enc_keys, &c->rho_st, &c->tally_rm, &c->tally_full, &c->rho, &c->tally, &c->tally_red, &c->ex, &c->ey, &c->xs, &c->soa,
                    &c->scratch, &c->slots, &c->rec_key, &c->rec_val, &c->rec_key2, &c->rec_val2,
                    &c->sort_tmp, &c->backup, &c->stats_d, &c->aos, &c->park_rec, &c->dset})
    b->release();
  if (c->stats_h) cudaFreeHost(c->stats_h);
  for (auto& ev : c->ev)
    if (ev) cudaEventDestroy(ev);
  for (auto& ev : c->chunk_ev)
    if (ev) cudaEventDestroy(ev);
  if (c->aux) cudaStreamDestroy(c->aux);
  if (c->comm) ncclCommDestroy(c->comm);
  if (c->own_stream && c->stream) cudaStreamDestroy(c->stream);
  delete c;
  return NT_OK;
}

// ---- mesh ----------------------------------------------------------
// The density is copied straight into device memory, validated there, and -- when the map
// holds few distinct values (density_format 0) -- encoded losslessly as u8/u16 material
// codes plus a number-density table, so the tracker's per-facet gather is 1-2 B instead of
// 8 B and the map stays L2-resident.
nt_status nt_init_mesh(nt_ctx* c, int32_t nx, int32_t ny, double width, double height,
                       const double* density) {
  NvtxRange nvtx_("nt_init_mesh");
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (nx < 1 || ny < 1) return fail(c, NT_ERR_ARG, "nx, ny must be >= 1 (got %d, %d)", nx, ny);
  if ((int64_t)nx * (int64_t)ny > (1ll << 31))
    return fail(c, NT_ERR_ARG, "nx * ny must be <= 2^31");
  if (!(width > 0.0) || !(height > 0.0) || !is_fin(width) || !is_fin(height))
    return fail(c, NT_ERR_ARG, "width, height must be finite and > 0");
  if (!density) return fail(c, NT_ERR_ARG, "density is NULL");
  // x-slabs (decomposition 1): this rank stores only its columns [floor(r nx/P),
  // floor((r+1) nx/P)) plus a one-column halo on each side (the density of the cell a
  // particle steps into before it is handed over), so mesh memory scales as 1/P
  int32_t x0 = 0, nxs = nx;
  if (c->opt.decomposition == 1) {
    const int64_t P = c->opt.nranks, r = c->opt.rank;
    const int32_t lo = (int32_t)((r * nx) / P), hi = (int32_t)(((r + 1) * nx) / P);
    x0 = lo > 0 ? lo - 1 : 0;
    nxs = (hi < nx ? hi + 1 : nx) - x0;
  }
  const int64_t cells = (int64_t)nxs * (int64_t)ny;   // stored cells
  c->stage = ST_CREATED;
  const int tiled = c->opt.layout == 0 ? 1 : 0;
  const int ntx = (nxs + 3) / 4, nty = (ny + 3) / 4;
  const int64_t cells_st = tiled ? (int64_t)ntx * nty * 16 : cells;
  if (cells_st >= (1ll << 32))
    return fail(c, NT_ERR_ARG, "the tiled mesh storage must hold < 2^32 cells");
  Mesh ml{};                              // the stored sub-mesh, in its own columns
  ml.nx = nxs;
  ml.gnx = nxs;
  ml.ny = ny;
  ml.tiled = tiled;
  ml.ntx = ntx;
  ml.strip = 16 * ntx;
  NT_CUDA(c, c->rho.ensure((size_t)cells * 8));
  NT_CUDA(c, c->tally.ensure((size_t)cells_st * 8));
  const bool reduce_in_step = c->comm && c->opt.decomposition != 1;
  if (reduce_in_step) NT_CUDA(c, c->tally_red.ensure((size_t)cells_st * 8));
  NT_CUDA(c, c->ex.ensure(((size_t)nx + 1) * 8));
  NT_CUDA(c, c->ey.ensure(((size_t)ny + 1) * 8));
  NT_CUDA(c, c->scratch.ensure(1024));
  // Upload in chunks on the context stream; each chunk is validated and its distinct values
  // collected (check_distinct_kernel) on the aux stream while the next chunk is copied, so
  // the device work hides under the H2D transfer.
  const bool codes = c->opt.density_format == 0 || c->opt.density_format == 2;
  unsigned long long* bad = reinterpret_cast<unsigned long long*>(c->scratch.as<char>() + 160);  // [3]
  NT_CUDA(c, c->dset.ensure((size_t)kDistinctSlots * 8));
  unsigned long long* dset = c->dset.as<unsigned long long>();
  NT_CUDA(c, cudaMemsetAsync(bad, 0, 24, c->stream));
  NT_CUDA(c, cudaMemsetAsync(dset, 0xff, (size_t)kDistinctSlots * 8, c->stream));
  if (nxs == nx) {
    constexpr int kChunks = 8;
    const int64_t per = (cells + kChunks - 1) / kChunks;
    for (int k = 0; k < kChunks; ++k) {
      const int64_t a = (int64_t)k * per, n = a < cells ? (cells - a < per ? cells - a : per) : 0;
      if (n <= 0) break;
      NT_CUDA(c, cudaMemcpyAsync(c->rho.as<double>() + a, density + a, (size_t)n * 8, cudaMemcpyDefault, c->stream));
      NT_CUDA(c, cudaEventRecord(c->chunk_ev[k], c->stream));
      NT_CUDA(c, cudaStreamWaitEvent(c->aux, c->chunk_ev[k], 0));
      if (codes) NT_CUDA(c, launch_check_distinct(c->rho.as<double>() + a, n, bad, dset, c->aux));
      else NT_CUDA(c, launch_density_check(c->rho.as<double>() + a, n, bad, c->aux));
    }
    NT_CUDA(c, cudaEventRecord(c->chunk_ev[8], c->aux));
    NT_CUDA(c, cudaStreamWaitEvent(c->stream, c->chunk_ev[8], 0));
  } else {
    NT_CUDA(c, cudaMemcpy2DAsync(c->rho.p, (size_t)nxs * 8, density + x0, (size_t)nx * 8,
                                 (size_t)nxs * 8, (size_t)ny, cudaMemcpyDefault, c->stream));
    if (codes) NT_CUDA(c, launch_check_distinct(c->rho.as<double>(), cells, bad, dset, c->stream));
    else NT_CUDA(c, launch_density_check(c->rho.as<double>(), cells, bad, c->stream));
  }
  unsigned long long hb[3] = {0, 0, 0};
  NT_CUDA(c, cudaMemcpyAsync(hb, bad, 24, cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  if (hb[0] != 0)
    return fail(c, NT_ERR_ARG, "%llu density values are not finite and >= 0", hb[0]);
  // distinct density values (for the lossless encoding): sorted from the set, or -- more
  // than kDistinctSlots / 2 of them -- by sorting every cell's bit pattern
  int fmt = kDensF64, nu = 0;
  if (codes) {
    if (hb[2] == 0) {
      nu = (int)hb[1];
      NT_CUDA(c, c->enc_keys.ensure((size_t)kDistinctSlots * 8));
      NT_CUDA(c, launch_distinct_sort(dset, c->enc_keys.as<unsigned long long>(), c->stream));
    } else {
      size_t tmp = 0;
      NT_CUDA(c, c->enc_keys.ensure((size_t)cells * 16));
      unsigned long long* k0 = c->enc_keys.as<unsigned long long>();
      unsigned long long* k1 = k0 + cells;
      int* d_count = reinterpret_cast<int*>(c->scratch.as<char>() + 8);
      NT_CUDA(c, density_distinct(c->rho.as<double>(), cells, k0, k1, nullptr, tmp, d_count, c->stream));
      NT_CUDA(c, c->sort_tmp.ensure(tmp));
      NT_CUDA(c, density_distinct(c->rho.as<double>(), cells, k0, k1, c->sort_tmp.p, tmp, d_count, c->stream));
      int hn = 0;
      NT_CUDA(c, cudaMemcpyAsync(&hn, d_count, 4, cudaMemcpyDeviceToHost, c->stream));
      NT_CUDA(c, cudaStreamSynchronize(c->stream));
      nu = hn;
    }
    if (nu <= 256) fmt = kDensU8;
    else if (nu <= 65536) fmt = kDensU16;
  }
  if (fmt != kDensF64) {
    const size_t cb = (size_t)cells_st * (fmt == kDensU8 ? 1 : 2);
    NT_CUDA(c, c->rho_code.ensure(cb));
    NT_CUDA(c, cudaMemsetAsync(c->rho_code.p, 0, cb, c->stream));        // tile padding
    NT_CUDA(c, c->nd_tab.ensure((size_t)nu * 8));
    NT_CUDA(c, launch_encode(c->rho.as<double>(), cells, ml, c->enc_keys.as<unsigned long long>(),
                             nu, c->ph.cn, fmt, c->rho_code.p, c->nd_tab.as<double>(), c->stream));
  }
  // block map (density_format 0, u8 codes with a spare code for "mixed"): the smallest
  // power-of-two block side >= 4 whose map fits kBlkMax bytes of shared memory
  int blk_shift = 0, blk_nbx = 0, blk_n = 0;
  if (fmt == kDensU8 && nu < (int)kBlkMixed && c->opt.density_format == 0) {
    for (int s = 2; s < 31; ++s) {
      const int64_t bx = ((int64_t)nxs + (1 << s) - 1) >> s, by = ((int64_t)ny + (1 << s) - 1) >> s;
      if (bx * by <= kBlkMax) {
        blk_shift = s;
        blk_nbx = (int)bx;
        blk_n = (int)(bx * by);
        break;
      }
    }
    Mesh mb = ml;
    mb.bshift = blk_shift;
    mb.nbx = blk_nbx;
    mb.nblk = blk_n;
    NT_CUDA(c, c->blk.ensure(align256((size_t)blk_n)));
    NT_CUDA(c, launch_block_map(c->rho_code.as<uint8_t>(), mb, c->blk.as<uint8_t>(), c->stream));
  }
  if (fmt == kDensF64 && tiled) {
    NT_CUDA(c, c->rho_st.ensure((size_t)cells_st * 8));
    NT_CUDA(c, cudaMemsetAsync(c->rho_st.p, 0, (size_t)cells_st * 8, c->stream));
    NT_CUDA(c, launch_relayout(c->rho.as<double>(), c->rho_st.as<double>(), cells, ml, true, c->stream));
  }
  NT_CUDA(c, cudaMemsetAsync(c->tally.p, 0, (size_t)cells_st * 8, c->stream));
  if (reduce_in_step) NT_CUDA(c, cudaMemsetAsync(c->tally_red.p, 0, (size_t)cells_st * 8, c->stream));
  launch_edges(c->ex.as<double>(), nx, width, c->ey.as<double>(), ny, height, c->stream);
  NT_CUDA(c, cudaGetLastError());
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  c->dens_fmt = fmt;
  c->dens_distinct = nu;
  c->dens_codes = nu;
  c->blk_shift = blk_shift;
  c->blk_nbx = blk_nbx;
  c->blk_n = blk_n;
  c->tiled = tiled;
  c->ntx = ntx;
  c->cells_st = cells_st;
  c->nx = nx;
  c->ny = ny;
  c->x0 = x0;
  c->nxs = nxs;
  c->W = width;
  c->H = height;
  c->stage = ST_MESH;
  return NT_OK;
}

// ---- cross sections ---------------------------------------------------------
nt_status nt_load_cross_sections(nt_ctx* c, const double* sk, const double* sv, int64_t ns,
                                 const double* ck, const double* cv, int64_t nc) {
  NvtxRange nvtx_("nt_load_cross_sections");
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->stage < ST_MESH) return fail(c, NT_ERR_STATE, "nt_init_mesh must come first");
  if (ns < 2 || nc < 2 || ns > (1ll << 30) || nc > (1ll << 30))
    return fail(c, NT_ERR_ARG, "table sizes must be in [2, 2^30]");
  if (!sk || !sv || !ck || !cv) return fail(c, NT_ERR_ARG, "table pointer is NULL");
  c->stage = ST_MESH;           // the tables are replaced: later stages are invalid from here
  const double* src[4] = {sk, sv, ck, cv};
  const int64_t len[4] = {ns, ns, nc, nc};
  // host (pageable or pinned) tables are validated and indexed in place and copied once;
  // device and managed tables are fetched to the host first (the fetch is ordered behind
  // earlier work on the context stream, which may still be writing a managed table)
  std::vector<double> hv[4];
  const double* h[4];
  for (int k = 0; k < 4; ++k) {
    cudaPointerAttributes pa;
    if (cudaPointerGetAttributes(&pa, src[k]) == cudaSuccess &&
        (pa.type == cudaMemoryTypeDevice || pa.type == cudaMemoryTypeManaged)) {
      NT_CUDA(c, fetch(hv[k], src[k], len[k], c->stream));
      h[k] = hv[k].data();
    } else {
      cudaGetLastError();   // clear a failed attribute query (plain host pointer on old drivers)
      h[k] = src[k];
    }
  }
  for (int k = 0; k < 4; k += 2) {
    for (int64_t j = 0; j < len[k]; ++j) {
      if (!is_fin(h[k][j])) return fail(c, NT_ERR_ARG, "table %d key %lld not finite", k / 2, (long long)j);
      if (j > 0 && !(h[k][j] > h[k][j - 1]))
        return fail(c, NT_ERR_ARG, "table %d keys not strictly increasing at %lld", k / 2, (long long)j);
      if (!is_fin(h[k + 1][j]) || !(h[k + 1][j] >= 0.0))
        return fail(c, NT_ERR_ARG, "table %d value %lld not finite and >= 0", k / 2, (long long)j);
    }
  }
  // bucket indexes over the IEEE bit patterns of the (positive) keys
  uint64_t base[2] = {0, 0};
  int32_t shift[2] = {0, 0}, nbk[2] = {0, 0};
  for (int t = 0; t < 2; ++t) {
    const double* k = h[2 * t];
    const int64_t n = len[2 * t];
    if (!(k[0] > 0.0)) continue;                       // index needs positive keys
    uint64_t b0, b1;
    std::memcpy(&b0, &k[0], 8);
    std::memcpy(&b1, &k[n - 1], 8);
    const uint64_t range = b1 - b0;
    // about four buckets per key (the bit patterns of log-spaced keys are linear within a
    // binade, so the keys per bucket vary by 2x): a bucket then almost always spans at most
    // one key and the lookup needs no search loop (xs_lookup)
    int64_t target = 4 * n;
    if (target > (1ll << 22)) target = 1ll << 22;
    int s = 0;
    while ((range >> s) >= (uint64_t)target) ++s;
    const int64_t nb = (int64_t)(range >> s) + 1;
    base[t] = b0;
    shift[t] = s;
    nbk[t] = (int32_t)nb;
  }
  // Device buffer: keys, values (as given), the bucket index [nb + 1], the interleaved
  // (key, value) pairs [n + 1] and the direct bucket rows [nb] (xs_search 0, 4).  Only the
  // caller's four arrays cross PCIe; the index, pairs and rows are built on the device
  // (xs_prepare: the index by a binary search per bucket, the same bins as a sweep).
  // unionised grid over both tables (xs_search 0): one bucketing, fine enough for the
  // denser table, over the union of both key ranges
  uint64_t ubase = 0;
  int32_t ushift = 0;
  int64_t unb = 0;
  if (nbk[0] > 0 && nbk[1] > 0) {
    uint64_t a0, a1, c0, c1;
    std::memcpy(&a0, &h[0][0], 8);
    std::memcpy(&a1, &h[0][len[0] - 1], 8);
    std::memcpy(&c0, &h[2][0], 8);
    std::memcpy(&c1, &h[2][len[2] - 1], 8);
    const uint64_t lo = a0 < c0 ? a0 : c0, hi = a1 > c1 ? a1 : c1;
    int64_t target = 4 * (len[0] > len[2] ? len[0] : len[2]);
    if (target > (1ll << 22)) target = 1ll << 22;
    int sh = 0;
    while (((hi - lo) >> sh) >= (uint64_t)target) ++sh;
    ubase = lo;
    ushift = sh;
    unb = (int64_t)((hi - lo) >> sh) + 1;
    if (unb * 96 > (32ll << 20)) unb = 0;      // as the rows: only while it stays L2-resident
  }
  size_t off[11], total = 0;
  for (int k = 0; k < 4; ++k) {
    off[k] = total;
    total += align256((size_t)len[k] * 8);
  }
  for (int t = 0; t < 2; ++t) {
    off[4 + t] = total;
    total += align256(((size_t)nbk[t] + 1) * 4 + 4);
  }
  for (int t = 0; t < 2; ++t) {
    off[6 + t] = total;
    total += align256(((size_t)len[2 * t] + 1) * 16);
  }
  // rows only while they stay comfortably L2-resident (the scatter sweep: 2^20-key tables
  // give 100+ MB of rows per table, and the rows then lose to the 4 B bucket index)
  constexpr int64_t kRowsMaxBytes = 32ll << 20;
  int64_t nrow_alloc[2] = {0, 0};
  for (int t = 0; t < 2; ++t) {
    nrow_alloc[t] = (int64_t)nbk[t] * 48 <= kRowsMaxBytes ? nbk[t] : 0;
    off[8 + t] = total;
    total += align256((size_t)nrow_alloc[t] * 48);
  }
  off[10] = total;
  total += align256((size_t)unb * 96);
  NT_CUDA(c, c->xs.ensure(total));
  for (int k = 0; k < 4; ++k)
    NT_CUDA(c, cudaMemcpyAsync(c->xs.as<char>() + off[k], h[k], (size_t)len[k] * 8,
                               cudaMemcpyDefault, c->stream));
  unsigned int* wide = reinterpret_cast<unsigned int*>(c->scratch.as<char>() + 128);  // [2]
  NT_CUDA(c, cudaMemsetAsync(wide, 0, 8, c->stream));
  for (int t = 0; t < 2; ++t)
    launch_xs_prepare(reinterpret_cast<const double*>(c->xs.as<char>() + off[2 * t]),
                      reinterpret_cast<const double*>(c->xs.as<char>() + off[2 * t + 1]),
                      len[2 * t], base[t], shift[t], nbk[t], nrow_alloc[t] > 0,
                      reinterpret_cast<uint32_t*>(c->xs.as<char>() + off[4 + t]),
                      reinterpret_cast<double2*>(c->xs.as<char>() + off[6 + t]),
                      reinterpret_cast<double2*>(c->xs.as<char>() + off[8 + t]), wide + t, c->stream);
  NT_CUDA(c, cudaMemsetAsync(wide + 2, 0, 4, c->stream));
  launch_xs_urows(reinterpret_cast<const double*>(c->xs.as<char>() + off[0]),
                  reinterpret_cast<const double2*>(c->xs.as<char>() + off[6]), len[0],
                  reinterpret_cast<const double*>(c->xs.as<char>() + off[2]),
                  reinterpret_cast<const double2*>(c->xs.as<char>() + off[7]), len[2],
                  ubase, ushift, unb, reinterpret_cast<double2*>(c->xs.as<char>() + off[10]),
                  wide + 2, c->stream);
  unsigned int hw[3] = {1, 1, 1};
  NT_CUDA(c, cudaMemcpyAsync(hw, wide, 12, cudaMemcpyDeviceToHost, c->stream));
  // direct bucket rows only where every bucket spans at most one key (then the bin is
  // idx[b] or idx[b] + 1)
  int64_t nrows[2] = {0, 0};
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  for (int t = 0; t < 2; ++t) nrows[t] = (nrow_alloc[t] > 0 && hw[t] == 0) ? nbk[t] : 0;
  c->xs_urow = (unb > 0 && hw[2] == 0) ? reinterpret_cast<const double2*>(c->xs.as<char>() + off[10]) : nullptr;
  c->tables.urow = nullptr;                 // selected per launch (xs_tables)
  c->tables.ubase = ubase;
  c->tables.ushift = ushift;
  c->tables.unb = (int32_t)unb;
  c->tables.ulast = h[0][len[0] - 1] < h[2][len[2] - 1] ? h[0][len[0] - 1] : h[2][len[2] - 1];
  c->xs_bytes = total;
  c->xs_persist_bytes = 0;
  if (c->opt.xs_l2_persist) {
    int maxp = 0;
    cudaDeviceGetAttribute(&maxp, cudaDevAttrMaxPersistingL2CacheSize, c->device);
    const size_t want = total < (size_t)maxp ? total : (size_t)maxp;
    if (want > 0 && cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, want) == cudaSuccess) {
      size_t got = 0;
      cudaDeviceGetLimit(&got, cudaLimitPersistingL2CacheSize);
      c->xs_persist_bytes = got;
    } else {
      cudaGetLastError();
    }
  }
  Table* T[2] = {&c->tables.s, &c->tables.c};
  for (int t = 0; t < 2; ++t) {
    T[t]->k = reinterpret_cast<const double*>(c->xs.as<char>() + off[2 * t]);
    T[t]->v = reinterpret_cast<const double*>(c->xs.as<char>() + off[2 * t + 1]);
    T[t]->idx = reinterpret_cast<const uint32_t*>(c->xs.as<char>() + off[4 + t]);
    T[t]->kv = reinterpret_cast<const double2*>(c->xs.as<char>() + off[6 + t]);
    T[t]->row = nullptr;                 // selected per launch (xs_tables)
    c->xs_row[t] = nrows[t] == 0 ? nullptr
                                   : reinterpret_cast<const double2*>(c->xs.as<char>() + off[8 + t]);
    T[t]->n = (int32_t)len[2 * t];
    T[t]->nb = nbk[t];
    T[t]->shift = shift[t];
    T[t]->base = base[t];
    T[t]->kfirst = h[2 * t][0];
    T[t]->klast = h[2 * t][(size_t)len[2 * t] - 1];
  }
  c->stage = ST_XS;
  return NT_OK;
}

// ---- particles ------------------------------------------------------------
static cudaError_t alloc_soa(nt_ctx* c, int64_t n) {
  const size_t N = (size_t)(n > 0 ? n : 1);
  const size_t b8 = align256(N * 8), b4 = align256(N * 4), b1 = align256(N);
  // 8 + 3 f64 columns, gid, 6 + 3 u32 columns, parking / arrival / emigrant / free queues, status
  cudaError_t e = c->soa.ensure(12 * b8 + 13 * b4 + b1);
  if (e != cudaSuccess) return e;
  char* q = c->soa.as<char>();
  double** d8[11] = {&c->p.x, &c->p.y, &c->p.ox, &c->p.oy, &c->p.e, &c->p.w, &c->p.mfp, &c->p.dep,
                     &c->p.dcen, &c->p.acc, &c->p.dstep};
  for (auto d : d8) { *d = reinterpret_cast<double*>(q); q += b8; }
  uint32_t** d4[7] = {&c->p.ctr, &c->p.nfac, &c->p.ncol, &c->p.ncen, &c->p.nf_s, &c->p.nc_s, &c->p.seq_s};
  c->p.cx = reinterpret_cast<int32_t*>(q); q += b4;
  c->p.cy = reinterpret_cast<int32_t*>(q); q += b4;
  for (auto d : d4) { *d = reinterpret_cast<uint32_t*>(q); q += b4; }
  c->defer_q = reinterpret_cast<int32_t*>(q); q += b4;
  c->arr_q = reinterpret_cast<int32_t*>(q); q += b4;
  c->out_q = reinterpret_cast<int32_t*>(q); q += b4;
  c->free_q = reinterpret_cast<int32_t*>(q); q += b4;
  c->p.gid = reinterpret_cast<int64_t*>(q); q += b8;
  c->p.status = reinterpret_cast<uint8_t*>(q);
  // resume_prefetch: one record per particle at most (a particle is parked once per step),
  // plus a batch of slack so the last batch's copies stay inside the buffer
  if (c->opt.resume_prefetch && c->opt.mode != NT_MODE_EVENT && !c->opt.deterministic) {
    const int64_t cap = ((int64_t)N + kRingB + 3) / 4 * 4;
    e = c->park_rec.ensure((size_t)cap * (kParkF64 * 8 + kParkU32 * 4));
    if (e != cudaSuccess) return e;
    c->park_cap = cap;
  }
  return cudaSuccess;
}

nt_status nt_inject_particles(nt_ctx* c, int64_t n_total, int64_t first_id, int64_t n_local,
                              double sx, double sy, double sw, double sh, double e0,
                              uint64_t seed) {
  NvtxRange nvtx_("nt_inject_particles");
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->stage < ST_XS) return fail(c, NT_ERR_STATE, "mesh and cross sections must be loaded first");
  if (n_total < 0 || first_id < 0 || n_local < 0 || first_id + n_local > n_total)
    return fail(c, NT_ERR_ARG, "need 0 <= first_id, n_local and first_id + n_local <= n_total");
  if (!(sw >= 0.0) || !(sh >= 0.0) || !(sx >= 0.0) || !(sy >= 0.0) || !(sx + sw <= c->W) ||
      !(sy + sh <= c->H))
    return fail(c, NT_ERR_ARG, "source rectangle must lie inside the mesh");
  if (!(e0 > 0.0) || !is_fin(e0)) return fail(c, NT_ERR_ARG, "initial_energy must be finite and > 0");
  const bool slab = c->opt.decomposition == 1;
  if (slab && c->opt.deterministic)
    return fail(c, NT_ERR_UNSUPPORTED, "x-slab decomposition supports the production tally only");
  if (slab && c->opt.mode != NT_MODE_HISTORY)
    return fail(c, NT_ERR_UNSUPPORTED, "x-slab decomposition supports history mode only");
  c->n_cap = slab ? (n_total > n_local ? n_total : n_local) : n_local;
  c->n_free = 0;
  c->n_arr = 0;
  c->stage = ST_XS;             // the particle store is replaced: no step until it is rebuilt
  NT_CUDA(c, alloc_soa(c, c->n_cap));
  if (slab) {
    const int64_t P = c->opt.nranks, r = c->opt.rank;
    c->slab_lo = (int32_t)((r * c->nx) / P);
    c->slab_hi = (int32_t)(((r + 1) * c->nx) / P);
  }
  InjectParams ip{};
  ip.p = c->p;
  ip.ex = c->ex.as<double>();
  ip.ey = c->ey.as<double>();
  ip.nx = c->nx;
  ip.ny = c->ny;
  ip.W = c->W;
  ip.H = c->H;
  ip.n_local = n_local;
  ip.first_id = first_id;
  ip.sx = sx;
  ip.sy = sy;
  ip.sw = sw;
  ip.sh = sh;
  ip.e0 = e0;
  ip.seed = seed;
  launch_inject(ip, c->stream);
  NT_CUDA(c, cudaGetLastError());
  c->n_total = n_total;
  c->first_id = first_id;
  c->n_local = n_local;
  c->seed = seed;
  c->stage = ST_PARTICLES;
  return NT_OK;
}

// ---- timestep ---------------------------------------------------------------------------
static TrackParams make_params(nt_ctx* c, double dt) {
  TrackParams tp{};
  tp.mesh.rho = (c->tiled && c->dens_fmt == kDensF64) ? c->rho_st.as<double>() : c->rho.as<double>();
  tp.mesh.tiled = c->tiled;
  tp.mesh.ntx = c->ntx;
  tp.mesh.strip = 16 * c->ntx;
  tp.mesh.rho8 = c->rho_code.as<uint8_t>();
  tp.mesh.rho16 = c->rho_code.as<uint16_t>();
  tp.mesh.nd_tab = c->nd_tab.as<double>();
  tp.mesh.fmt = c->dens_fmt;
  tp.mesh.ncodes = c->dens_codes;
  tp.mesh.blk = c->blk_n > 0 ? c->blk.as<uint8_t>() : nullptr;
  tp.mesh.bshift = c->blk_shift;
  tp.mesh.nbx = c->blk_nbx;
  tp.mesh.nblk = c->blk_n;
  tp.mesh.tally = c->tally.as<double>();
  tp.mesh.ex = c->ex.as<double>();
  tp.mesh.ey = c->ey.as<double>();
  tp.mesh.nx = c->nxs;
  tp.mesh.gnx = c->nx;
  tp.mesh.x0 = c->x0;
  tp.mesh.wx = c->W;
  tp.mesh.wy = c->H;
  tp.mesh.ny = c->ny;
  tp.xs = xs_tables(c);
  tp.ph = c->ph;
  tp.p = c->p;
  tp.n = c->n_local;
  tp.lo = 0;
  tp.hi = c->n_local;
  tp.first_id = c->first_id;
  tp.seed = c->seed;
  tp.dt = dt;
  tp.max_events = c->opt.max_events_per_history;
  if (c->opt.tally_mode == 3) {       // the hot window, clipped to the mesh
    tp.hot_x0 = c->opt.hot_x0 < c->nx ? c->opt.hot_x0 : c->nx - 1;
    tp.hot_y0 = c->opt.hot_y0 < c->ny ? c->opt.hot_y0 : c->ny - 1;
    tp.hot_nx = c->opt.hot_nx < c->nx - tp.hot_x0 ? c->opt.hot_nx : c->nx - tp.hot_x0;
    tp.hot_ny = c->opt.hot_ny < c->ny - tp.hot_y0 ? c->opt.hot_ny : c->ny - tp.hot_y0;
  }
  tp.refill_min = c->opt.refill_min > 0 ? c->opt.refill_min : 4;

  char* s = c->scratch.as<char>();
  tp.counter = reinterpret_cast<unsigned long long*>(s);
  tp.stats_u = reinterpret_cast<unsigned long long*>(s + 256);
  tp.stats_f = reinterpret_cast<double*>(s + 512);
  tp.slot_f = c->slots.as<double>();
  return tp;
}

// Persistent grid of the history kernel: SMs x resident CTAs (ctas_per_sm caps it).
static int history_grid(nt_ctx* c, bool det) {
  int per_sm = history_max_ctas_per_sm(det, c->dens_fmt, c->tiled != 0, c->blk_n > 0,
                                       c->opt.ctas_per_sm, c->opt.tally_mode);
  if (per_sm < 1) per_sm = 1;
  if (c->opt.ctas_per_sm > 0 && c->opt.ctas_per_sm < per_sm) per_sm = c->opt.ctas_per_sm;
  return c->sm_count * per_sm;
}

// Deterministic mode: batches of <= 65536 particles, records sorted by (cell, particle,
// sequence) and applied serially per cell, batch after batch -> the oracle's sum order.
// A batch whose records overflow the buffer is restored (particles and statistics) and
// re-run with a larger buffer or, at the buffer limit, half the particles.
static nt_status det_snapshot(nt_ctx* c, int64_t lo, int64_t nb, bool restore) {
  char* b = c->backup.as<char>();
  auto mv = [&](void* col, size_t sz) -> cudaError_t {
    char* d = static_cast<char*>(col) + (size_t)lo * sz;
    cudaError_t e = restore ? cudaMemcpyAsync(d, b, (size_t)nb * sz, cudaMemcpyDeviceToDevice, c->stream)
                            : cudaMemcpyAsync(b, d, (size_t)nb * sz, cudaMemcpyDeviceToDevice, c->stream);
    b += align256((size_t)nb * sz);
    return e;
  };
  void* d8[8] = {c->p.x, c->p.y, c->p.ox, c->p.oy, c->p.e, c->p.w, c->p.mfp, c->p.dep};
  for (void* d : d8) NT_CUDA(c, mv(d, 8));
  void* d4[6] = {c->p.cx, c->p.cy, c->p.ctr, c->p.nfac, c->p.ncol, c->p.ncen};
  for (void* d : d4) NT_CUDA(c, mv(d, 4));
  NT_CUDA(c, mv(c->p.status, 1));
  // step statistics accumulated so far (scratch bytes [256, 1024))
  char* s = c->scratch.as<char>() + 256;
  NT_CUDA(c, restore ? cudaMemcpyAsync(s, b, 768, cudaMemcpyDeviceToDevice, c->stream)
                     : cudaMemcpyAsync(b, s, 768, cudaMemcpyDeviceToDevice, c->stream));
  return NT_OK;
}

// History kernel with regime parking: phase 1 tracks [lo, hi) -- or, with src_count, the
// parked particles queued in c->arr_q (slab arrivals) -- and parks lonely collisions;
// phase 2 resumes them.  (Measured alternative: 4 phases, even ones parking lonely facets
// -- split 132 -> 130 ms but csp 31 -> 35 ms, each phase adding its own tail of long
// streaming histories.)  With slabs, both phases hand emigrants to out_q.
// (Measured and rejected in round 2: a third phase for the streamers phase 2 finds --
// particles scattered back out of dense matter -- csp 27.1 -> 27.8-29.6 ms: too few of them
// to fill the GPU, so the third launch is one long latency-bound tail; profiles/ab.)
// scratch [0, 8): phase-1 counter, [16, 24): parking queue length, [32, 40): phase-2
// counter, [40, 48): emigrant count, [64, 72): arrivals count, [88, 96): fused-phase queue
// positions claimed, [96, 100): fused-phase producer warps done.
static nt_status track_phases(nt_ctx* c, const TrackParams& bp_in, bool det, uint32_t& launches,
                              const unsigned long long* src_count, bool slab) {
  NvtxRange nvtx_("history phases");
  char* s = c->scratch.as<char>();
  TrackParams bp = bp_in;
  // particle_layout 1 (AoS ablation): the kernels work on 128 B records, copied from and back
  // to the structure-of-arrays store around the phases (production, default kernel only)
  const bool aos = c->opt.particle_layout == 1 && !det && !slab;
  if (aos) {
    NT_CUDA(c, c->aos.ensure((size_t)(c->n_local > 0 ? c->n_local : 1) * sizeof(ParticleAoS)));
    bp.aos = c->aos.as<ParticleAoS>();
    launch_aos_copy(c->p, bp.aos, c->n_local, true, c->stream);
    ++launches;
  }
  unsigned long long* qlen = reinterpret_cast<unsigned long long*>(s + 16);
  NT_CUDA(c, cudaMemsetAsync(s + 16, 0, 24, c->stream));
  const int grid = history_grid(c, det);
  // fused phases: one launch, consumers resume parked particles during phase 1 (the
  // conditions mirror the kernel selection in nt_kernels.cu history_fn)
  const bool var = c->ph.vacuum || c->ph.analog || c->ph.roulette;
  const bool fused = c->opt.fused_consumers > 0 && !det && !slab && !src_count && !var && !aos &&
                     c->dens_fmt == kDensU8 && c->blk_n > 0 && c->opt.tally_mode == 0 &&
                     c->opt.xs_search != 2 && c->opt.ctas_per_sm < 7;
  if (fused) {
    NvtxRange nvtx2_("fused phases");
    NT_CUDA(c, cudaMemsetAsync(c->defer_q, 0, (size_t)(c->n_local > 0 ? c->n_local : 1) * 4, c->stream));
    NT_CUDA(c, cudaMemsetAsync(s + 88, 0, 16, c->stream));
    TrackParams p = bp;
    p.phase = 1;
    p.park_q = c->defer_q;
    p.park_count = qlen;
    p.park_coll_below = c->opt.defer_below;
    int coll = (c->opt.fused_consumers - 1) * c->sm_count;   // dedicated consumer CTAs
    if (coll >= grid) coll = grid - 1;
    p.coll_ctas = coll;
    p.n_prod = (uint32_t)(grid - coll) * (uint32_t)(kHistoryBlock / 32);
    p.park_taken = reinterpret_cast<unsigned long long*>(s + 88);
    p.prod_done = reinterpret_cast<unsigned int*>(s + 96);
    launch_history(p, det, grid, c->opt.ctas_per_sm, c->opt.tally_mode, c->opt.xs_search, slab,
                   c->stream);
    ++launches;
    NT_CUDA(c, cudaGetLastError());
    return NT_OK;
  }
  // resume_prefetch: record parking + the phase-2 ring, default kernel options only (the
  // conditions mirror the kernel selection in nt_kernels.cu history_fn)
  const bool ring = c->opt.resume_prefetch && c->park_cap > 0 && !det && !slab && !src_count &&
                    !var && !aos && c->dens_fmt == kDensU8 && c->blk_n > 0 &&
                    c->opt.tally_mode == 0 && c->opt.xs_search != 2 && c->opt.ctas_per_sm < 7;
  for (int ph = 1; ph <= 2; ++ph) {
    TrackParams p = bp;
    p.phase = ph;
    int g = grid;
    if (ring) {
      p.park_rec = c->park_rec.as<double>();
      p.park_cap = c->park_cap;
      if (ph == 2) {                 // the ring's shared memory may lower the residency
        const int per_sm = history_ring_ctas_per_sm(c->tiled != 0);
        if (per_sm > 0 && per_sm * c->sm_count < g) g = per_sm * c->sm_count;
      }
    }
    if (slab) {
      p.slab_lo = c->slab_lo;
      p.slab_hi = c->slab_hi;
      p.out_q = c->out_q;
      p.out_count = reinterpret_cast<unsigned long long*>(s + 40);
    }
    if (ph == 2) {
      p.resume_q = c->defer_q;
      p.resume_count = qlen;
      p.counter = reinterpret_cast<unsigned long long*>(s + 32);
    } else {
      if (src_count) {
        p.resume_q = c->arr_q;
        p.resume_count = src_count;
      }
      p.park_q = c->defer_q;
      p.park_count = qlen;
      p.park_coll_below = c->opt.defer_below;
    }
    launch_history(p, det, g, c->opt.ctas_per_sm, c->opt.tally_mode, c->opt.xs_search, slab,
                   c->stream);
    ++launches;
  }
  if (aos) {
    launch_aos_copy(c->p, bp.aos, c->n_local, false, c->stream);
    ++launches;
  }
  NT_CUDA(c, cudaGetLastError());
  return NT_OK;
}

// Track one batch [bp.lo, bp.hi) in the context's mode (history kernel or event loop).
static nt_status track_range(nt_ctx* c, const TrackParams& bp, bool det, uint32_t& launches) {
  if (c->opt.mode == NT_MODE_EVENT) {
    if (!c->evs) c->evs = event_state_create();
    if (!c->evs) return fail(c, NT_ERR_OOM, "event state");
    return event_run_range(c->evs, bp, det, c->sm_count, c->stream, launches, c->err);
  }
  return track_phases(c, bp, det, launches, nullptr, false);
}

static nt_status run_det(nt_ctx* c, const TrackParams& tp, uint32_t& launches) {
  int cell_bits = 0;
  while ((1ull << cell_bits) < (unsigned long long)c->cells_st) ++cell_bits;
  if (cell_bits > 24)
    return fail(c, NT_ERR_UNSUPPORTED, "deterministic mode supports at most 2^24 cells");
  if (c->rec_cap == 0) c->rec_cap = 1ull << 20;
  const unsigned long long kMaxCap = 1ull << 27;
  int64_t batch = c->opt.det_batch;
  unsigned long long* rec_count = reinterpret_cast<unsigned long long*>(c->scratch.as<char>() + 8);
  int64_t lo = 0;
  while (lo < c->n_local) {
    const int64_t hi = lo + batch < c->n_local ? lo + batch : c->n_local;
    const int64_t nb = hi - lo;
    NT_CUDA(c, c->rec_key.ensure(c->rec_cap * 8));
    NT_CUDA(c, c->rec_val.ensure(c->rec_cap * 8));
    NT_CUDA(c, c->rec_key2.ensure(c->rec_cap * 8));
    NT_CUDA(c, c->rec_val2.ensure(c->rec_cap * 8));
    NT_CUDA(c, c->backup.ensure(15 * align256((size_t)nb * 8) + 4096));
    nt_status st = det_snapshot(c, lo, nb, false);
    if (st != NT_OK) return st;
    TrackParams bp = tp;
    bp.lo = lo;
    bp.hi = hi;
    bp.rec_key = c->rec_key.as<unsigned long long>();
    bp.rec_val = c->rec_val.as<double>();
    bp.rec_cap = c->rec_cap;
    bp.rec_count = rec_count;
    NT_CUDA(c, cudaMemsetAsync(c->scratch.p, 0, 16, c->stream));   // work counter, records
    st = track_range(c, bp, true, launches);
    if (st != NT_OK) return st;
    unsigned long long nrec = 0;
    NT_CUDA(c, cudaMemcpyAsync(&nrec, rec_count, 8, cudaMemcpyDeviceToHost, c->stream));
    NT_CUDA(c, cudaStreamSynchronize(c->stream));
    if (nrec > c->rec_cap) {
      st = det_snapshot(c, lo, nb, true);
      if (st != NT_OK) return st;
      if (c->rec_cap < kMaxCap) {
        while (c->rec_cap < nrec && c->rec_cap < kMaxCap) c->rec_cap <<= 1;
      } else if (batch > 1) {
        batch /= 2;
      } else {
        return fail(c, NT_ERR_UNSUPPORTED, "deterministic record buffer overflow");
      }
      continue;
    }
    if (nrec > 0) {
      size_t tmp = 0;
      NT_CUDA(c, sort_pairs(nullptr, tmp, bp.rec_key, c->rec_key2.as<unsigned long long>(),
                            bp.rec_val, c->rec_val2.as<double>(), nrec, 40 + cell_bits, c->stream));
      NT_CUDA(c, c->sort_tmp.ensure(tmp));
      NT_CUDA(c, sort_pairs(c->sort_tmp.p, tmp, bp.rec_key, c->rec_key2.as<unsigned long long>(),
                            bp.rec_val, c->rec_val2.as<double>(), nrec, 40 + cell_bits, c->stream));
      launch_det_apply(c->rec_key2.as<unsigned long long>(), c->rec_val2.as<double>(), nrec,
                       tp.mesh.tally, c->stream);
      launches += 2;
      NT_CUDA(c, cudaGetLastError());
    }
    lo = hi;
  }
  return NT_OK;
}

// ---- x-slab decomposition ---------------------------------------------
// One round: the first round tracks this rank's own particles [0, n_local) (status 1), later
// rounds the arrivals queued by nt_slab_import; emigrants are left in out_q.
static nt_status slab_round(nt_ctx* c, const TrackParams& tp, uint32_t& launches, int64_t* n_out) {
  char* s = c->scratch.as<char>();
  unsigned long long* out_count = reinterpret_cast<unsigned long long*>(s + 40);
  unsigned long long* arr_count = reinterpret_cast<unsigned long long*>(s + 64);
  NT_CUDA(c, cudaMemsetAsync(s, 0, 8, c->stream));                // phase-1 work counter
  NT_CUDA(c, cudaMemsetAsync(out_count, 0, 8, c->stream));
  TrackParams bp = tp;
  bp.hi = c->n_local;
  nt_status st = NT_OK;
  if (c->slab_round == 0) {
    st = track_phases(c, bp, false, launches, nullptr, true);
  } else if (c->n_arr > 0) {
    const unsigned long long na = (unsigned long long)c->n_arr;
    NT_CUDA(c, cudaMemcpyAsync(arr_count, &na, 8, cudaMemcpyHostToDevice, c->stream));
    st = track_phases(c, bp, false, launches, arr_count, true);
  }
  if (st != NT_OK) return st;
  unsigned long long no = 0;
  NT_CUDA(c, cudaMemcpyAsync(&no, out_count, 8, cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  c->n_arr = 0;
  ++c->slab_round;
  *n_out = (int64_t)no;
  return NT_OK;
}

// Pack the round's emigrants into c->slab_buf (left-going first); counts in *nl, *nr.
static nt_status slab_pack(nt_ctx* c, const TrackParams& tp, int64_t n_out, int64_t* nl,
                           int64_t* nr) {
  char* s = c->scratch.as<char>();
  unsigned long long* cnt = reinterpret_cast<unsigned long long*>(s + 48);
  NT_CUDA(c, c->slab_buf.ensure((size_t)(n_out > 0 ? n_out : 1) * sizeof(SlabRec)));
  NT_CUDA(c, cudaMemsetAsync(cnt, 0, 16, c->stream));
  TrackParams p = tp;
  p.slab_lo = c->slab_lo;
  p.slab_hi = c->slab_hi;
  launch_slab_pack(p, c->out_q, n_out, c->slab_buf.as<SlabRec>(), cnt, c->stream);
  NT_CUDA(c, cudaGetLastError());
  unsigned long long h[2] = {0, 0};
  NT_CUDA(c, cudaMemcpyAsync(h, cnt, 16, cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  *nl = (int64_t)h[0];
  *nr = (int64_t)h[1];
  return NT_OK;
}

// The emigrants' slots (out_q) become free for arrivals.
static cudaError_t slab_free_slots(nt_ctx* c, int64_t n_out) {
  if (n_out <= 0) return cudaSuccess;
  const cudaError_t e = cudaMemcpyAsync(c->free_q + c->n_free, c->out_q, (size_t)n_out * 4,
                                        cudaMemcpyDeviceToDevice, c->stream);
  c->n_free += n_out;
  return e;
}

// Store n records (device memory) as parked particles queued for the next round: first in
// free slots, then appended.
static nt_status slab_unpack(nt_ctx* c, const SlabRec* d, int64_t n) {
  if (n <= 0) return NT_OK;
  const int64_t m = n < c->n_free ? n : c->n_free;
  if (c->n_local + (n - m) > c->n_cap)
    return fail(c, NT_ERR_ARG, "slab import exceeds the particle store (%lld + %lld > %lld)",
                (long long)c->n_local, (long long)(n - m), (long long)c->n_cap);
  c->n_free -= m;
  launch_slab_unpack(c->p, d, n, c->free_q + c->n_free, m, c->n_local, c->arr_q + c->n_arr,
                     c->stream);
  NT_CUDA(c, cudaGetLastError());
  c->n_local += n - m;
  c->n_arr += n;
  return NT_OK;
}

// nt_run_timestep with slabs: rounds until no rank has emigrants; with a communicator the
// emigrants go to the neighbouring ranks over NCCL (counts, then records), and an allreduce
// of the emigrant count ends the loop.
static nt_status run_slab_nccl(nt_ctx* c, const TrackParams& tp, uint32_t& launches) {
  c->slab_round = 0;
  c->n_arr = 0;
  const int P = c->opt.nranks, r = c->opt.rank;
  for (int round = 0;; ++round) {
    if (round > 4 * (c->nx + c->ny) + 16)
      return fail(c, NT_ERR_STATE, "slab exchange did not terminate");
    int64_t n_out = 0;
    nt_status st = slab_round(c, tp, launches, &n_out);
    if (st != NT_OK) return st;
    if (!c->comm) {
      if (n_out != 0) return fail(c, NT_ERR_STATE, "emigrants without a communicator");
      return NT_OK;
    }
    int64_t nl = 0, nr = 0;
    st = slab_pack(c, tp, n_out, &nl, &nr);
    if (st != NT_OK) return st;
    NT_CUDA(c, slab_free_slots(c, n_out));
    // counts to / from the neighbours, then the records
    char* s = c->scratch.as<char>();
    long long* dc = reinterpret_cast<long long*>(s + 128);   // [send l, send r, recv l, recv r, tot]
    const long long hsend[3] = {(long long)nl, (long long)nr, (long long)n_out};
    NT_CUDA(c, cudaMemcpyAsync(dc, hsend, 16, cudaMemcpyHostToDevice, c->stream));
    NT_CUDA(c, cudaMemcpyAsync(dc + 4, hsend + 2, 8, cudaMemcpyHostToDevice, c->stream));
    NT_CUDA(c, cudaMemsetAsync(dc + 2, 0, 16, c->stream));
    NT_NCCL(c, ncclGroupStart());
    if (r > 0) {
      NT_NCCL(c, ncclSend(dc + 0, 1, ncclInt64, r - 1, c->comm, c->stream));
      NT_NCCL(c, ncclRecv(dc + 2, 1, ncclInt64, r - 1, c->comm, c->stream));
    }
    if (r + 1 < P) {
      NT_NCCL(c, ncclSend(dc + 1, 1, ncclInt64, r + 1, c->comm, c->stream));
      NT_NCCL(c, ncclRecv(dc + 3, 1, ncclInt64, r + 1, c->comm, c->stream));
    }
    NT_NCCL(c, ncclGroupEnd());
    NT_NCCL(c, ncclAllReduce(dc + 4, dc + 4, 1, ncclInt64, ncclSum, c->comm, c->stream));
    long long hrecv[3] = {0, 0, 0};
    NT_CUDA(c, cudaMemcpyAsync(hrecv, dc + 2, 24, cudaMemcpyDeviceToHost, c->stream));
    NT_CUDA(c, cudaStreamSynchronize(c->stream));
    if (hrecv[2] == 0) return NT_OK;                       // nobody moves: step done
    const int64_t nin = hrecv[0] + hrecv[1];
    const size_t rb = sizeof(SlabRec);
    NT_CUDA(c, c->slab_rbuf.ensure((size_t)(nin > 0 ? nin : 1) * rb));
    char* sb = c->slab_buf.as<char>();
    char* rbuf = c->slab_rbuf.as<char>();
    NT_NCCL(c, ncclGroupStart());
    if (r > 0) {
      if (nl) NT_NCCL(c, ncclSend(sb, (size_t)nl * rb, ncclUint8, r - 1, c->comm, c->stream));
      if (hrecv[0]) NT_NCCL(c, ncclRecv(rbuf, (size_t)hrecv[0] * rb, ncclUint8, r - 1, c->comm, c->stream));
    }
    if (r + 1 < P) {
      if (nr) NT_NCCL(c, ncclSend(sb + (size_t)(n_out - nr) * rb, (size_t)nr * rb, ncclUint8, r + 1,
                                  c->comm, c->stream));
      if (hrecv[1]) NT_NCCL(c, ncclRecv(rbuf + (size_t)hrecv[0] * rb, (size_t)hrecv[1] * rb, ncclUint8,
                                        r + 1, c->comm, c->stream));
    }
    NT_NCCL(c, ncclGroupEnd());
    st = slab_unpack(c, c->slab_rbuf.as<SlabRec>(), nin);
    if (st != NT_OK) return st;
  }
}

// Step statistics from the reduced counters; the return status reports device anomalies.
static nt_status finish_stats(nt_ctx* c, const double* hs, float track_ms, float reduce_ms,
                              float step_ms, uint32_t launches, nt_step_stats* stats) {
  nt_step_stats s{};
  s.n_alive_start = (uint64_t)hs[SU_ALIVE];
  s.n_facets = (uint64_t)hs[SU_FACETS];
  s.n_collisions = (uint64_t)hs[SU_COLLISIONS];
  s.n_census = (uint64_t)hs[SU_CENSUS];
  s.n_killed = (uint64_t)hs[SU_KILLED];
  s.n_xs_range = (uint64_t)hs[SU_XS_RANGE];
  s.n_nonfinite = (uint64_t)hs[SU_NONFINITE];
  s.n_event_cap = (uint64_t)hs[SU_EVENT_CAP];
  s.tally_total = hs[SU_COUNT + SF_TALLY];
  s.census_energy = hs[SU_COUNT + SF_CENSUS_E];
  s.census_weight = hs[SU_COUNT + SF_CENSUS_W];
  s.killed_energy = hs[SU_COUNT + SF_KILLED_E];
  s.killed_weight = hs[SU_COUNT + SF_KILLED_W];
  s.absorbed_weight = hs[SU_COUNT + SF_ABSORBED_W];
  s.n_escaped = (uint64_t)hs[SU_ESCAPED];
  s.n_absorbed = (uint64_t)hs[SU_ABSORBED];
  s.escaped_energy = hs[SU_COUNT + SF_ESCAPED_E];
  s.escaped_weight = hs[SU_COUNT + SF_ESCAPED_W];
  s.absorbed_energy = hs[SU_COUNT + SF_ABSORBED_E];
  s.roulette_gain = hs[SU_COUNT + SF_ROULETTE];
  s.track_ms = track_ms;
  s.reduce_ms = reduce_ms;
  s.step_ms = step_ms + reduce_ms;
  s.n_launches = launches;
  if (stats) *stats = s;
  c->stage = ST_STEPPED;
  if (hs[SU_REC_OVERFLOW] > 0) return fail(c, NT_ERR_UNSUPPORTED, "flush sequence overflow (>2^24 flushes in one history)");
  if (s.n_nonfinite) return fail(c, NT_ERR_NONFINITE, "%llu particles ended non-finite", (unsigned long long)s.n_nonfinite);
  if (s.n_event_cap) return fail(c, NT_ERR_EVENT_CAP, "%llu histories hit max_events_per_history", (unsigned long long)s.n_event_cap);
  if (s.n_xs_range) return fail(c, NT_ERR_XS_RANGE, "%llu lookups outside the table range", (unsigned long long)s.n_xs_range);
  return NT_OK;
}

static nt_status step_prologue(nt_ctx* c, double dt) {
  if (c->stage < ST_PARTICLES) return fail(c, NT_ERR_STATE, "nt_inject_particles must come first");
  if (!(dt > 0.0) || !is_fin(dt)) return fail(c, NT_ERR_ARG, "dt must be finite and > 0");
  NT_CUDA(c, c->scratch.ensure(1024));
  // per-thread statistic slots for the largest persistent grid (16 CTAs per SM)
  NT_CUDA(c, c->slots.ensure((size_t)c->sm_count * 16 * kHistoryBlock * SF_COUNT * 8));
  NT_CUDA(c, cudaEventRecord(c->ev[0], c->stream));
  NT_CUDA(c, cudaMemsetAsync(c->tally.p, 0, (size_t)c->cells_st * 8, c->stream));
  NT_CUDA(c, cudaMemsetAsync(c->scratch.p, 0, 1024, c->stream));
  NT_CUDA(c, cudaEventRecord(c->ev[1], c->stream));
  return NT_OK;
}

nt_status nt_run_timestep(nt_ctx* c, double dt, nt_step_stats* stats) {
  NvtxRange nvtx_("nt_run_timestep");
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  {
    const nt_status st = step_prologue(c, dt);
    if (st != NT_OK) return st;
  }
  const size_t cells = (size_t)c->cells_st;   // storage layout (tiles padded with zeros)
  uint32_t launches = 0;
  const bool det = c->opt.deterministic != 0;
  const TrackParams tp = make_params(c, dt);
  {
    XsWindow xw(c);
    const nt_status st = c->opt.decomposition == 1 ? run_slab_nccl(c, tp, launches)
                         : det ? run_det(c, tp, launches) : track_range(c, tp, false, launches);
    if (st != NT_OK) return st;
  }
  NT_CUDA(c, cudaEventRecord(c->ev[2], c->stream));
  // statistics -> one f64 vector on the device (u64 counts < 2^53 convert exactly); with a
  // communicator the tally (out of place: the local partial stays in c->tally) and the
  // statistics are summed over ranks in one NCCL group; one D2H copy, one synchronisation.
  // Nothing here allocates (stats_d, stats_h and tally_red exist since nt_create /
  // nt_init_mesh).
  double* sd = c->stats_d.as<double>();
  {
    char* s = c->scratch.as<char>();
    launch_stats_to_f64(reinterpret_cast<const unsigned long long*>(s + 256),
                        reinterpret_cast<const double*>(s + 512), sd, c->stream);
    ++launches;
    NT_CUDA(c, cudaGetLastError());
  }
  if (c->comm) {
    NvtxRange nvtx_("tally + stats allreduce");
    // (x-slabs own disjoint columns: their tallies are assembled at read time, nt_read_tally)
    NT_CUDA(c, cudaEventRecord(c->ev[3], c->stream));
    NT_NCCL(c, ncclGroupStart());
    if (c->opt.decomposition != 1)
      NT_NCCL(c, ncclAllReduce(c->tally.p, c->tally_red.p, cells, ncclFloat64, ncclSum, c->comm, c->stream));
    NT_NCCL(c, ncclAllReduce(sd, sd, SU_COUNT + SF_COUNT, ncclFloat64, ncclSum, c->comm, c->stream));
    NT_NCCL(c, ncclGroupEnd());
    NT_CUDA(c, cudaEventRecord(c->ev[4], c->stream));
  }
  NT_CUDA(c, cudaMemcpyAsync(c->stats_h, sd, (SU_COUNT + SF_COUNT) * sizeof(double),
                             cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  double hs[SU_COUNT + SF_COUNT];
  std::memcpy(hs, c->stats_h, sizeof hs);
  float reduce_ms = 0.f;
  if (c->comm) {
    cudaEventElapsedTime(&reduce_ms, c->ev[3], c->ev[4]);
    ncclResult_t async_err;
    ncclCommGetAsyncError(c->comm, &async_err);
    if (async_err != ncclSuccess) return fail(c, NT_ERR_NCCL, "NCCL async error: %s", ncclGetErrorString(async_err));
  }
  float track_ms = 0.f, step_ms = 0.f;
  cudaEventElapsedTime(&track_ms, c->ev[1], c->ev[2]);
  cudaEventElapsedTime(&step_ms, c->ev[0], c->ev[2]);
  return finish_stats(c, hs, track_ms, reduce_ms, step_ms, launches, stats);
}

// ---- x-slab decomposition driven by the caller ---------------------------------------------
int64_t nt_slab_record_bytes(void) { return (int64_t)sizeof(SlabRec); }

static nt_status slab_check(nt_ctx* c) {
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->opt.decomposition != 1) return fail(c, NT_ERR_STATE, "the context was not created with decomposition = 1");
  return NT_OK;
}

nt_status nt_slab_begin(nt_ctx* c, double dt) {
  nt_status st = slab_check(c);
  if (st != NT_OK) return st;
  st = step_prologue(c, dt);
  if (st != NT_OK) return st;
  c->slab_dt = dt;
  c->slab_round = 0;
  c->n_arr = 0;
  c->slab_launches = 0;
  return NT_OK;
}

nt_status nt_slab_round(nt_ctx* c, int64_t* n_emigrants) {
  NvtxRange nvtx_("nt_slab_round");
  nt_status st = slab_check(c);
  if (st != NT_OK) return st;
  if (!n_emigrants) return fail(c, NT_ERR_ARG, "n_emigrants is NULL");
  if (!(c->slab_dt > 0.0)) return fail(c, NT_ERR_STATE, "nt_slab_begin must come first");
  const TrackParams tp = make_params(c, c->slab_dt);
  return slab_round(c, tp, c->slab_launches, n_emigrants);
}

nt_status nt_slab_export(nt_ctx* c, void* dst, int64_t capacity, int64_t* n_left, int64_t* n_right) {
  NvtxRange nvtx_("nt_slab_export");
  nt_status st = slab_check(c);
  if (st != NT_OK) return st;
  if (!dst || !n_left || !n_right) return fail(c, NT_ERR_ARG, "NULL argument");
  unsigned long long n_out = 0;
  NT_CUDA(c, cudaMemcpy(&n_out, c->scratch.as<char>() + 40, 8, cudaMemcpyDeviceToHost));
  if ((int64_t)n_out > capacity) return fail(c, NT_ERR_ARG, "capacity %lld < %llu emigrants", (long long)capacity, n_out);
  const TrackParams tp = make_params(c, c->slab_dt);
  st = slab_pack(c, tp, (int64_t)n_out, n_left, n_right);
  if (st != NT_OK) return st;
  NT_CUDA(c, cudaMemcpyAsync(dst, c->slab_buf.p, (size_t)n_out * sizeof(SlabRec), cudaMemcpyDefault, c->stream));
  NT_CUDA(c, slab_free_slots(c, (int64_t)n_out));
  NT_CUDA(c, cudaMemsetAsync(c->scratch.as<char>() + 40, 0, 8, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  return NT_OK;
}

nt_status nt_slab_import(nt_ctx* c, const void* src, int64_t n) {
  NvtxRange nvtx_("nt_slab_import");
  nt_status st = slab_check(c);
  if (st != NT_OK) return st;
  if (n < 0 || (n > 0 && !src)) return fail(c, NT_ERR_ARG, "bad import");
  if (n == 0) return NT_OK;
  NT_CUDA(c, c->slab_rbuf.ensure((size_t)n * sizeof(SlabRec)));
  NT_CUDA(c, cudaMemcpyAsync(c->slab_rbuf.p, src, (size_t)n * sizeof(SlabRec), cudaMemcpyDefault, c->stream));
  st = slab_unpack(c, c->slab_rbuf.as<SlabRec>(), n);
  if (st != NT_OK) return st;
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  return NT_OK;
}

nt_status nt_slab_end(nt_ctx* c, nt_step_stats* stats) {
  nt_status st = slab_check(c);
  if (st != NT_OK) return st;
  NT_CUDA(c, cudaEventRecord(c->ev[2], c->stream));
  unsigned long long hu[SU_COUNT];
  double hf[SF_COUNT], hs[SU_COUNT + SF_COUNT];
  char* s = c->scratch.as<char>();
  NT_CUDA(c, cudaMemcpyAsync(hu, s + 256, sizeof hu, cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaMemcpyAsync(hf, s + 512, sizeof hf, cudaMemcpyDeviceToHost, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  for (int k = 0; k < SU_COUNT; ++k) hs[k] = (double)hu[k];
  for (int k = 0; k < SF_COUNT; ++k) hs[SU_COUNT + k] = hf[k];
  float track_ms = 0.f, step_ms = 0.f;
  cudaEventElapsedTime(&track_ms, c->ev[1], c->ev[2]);
  cudaEventElapsedTime(&step_ms, c->ev[0], c->ev[2]);
  c->slab_dt = 0.0;
  return finish_stats(c, hs, track_ms, 0.f, step_ms, c->slab_launches, stats);
}

nt_status nt_particle_slots(nt_ctx* c, int64_t* n_slots) {
  if (!c || !n_slots) return NT_ERR_ARG;
  *n_slots = c->n_local;
  return NT_OK;
}

// ---- read-back ---------------------------------------------------------------------------
nt_status nt_read_tally(nt_ctx* c, double* dst, int32_t reduced) {
  NvtxRange nvtx_("nt_read_tally");
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->stage < ST_MESH) return fail(c, NT_ERR_STATE, "no mesh");
  if (!dst) return fail(c, NT_ERR_ARG, "dst is NULL");
  const bool slab = c->opt.decomposition == 1;
  const int64_t cells = (int64_t)c->nxs * (int64_t)c->ny;         // stored cells
  const double* src = (reduced && c->comm && !slab) ? c->tally_red.as<double>() : c->tally.as<double>();
  if (!src) return fail(c, NT_ERR_STATE, "no tally yet");
  if (c->tiled) {            // storage layout -> row-major [ny][nxs]
    NT_CUDA(c, c->tally_rm.ensure((size_t)cells * 8));
    Mesh ml{};
    ml.nx = c->nxs;
    ml.gnx = c->nxs;
    ml.ny = c->ny;
    ml.tiled = 1;
    ml.ntx = c->ntx;
    ml.strip = 16 * c->ntx;
    NT_CUDA(c, launch_relayout(src, c->tally_rm.as<double>(), cells, ml, false, c->stream));
    src = c->tally_rm.as<double>();
  }
  if (slab) {
    // the stored columns into a whole-mesh map (zero elsewhere); reduced with a
    // communicator: the sum over the ranks' disjoint slabs
    const int64_t all = (int64_t)c->nx * (int64_t)c->ny;
    NT_CUDA(c, c->tally_full.ensure((size_t)all * 8));
    double* full = c->tally_full.as<double>();
    NT_CUDA(c, cudaMemsetAsync(full, 0, (size_t)all * 8, c->stream));
    NT_CUDA(c, cudaMemcpy2DAsync(full + c->x0, (size_t)c->nx * 8, src, (size_t)c->nxs * 8,
                                 (size_t)c->nxs * 8, (size_t)c->ny, cudaMemcpyDeviceToDevice, c->stream));
    if (reduced && c->comm)
      NT_NCCL(c, ncclAllReduce(full, full, (size_t)all, ncclFloat64, ncclSum, c->comm, c->stream));
    NT_CUDA(c, cudaMemcpyAsync(dst, full, (size_t)all * 8, cudaMemcpyDefault, c->stream));
  } else {
    NT_CUDA(c, cudaMemcpyAsync(dst, src, (size_t)cells * 8, cudaMemcpyDefault, c->stream));
  }
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  return NT_OK;
}

static nt_status copy_particles(nt_ctx* c, int64_t first, int64_t count, const nt_particles* v,
                                bool to_dev) {
  if (!c) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->stage < ST_PARTICLES) return fail(c, NT_ERR_STATE, "no particles");
  if (!v || first < 0 || count < 0 || first + count > c->n_local)
    return fail(c, NT_ERR_ARG, "range [first, first+count) outside the local particles");
  struct F { void* host; void* dev; size_t sz; };
  const F f[] = {
      {v->x, c->p.x, 8}, {v->y, c->p.y, 8}, {v->ox, c->p.ox, 8}, {v->oy, c->p.oy, 8},
      {v->e, c->p.e, 8}, {v->w, c->p.w, 8}, {v->mfp, c->p.mfp, 8}, {v->cx, c->p.cx, 4},
      {v->cy, c->p.cy, 4}, {v->ctr, c->p.ctr, 4}, {v->status, c->p.status, 1},
      {v->nfac, c->p.nfac, 4}, {v->ncol, c->p.ncol, 4}, {v->ncen, c->p.ncen, 4},
      {v->dep, c->p.dep, 8}, {v->gid, c->p.gid, 8}};
  for (const F& x : f) {
    if (!x.host) continue;
    char* d = static_cast<char*>(x.dev) + (size_t)first * x.sz;
    if (to_dev)
      NT_CUDA(c, cudaMemcpyAsync(d, x.host, (size_t)count * x.sz, cudaMemcpyDefault, c->stream));
    else
      NT_CUDA(c, cudaMemcpyAsync(x.host, d, (size_t)count * x.sz, cudaMemcpyDefault, c->stream));
  }
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  return NT_OK;
}

nt_status nt_read_particles(nt_ctx* c, int64_t first, int64_t count, const nt_particles* dst) {
  return copy_particles(c, first, count, dst, false);
}

nt_status nt_write_particles(nt_ctx* c, int64_t first, int64_t count, const nt_particles* src) {
  return copy_particles(c, first, count, src, true);
}

// ---- verification entry points -----------------------------------------------------------
int64_t nt_debug_alloc_count(void) { return (int64_t)nt::g_device_allocs.load(); }

int64_t nt_debug_mesh_bytes(const nt_ctx* c) {
  if (!c) return -1;
  int64_t b = 0;
  for (const DevBuf* d : {&c->rho, &c->tally, &c->tally_red, &c->rho_code, &c->blk, &c->rho_st})
    b += (int64_t)d->bytes;
  return b;
}

int32_t nt_debug_density_format(const nt_ctx* c, int32_t* n_distinct) {
  if (!c || c->stage < ST_MESH) return -1;
  if (n_distinct) *n_distinct = c->dens_distinct;
  return c->dens_fmt;
}

int32_t nt_debug_xs_rows(const nt_ctx* c) {
  if (!c) return -1;
  return (c->xs_row[0] ? 1 : 0) | (c->xs_row[1] ? 2 : 0) | (c->xs_urow ? 4 : 0);
}

nt_status nt_debug_threefry(nt_ctx* c, const uint64_t* in, int64_t n, uint64_t* out) {
  if (!c || !in || !out || n < 0) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  DevBuf a, b;
  NT_CUDA(c, a.ensure((size_t)n * 32 + 32));
  NT_CUDA(c, b.ensure((size_t)n * 16 + 16));
  NT_CUDA(c, copy_in(a.p, in, (size_t)n * 32, c->stream));
  launch_threefry_debug(a.as<uint64_t>(), n, b.as<uint64_t>(), c->stream);
  NT_CUDA(c, cudaGetLastError());
  NT_CUDA(c, cudaMemcpyAsync(out, b.p, (size_t)n * 16, cudaMemcpyDefault, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  a.release();
  b.release();
  return NT_OK;
}

nt_status nt_debug_xs(nt_ctx* c, const double* energies, int64_t n, double* out_s, double* out_a) {
  if (!c || !energies || !out_s || !out_a || n < 0) return NT_ERR_ARG;
  cudaSetDevice(c->device);
  if (c->stage < ST_XS) return fail(c, NT_ERR_STATE, "no cross sections loaded");
  DevBuf a, b;
  NT_CUDA(c, a.ensure((size_t)n * 8 + 8));
  NT_CUDA(c, b.ensure((size_t)n * 16 + 16));
  NT_CUDA(c, copy_in(a.p, energies, (size_t)n * 8, c->stream));
  launch_xs_debug(xs_tables(c), a.as<double>(), n, b.as<double>(), b.as<double>() + n, c->stream);
  NT_CUDA(c, cudaGetLastError());
  NT_CUDA(c, cudaMemcpyAsync(out_s, b.p, (size_t)n * 8, cudaMemcpyDefault, c->stream));
  NT_CUDA(c, cudaMemcpyAsync(out_a, b.as<double>() + n, (size_t)n * 8, cudaMemcpyDefault, c->stream));
  NT_CUDA(c, cudaStreamSynchronize(c->stream));
  a.release();
  b.release();
  return NT_OK;
}

}  // extern "C"
