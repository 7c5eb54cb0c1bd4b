// nt_event.cu -- event-based (Over Events) variant of the tracker, P:358-390 (§V-B).
//
// Listing 2 advances every particle by one event per iteration.  One iteration here is two
// kernels: ev_compact builds the three event queues (collision, facet, census) from each
// particle's classified next event -- warp ballots + popc give each lane its rank, a
// block-wide prefix sum over the warps orders the block's chunk, and one atomicAdd per
// block per queue places the chunk -- so every queue is a set of particle-index-ordered
// runs and the handlers' column accesses stay coalesced; then ev_step handles every queued
// event (one thread per event) and classifies that particle's next event.
// The per-particle cached state that Over Particles keeps in registers lives
// in memory columns here.  The iteration loop stays on the device: a CUDA graph
// whose conditional WHILE node runs [ev_compact, ev_step] until the queues are empty (the
// last compaction block sets the loop condition with cudaGraphSetConditional).
// Arithmetic: DESIGN.md §3, identical to the history kernel, so per-particle results
// match it (and the oracle) bit for bit.
#include <cstdlib>
#include <cstring>
#include <cub/device/device_radix_sort.cuh>

#include "nt_event.h"

namespace nt {

struct EvCols {
  double *st, *pa, *H, *nd, *dcen, *acc, *dstep, *iox, *ioy, *exn, *eyn, *evd;
  uint32_t *nf, *nc, *seq;
  uint8_t *evax;
  uint8_t *evtype;          // next event: 0 collision, 1 facet, 2 census, 3 none (ended/dead)
};

struct EvCtl {
  unsigned int cnt[3];      // queue lengths being built by ev_compact
  unsigned int cur[3];      // queue lengths of this iteration (read by ev_step)
  unsigned int done;        // ev_compact blocks finished (last-block detection)
  unsigned int iter;
};

struct EvQueues {
  int32_t* q[3];
};

constexpr int kEvBlock = 256;
constexpr int kStatSlots = 1024;

struct EventState {
  int64_t cap = 0;
  void* mem = nullptr;
  EvCols cols{};
  EvQueues qs{};
  EvCtl* ctl = nullptr;
  TrackParams* d_tp = nullptr;
  unsigned long long* slot_u = nullptr;  // [kStatSlots][SU_COUNT]
  double* slot_f = nullptr;              // [kStatSlots][SF_COUNT]
  cudaGraph_t graph = nullptr;
  cudaGraphExec_t exec = nullptr;
  int grid = 0;
  bool graph_det = false;
  int graph_fmt = -1;
};

// ---------------------------------------------------------------------------------------
__device__ __forceinline__ double ev_inf() { return __longlong_as_double(0x7ff0000000000000ll); }

struct Acc {   // per-thread statistics, flushed to a block slot
  uint32_t u[SU_COUNT];
  double f[SF_COUNT];
};

template <int kFmt>
__device__ __forceinline__ double ev_nd(const Mesh& M, int64_t cell, double cn) {
  return number_density<kFmt>(M, M.nd_tab, cell, cn);
}

template <bool kDet>
__device__ __forceinline__ void ev_flush(const TrackParams& P, const EvCols& C, int32_t i,
                                         int32_t cx, int32_t cy, double& acc, double& dstep,
                                         Acc& a) {
  const int64_t cell = cell_index(P.mesh, cx, cy);
  if constexpr (kDet) {
    const uint32_t seq = C.seq[i];
    const unsigned long long slot = atomicAdd(P.rec_count, 1ull);
    if (slot < P.rec_cap) {
      P.rec_key[slot] = ((unsigned long long)cell << 40) |
                        ((unsigned long long)((int64_t)i - P.lo) << 24) |
                        (unsigned long long)(seq & 0xffffffu);
      P.rec_val[slot] = acc;
    }
    if (seq >= (1u << 24)) a.u[SU_REC_OVERFLOW] += 1u;
    C.seq[i] = seq + 1u;
  } else {
    atomicAdd(P.mesh.tally + cell, acc);
  }
  dstep += acc;
  acc = 0.0;
}

// Final write-back of a history that ended (census: alive = true; kill: false).
__device__ __forceinline__ void ev_finish(const TrackParams& P, const EvCols& C, int32_t i,
                                          double x, double y, double ox, double oy, double e,
                                          double w, double mfp, double dstep, int32_t cx,
                                          int32_t cy, uint32_t ctr, bool alive, Acc& a) {
  const uint32_t nf = C.nf[i], nc = C.nc[i];
  if (!(isfinite(x) && isfinite(y) && isfinite(e) && isfinite(w))) a.u[SU_NONFINITE] += 1u;
  P.p.x[i] = x;
  P.p.y[i] = y;
  P.p.ox[i] = ox;
  P.p.oy[i] = oy;
  P.p.e[i] = e;
  P.p.w[i] = w;
  P.p.mfp[i] = mfp;
  P.p.dep[i] += dstep;
  P.p.cx[i] = cx;
  P.p.cy[i] = cy;
  P.p.ctr[i] = ctr;
  P.p.nfac[i] += nf;
  P.p.ncol[i] += nc;
  if (alive) P.p.ncen[i] += 1u; else P.p.status[i] = 0u;
  a.u[SU_FACETS] += nf;
  a.u[SU_COLLISIONS] += nc;
  a.f[SF_TALLY] += dstep;
}

// calculate_time_to_events + determine_next_event (Listing 2).  Returns the queue of the
// particle's next event, or -1 if the history ended here (event cap).
template <bool kDet>
__device__ __forceinline__ int ev_classify(const TrackParams& P, const EvCols& C, int32_t i,
                                           double x, double y, double ox, double oy,
                                           double iox, double ioy, double mfp, double dcen,
                                           double nd, double st, double exn, double eyn,
                                           Acc& a) {
  if ((int64_t)(C.nf[i] + C.nc[i]) >= P.max_events) {
    // guard (R27): count, flush, kill
    double acc = C.acc[i], dstep = C.dstep[i];
    const int32_t cx = P.p.cx[i], cy = P.p.cy[i];
    a.u[SU_EVENT_CAP] += 1u;
    ev_flush<kDet>(P, C, i, cx, cy, acc, dstep, a);
    const double e = P.p.e[i], w = P.p.w[i];
    a.u[SU_KILLED] += 1u;
    a.f[SF_KILLED_E] += w * e;
    a.f[SF_KILLED_W] += w;
    ev_finish(P, C, i, x, y, ox, oy, e, w, mfp, dstep, cx, cy, P.p.ctr[i], false, a);
    return -1;
  }
  const double sig = nd * st;
  double tx = (exn - x) * iox;
  tx = tx < 0.0 ? 0.0 : tx;
  tx = ox != 0.0 ? tx : ev_inf();
  double ty = (eyn - y) * ioy;
  ty = ty < 0.0 ? 0.0 : ty;
  ty = oy != 0.0 ? ty : ev_inf();
  const bool ax = tx < ty;
  const double df = ax ? tx : ty;
  const double dc = sig > 0.0 ? mfp / sig : ev_inf();
  const double ds = dcen;
  int type;
  double d;
  if (dc < df && dc < ds) { type = 0; d = dc; }
  else if (df < ds) { type = 1; d = df; }
  else { type = 2; d = ds; }
  C.evd[i] = d;
  C.evax[i] = ax ? 1u : 0u;
  return type;
}

__device__ __forceinline__ void acc_zero(Acc& a) {
#pragma unroll
  for (int k = 0; k < SU_COUNT; ++k) a.u[k] = 0u;
#pragma unroll
  for (int k = 0; k < SF_COUNT; ++k) a.f[k] = 0.0;
}

// Reduce a block's per-thread statistics into stat slot (blockIdx.x % kStatSlots).
__device__ void acc_flush(Acc& a, unsigned long long* slot_u, double* slot_f) {
  __shared__ unsigned long long s_u[SU_COUNT];
  __shared__ double s_f[SF_COUNT];
  if (threadIdx.x < SU_COUNT) s_u[threadIdx.x] = 0;
  if (threadIdx.x < SF_COUNT) s_f[threadIdx.x] = 0.0;
  __syncthreads();
#pragma unroll
  for (int k = 0; k < SU_COUNT; ++k) {
    unsigned long long v = a.u[k];
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if ((threadIdx.x & 31) == 0 && v) atomicAdd(&s_u[k], v);
  }
#pragma unroll
  for (int k = 0; k < SF_COUNT; ++k) {
    double v = a.f[k];
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if ((threadIdx.x & 31) == 0 && v != 0.0) atomicAdd(&s_f[k], v);
  }
  __syncthreads();
  const int slot = blockIdx.x % kStatSlots;
  if (threadIdx.x < SU_COUNT && s_u[threadIdx.x])
    atomicAdd(slot_u + slot * SU_COUNT + threadIdx.x, s_u[threadIdx.x]);
  if (threadIdx.x < SF_COUNT && s_f[threadIdx.x] != 0.0)
    atomicAdd(slot_f + slot * SF_COUNT + threadIdx.x, s_f[threadIdx.x]);
}

// ---------------------------------------------------------------------------------------
// ev_init: load each alive particle of [lo, hi), set up its cached state and first event.
template <bool kDet, int kFmt>
__global__ void __launch_bounds__(kEvBlock)
ev_init_kernel(const TrackParams* __restrict__ Pp, EvCols C, unsigned long long* slot_u,
               double* slot_f) {
  const TrackParams& P = *Pp;
  Acc a;
  acc_zero(a);
  const int64_t span = P.hi - P.lo;
  for (int64_t j = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; j < span;
       j += (int64_t)gridDim.x * blockDim.x) {
    const int32_t i = (int32_t)(P.lo + j);
    int type = 3;
    if (P.p.status[i] == 1u) {
      const double x = P.p.x[i], y = P.p.y[i], ox = P.p.ox[i], oy = P.p.oy[i];
      const double e = P.p.e[i], mfp = P.p.mfp[i];
      const int32_t cx = P.p.cx[i], cy = P.p.cy[i];
      uint32_t nrange = 0;
      const Mat m = refresh_xs(P.xs, P.ph, e, nrange);
      a.u[SU_XS_RANGE] += nrange;
      const double nd = ev_nd<kFmt>(P.mesh, cell_index(P.mesh, cx, cy), P.ph.cn);
      const double exn = __ldg(P.mesh.ex + cx + (ox > 0.0 ? 1 : 0));
      const double eyn = __ldg(P.mesh.ey + cy + (oy > 0.0 ? 1 : 0));
      const double dcen = speed(e, P.ph) * P.dt;
      const double iox = 1.0 / ox, ioy = 1.0 / oy;
      C.st[i] = m.st;
      C.pa[i] = m.pa;
      C.H[i] = m.H;
      C.nd[i] = nd;
      C.dcen[i] = dcen;
      C.acc[i] = 0.0;
      C.dstep[i] = 0.0;
      C.iox[i] = iox;
      C.ioy[i] = ioy;
      C.exn[i] = exn;
      C.eyn[i] = eyn;
      C.nf[i] = 0u;
      C.nc[i] = 0u;
      if (kDet) C.seq[i] = 0u;
      a.u[SU_ALIVE] += 1u;
      type = ev_classify<kDet>(P, C, i, x, y, ox, oy, iox, ioy, mfp, dcen, nd, m.st, exn, eyn, a);
    }
    C.evtype[i] = (uint8_t)(type < 0 ? 3 : type);
  }
  acc_flush(a, slot_u, slot_f);
}

// ev_compact: queues of this iteration from the particles' next-event types.  Each block
// takes contiguous chunks of kCompactItems particles per thread; warp ballots + popc rank
// the lanes, a block-wide exclusive scan over the warps orders the chunk, and one atomicAdd
// per queue places it.  The last block to finish publishes the lengths and sets the WHILE
// condition (continue while any queue is non-empty).
constexpr int kCompactItems = 8;

__global__ void __launch_bounds__(kEvBlock)
ev_compact_kernel(const TrackParams* __restrict__ Pp, EvCols C, EvQueues Q, EvCtl* ctl,
                  cudaGraphConditionalHandle h, int in_graph) {
  __shared__ unsigned s_wsum[3][kEvBlock / 32];
  __shared__ unsigned s_base[3];
  __shared__ bool s_last;
  const TrackParams& P = *Pp;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int64_t lo = P.lo, span = P.hi - P.lo;
  constexpr int64_t kChunk = (int64_t)kEvBlock * kCompactItems;
  for (int64_t cb = (int64_t)blockIdx.x * kChunk; cb < span; cb += (int64_t)gridDim.x * kChunk) {
    // this thread's kCompactItems consecutive particles
    const int64_t j0 = cb + (int64_t)threadIdx.x * kCompactItems;
    uint8_t ty[kCompactItems];
#pragma unroll
    for (int k = 0; k < kCompactItems; ++k)
      ty[k] = (j0 + k < span) ? C.evtype[lo + j0 + k] : (uint8_t)3;
    unsigned cnt[3] = {0u, 0u, 0u};
#pragma unroll
    for (int k = 0; k < kCompactItems; ++k)
      if (ty[k] < 3) ++cnt[ty[k]];
    // inclusive warp scan of the per-thread counts (3 queues)
    unsigned inc[3];
#pragma unroll
    for (int q = 0; q < 3; ++q) {
      unsigned v = cnt[q];
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const unsigned n = __shfl_up_sync(kFull, v, o);
        if (lane >= o) v += n;
      }
      inc[q] = v;
      if (lane == 31) s_wsum[q][warp] = v;
    }
    __syncthreads();
    if (threadIdx.x < 3) {
      unsigned tot = 0;
      for (int w = 0; w < kEvBlock / 32; ++w) {
        const unsigned v = s_wsum[threadIdx.x][w];
        s_wsum[threadIdx.x][w] = tot;          // exclusive prefix over warps
        tot += v;
      }
      s_base[threadIdx.x] = tot ? atomicAdd(&ctl->cnt[threadIdx.x], tot) : 0u;
    }
    __syncthreads();
    unsigned pos[3];
#pragma unroll
    for (int q = 0; q < 3; ++q) pos[q] = s_base[q] + s_wsum[q][warp] + inc[q] - cnt[q];
#pragma unroll
    for (int k = 0; k < kCompactItems; ++k) {
      const int t = ty[k];
      if (t < 3) Q.q[t][pos[t]++] = (int32_t)(lo + j0 + k);
    }
    __syncthreads();
  }
  // last block: publish this iteration's queue lengths and the loop condition
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) s_last = atomicAdd(&ctl->done, 1u) == gridDim.x - 1;
  __syncthreads();
  if (s_last && threadIdx.x == 0) {
    __threadfence();
    volatile EvCtl* vc = ctl;
    unsigned tot = 0;
    for (int q = 0; q < 3; ++q) {
      const unsigned v = vc->cnt[q];
      vc->cur[q] = v;
      vc->cnt[q] = 0u;
      tot += v;
    }
    vc->done = 0u;
    vc->iter = vc->iter + 1u;
    if (in_graph) cudaGraphSetConditional(h, tot > 0u ? 1u : 0u);
  }
}

// ev_step: handle every queued event of this iteration and enqueue the next ones.
template <bool kDet, int kFmt>
__global__ void __launch_bounds__(kEvBlock, 3)
ev_step_kernel(const TrackParams* __restrict__ Pp, EvCols C, EvQueues Q, const EvCtl* ctl,
               unsigned long long* slot_u, double* slot_f) {
  const TrackParams& P = *Pp;
  const Phys& ph = P.ph;
  const unsigned n0 = ctl->cur[0], n1 = ctl->cur[1], n2 = ctl->cur[2];
  const unsigned total = n0 + n1 + n2;
  Acc a;
  acc_zero(a);
  const int32_t nx = P.mesh.nx, ny = P.mesh.ny;
  for (unsigned j = blockIdx.x * blockDim.x + threadIdx.x; j < total; j += gridDim.x * blockDim.x) {
    int next = 3;
    {
      const int seg = j < n0 ? 0 : (j < n0 + n1 ? 1 : 2);
      const int32_t i = Q.q[seg][j - (seg == 0 ? 0u : (seg == 1 ? n0 : n0 + n1))];
      double x = P.p.x[i], y = P.p.y[i], ox = P.p.ox[i], oy = P.p.oy[i];
      const double w0 = P.p.w[i];
      double mfp = P.p.mfp[i];
      int32_t cx = P.p.cx[i], cy = P.p.cy[i];
      double dcen = C.dcen[i], acc = C.acc[i], dstep = C.dstep[i];
      double nd = C.nd[i], st = C.st[i];
      const double H = C.H[i], d = C.evd[i];
      const double sig = nd * st;
      if (seg == 0) {
        // ---- collision ----
        double e = P.p.e[i], w = w0;
        uint32_t ctr = P.p.ctr[i];
        acc += ((w * d) * sig) * H;
        x = x + d * ox;
        y = y + d * oy;
        dcen = dcen - d;
        const U64x2 r = threefry2x64_20((uint64_t)ctr, 0, (uint64_t)(P.first_id + i), P.seed);
        ctr += 1u;
        C.nc[i] += 1u;
        double mfp_u = u01(r.b);                    // the draw for the new n_mfp
        bool absorbed = false;
        if (!ph.analog) {                           // implicit capture
          w = w * (1.0 - C.pa[i]);
          a.f[SF_ABSORBED_W] += w0 - w;
        } else if (u01(r.b) < C.pa[i]) {           // sampled absorption (R31)
          absorbed = true;
        } else {                                    // scatter: n_mfp from the next counter
          const U64x2 r2 = threefry2x64_20((uint64_t)ctr, 0, (uint64_t)(P.first_id + i), P.seed);
          ctr += 1u;
          mfp_u = u01(r2.a);
        }
        if (absorbed) {
          ev_flush<kDet>(P, C, i, cx, cy, acc, dstep, a);
          a.f[SF_ABSORBED_W] += w;
          a.f[SF_ABSORBED_E] += w * e;
          a.u[SU_ABSORBED] += 1u;
          ev_finish(P, C, i, x, y, ox, oy, e, w, mfp, dstep, cx, cy, ctr, false, a);
        } else {
        const double mu = 1.0 - 2.0 * u01(r.a);
        const double e2 = e * (((ph.AA + ph.twoA * mu) + 1.0) / ph.Ap1sq);
        const double ct = 0.5 * (ph.Ap1 * sqrt(e2 / e) - ph.Am1 * sqrt(e / e2));
        const double sgn = (r.a & 1ull) ? -1.0 : 1.0;
        const double q = 1.0 - ct * ct;
        const double stt = sgn * sqrt(q > 0.0 ? q : 0.0);
        const double nox = ox * ct - oy * stt;
        const double noy = ox * stt + oy * ct;
        ox = nox;
        oy = noy;
        const double tcen = dcen / speed(e, ph);
        e = e2;
        bool kill = e < ph.e_min || w < ph.w_min;   // termination
        if (kill && ph.roulette && !(e < ph.e_min)) {
          // Russian roulette (R32): survive with probability w / w_s at weight w_s
          const U64x2 r3 = threefry2x64_20((uint64_t)ctr, 0, (uint64_t)(P.first_id + i), P.seed);
          ctr += 1u;
          if (u01(r3.a) < w / ph.w_roul) {
            a.f[SF_ROULETTE] += ph.w_roul - w;
            w = ph.w_roul;
            kill = false;
          }
        }
        if (kill) {
          ev_flush<kDet>(P, C, i, cx, cy, acc, dstep, a);
          a.f[SF_KILLED_E] += w * e;
          a.f[SF_KILLED_W] += w;
          a.u[SU_KILLED] += 1u;
          ev_finish(P, C, i, x, y, ox, oy, e, w, mfp, dstep, cx, cy, ctr, false, a);
        } else {
          const double exn = __ldg(P.mesh.ex + cx + (ox > 0.0 ? 1 : 0));
          const double eyn = __ldg(P.mesh.ey + cy + (oy > 0.0 ? 1 : 0));
          dcen = tcen * speed(e, ph);
          uint32_t nrange = 0;
          const Mat m = refresh_xs(P.xs, ph, e, nrange);
          a.u[SU_XS_RANGE] += nrange;
          const double iox = 1.0 / ox, ioy = 1.0 / oy;
          mfp = -log(mfp_u);
          P.p.x[i] = x;
          P.p.y[i] = y;
          P.p.ox[i] = ox;
          P.p.oy[i] = oy;
          P.p.e[i] = e;
          P.p.w[i] = w;
          P.p.mfp[i] = mfp;
          P.p.ctr[i] = ctr;
          C.st[i] = m.st;
          C.pa[i] = m.pa;
          C.H[i] = m.H;
          C.dcen[i] = dcen;
          C.acc[i] = acc;
          C.iox[i] = iox;
          C.ioy[i] = ioy;
          C.exn[i] = exn;
          C.eyn[i] = eyn;
          next = ev_classify<kDet>(P, C, i, x, y, ox, oy, iox, ioy, mfp, dcen, nd, m.st, exn,
                                   eyn, a);
        }
        }
      } else if (seg == 1) {
        // ---- facet ----
        const bool ax = C.evax[i] != 0;
        double iox = C.iox[i], ioy = C.ioy[i], exn = C.exn[i], eyn = C.eyn[i];
        acc += ((w0 * d) * sig) * H;
        const double nm = mfp - d * sig;
        mfp = nm > 0.0 ? nm : 0.0;
        dcen = dcen - d;
        const double xm = x + d * ox, ym = y + d * oy;
        x = ax ? exn : xm;
        y = ax ? ym : eyn;
        ev_flush<kDet>(P, C, i, cx, cy, acc, dstep, a);
        const int32_t c = ax ? cx : cy;
        const bool pos = ax ? (ox > 0.0) : (oy > 0.0);
        const int32_t last = (ax ? nx : ny) - 1;
        const bool refl = pos ? (c == last) : (c == 0);
        if (refl && ph.vacuum) {
          // ---- vacuum boundary (R30): the facet ends the history (escape) ----
          C.nf[i] += 1u;
          a.u[SU_ESCAPED] += 1u;
          a.f[SF_ESCAPED_E] += w0 * P.p.e[i];
          a.f[SF_ESCAPED_W] += w0;
          ev_finish(P, C, i, x, y, ox, oy, P.p.e[i], w0, mfp, dstep, cx, cy, P.p.ctr[i], false, a);
          C.evtype[i] = 3u;
          continue;
        }
        const int32_t c2 = refl ? c : (pos ? c + 1 : c - 1);
        cx = ax ? c2 : cx;
        cy = ax ? cy : c2;
        const bool fx = refl && ax, fy = refl && !ax;
        ox = fx ? -ox : ox;
        iox = fx ? -iox : iox;
        oy = fy ? -oy : oy;
        ioy = fy ? -ioy : ioy;
        const bool pos2 = refl ? !pos : pos;
        const double ev = __ldg((ax ? P.mesh.ex : P.mesh.ey) + (pos2 ? c2 + 1 : c2));
        nd = ev_nd<kFmt>(P.mesh, cell_index(P.mesh, cx, cy), ph.cn);
        exn = ax ? ev : exn;
        eyn = ax ? eyn : ev;
        C.nf[i] += 1u;
        P.p.x[i] = x;
        P.p.y[i] = y;
        if (fx) P.p.ox[i] = ox;
        if (fy) P.p.oy[i] = oy;
        P.p.mfp[i] = mfp;
        P.p.cx[i] = cx;
        P.p.cy[i] = cy;
        C.dcen[i] = dcen;
        C.acc[i] = acc;
        C.dstep[i] = dstep;
        C.nd[i] = nd;
        if (fx) C.iox[i] = iox;
        if (fy) C.ioy[i] = ioy;
        if (ax) C.exn[i] = exn; else C.eyn[i] = eyn;
        next = ev_classify<kDet>(P, C, i, x, y, ox, oy, iox, ioy, mfp, dcen, nd, st, exn, eyn, a);
      } else {
        // ---- census ----
        const double e = P.p.e[i];
        acc += ((w0 * d) * sig) * H;
        x = x + d * ox;
        y = y + d * oy;
        const double nm = mfp - d * sig;
        mfp = nm > 0.0 ? nm : 0.0;
        ev_flush<kDet>(P, C, i, cx, cy, acc, dstep, a);
        a.u[SU_CENSUS] += 1u;
        a.f[SF_CENSUS_E] += w0 * e;
        a.f[SF_CENSUS_W] += w0;
        ev_finish(P, C, i, x, y, ox, oy, e, w0, mfp, dstep, cx, cy, P.p.ctr[i], true, a);
      }
      C.evtype[i] = (uint8_t)(next < 0 ? 3 : next);
    }
  }
  acc_flush(a, slot_u, slot_f);
}

// Sum the statistic slots into the step statistics.
__global__ void ev_stats_kernel(const unsigned long long* __restrict__ slot_u,
                                const double* __restrict__ slot_f, unsigned long long* su,
                                double* sf) {
  const int k = blockIdx.x;
  if (k < SU_COUNT) {
    unsigned long long v = 0;
    for (int s = threadIdx.x; s < kStatSlots; s += blockDim.x) v += slot_u[s * SU_COUNT + k];
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if ((threadIdx.x & 31) == 0 && v) atomicAdd(su + k, v);
  } else {
    const int kf = k - SU_COUNT;
    double v = 0.0;
    for (int s = threadIdx.x; s < kStatSlots; s += blockDim.x) v += slot_f[s * SF_COUNT + kf];
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if ((threadIdx.x & 31) == 0 && v != 0.0) atomicAdd(sf + kf, v);
  }
}

// ---------------------------------------------------------------------------------------
template <bool kDet, int kFmt>
struct EvFns {
  static void* init() { return (void*)ev_init_kernel<kDet, kFmt>; }
  static void* step() { return (void*)ev_step_kernel<kDet, kFmt>; }
};

static void* ev_fn(bool det, int fmt, bool step) {
#define NT_EV(D, F) return step ? EvFns<D, F>::step() : EvFns<D, F>::init()
  if (det) {
    if (fmt == kDensU8) NT_EV(true, kDensU8);
    if (fmt == kDensU16) NT_EV(true, kDensU16);
    NT_EV(true, kDensF64);
  }
  if (fmt == kDensU8) NT_EV(false, kDensU8);
  if (fmt == kDensU16) NT_EV(false, kDensU16);
  NT_EV(false, kDensF64);
#undef NT_EV
}

EventState* event_state_create() { return new EventState(); }

static void graph_release(EventState* s) {
  if (s->exec) cudaGraphExecDestroy(s->exec);
  if (s->graph) cudaGraphDestroy(s->graph);
  s->exec = nullptr;
  s->graph = nullptr;
}

void event_state_destroy(EventState* s) {
  if (!s) return;
  graph_release(s);
  if (s->mem) cudaFree(s->mem);
  delete s;
}

void event_state_invalidate(EventState* s) { (void)s; }

static size_t a256(size_t b) { return (b + 255) & ~(size_t)255; }

static cudaError_t ensure_capacity(EventState* s, int64_t n) {
  if (n <= s->cap && s->mem) return cudaSuccess;
  graph_release(s);
  if (s->mem) cudaFree(s->mem);
  s->mem = nullptr;
  const size_t N = (size_t)(n > 0 ? n : 1);
  const size_t b8 = a256(N * 8), b4 = a256(N * 4), b1 = a256(N);
  const size_t total = 12 * b8 + 3 * b4 + 2 * b1 + 3 * b4 + a256(sizeof(EvCtl)) +
                       a256(sizeof(TrackParams)) + a256(kStatSlots * SU_COUNT * 8) +
                       a256(kStatSlots * SF_COUNT * 8);
  cudaError_t e = cudaMalloc(&s->mem, total);
  if (e != cudaSuccess) {
    s->mem = nullptr;
    s->cap = 0;
    return e;
  }
  char* q = static_cast<char*>(s->mem);
  double** d8[12] = {&s->cols.st, &s->cols.pa, &s->cols.H, &s->cols.nd, &s->cols.dcen,
                     &s->cols.acc, &s->cols.dstep, &s->cols.iox, &s->cols.ioy, &s->cols.exn,
                     &s->cols.eyn, &s->cols.evd};
  for (auto d : d8) { *d = reinterpret_cast<double*>(q); q += b8; }
  s->cols.nf = reinterpret_cast<uint32_t*>(q); q += b4;
  s->cols.nc = reinterpret_cast<uint32_t*>(q); q += b4;
  s->cols.seq = reinterpret_cast<uint32_t*>(q); q += b4;
  s->cols.evax = reinterpret_cast<uint8_t*>(q); q += b1;
  s->cols.evtype = reinterpret_cast<uint8_t*>(q); q += b1;
  for (int k = 0; k < 3; ++k) { s->qs.q[k] = reinterpret_cast<int32_t*>(q); q += b4; }
  s->ctl = reinterpret_cast<EvCtl*>(q); q += a256(sizeof(EvCtl));
  s->d_tp = reinterpret_cast<TrackParams*>(q); q += a256(sizeof(TrackParams));
  s->slot_u = reinterpret_cast<unsigned long long*>(q); q += a256(kStatSlots * SU_COUNT * 8);
  s->slot_f = reinterpret_cast<double*>(q);
  s->cap = n;
  return cudaSuccess;
}

// Build the device-side iteration loop: WHILE (any queue non-empty) { ev_compact; ev_step }.
static cudaError_t build_graph(EventState* s, bool det, int fmt, int sm_count) {
  graph_release(s);
  cudaError_t e = cudaGraphCreate(&s->graph, 0);
  if (e != cudaSuccess) return e;
  cudaGraphConditionalHandle h;
  e = cudaGraphConditionalHandleCreate(&h, s->graph, 1, cudaGraphCondAssignDefault);
  if (e != cudaSuccess) return e;
  alignas(cudaGraphNodeParams) unsigned char cp_buf[sizeof(cudaGraphNodeParams)] = {};
  cudaGraphNodeParams& cp = *reinterpret_cast<cudaGraphNodeParams*>(cp_buf);
  cp.type = cudaGraphNodeTypeConditional;
  cp.conditional.handle = h;
  cp.conditional.type = cudaGraphCondTypeWhile;
  cp.conditional.size = 1;
  cudaGraphNode_t cnode;
  e = cudaGraphAddNode(&cnode, s->graph, nullptr, 0, &cp);
  if (e != cudaSuccess) return e;
  cudaGraph_t body = cp.conditional.phGraph_out[0];

  int per_sm = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, ev_fn(det, fmt, true), kEvBlock, 0);
  if (per_sm < 1) per_sm = 1;
  s->grid = sm_count * per_sm;
  int per_sm_c = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm_c, ev_compact_kernel, kEvBlock, 0);
  if (per_sm_c < 1) per_sm_c = 1;
  const int grid_c = sm_count * (per_sm_c < 4 ? per_sm_c : 4);

  const TrackParams* tp = s->d_tp;
  EvCols cols = s->cols;
  EvQueues qs = s->qs;
  EvCtl* ctl = s->ctl;
  const EvCtl* cctl = s->ctl;
  unsigned long long* su = s->slot_u;
  double* sf = s->slot_f;

  int in_graph = 1;
  void* cmp_args[] = {&tp, &cols, &qs, &ctl, &h, &in_graph};
  cudaKernelNodeParams kc;
  std::memset(&kc, 0, sizeof kc);
  kc.func = (void*)ev_compact_kernel;
  kc.gridDim = dim3(grid_c);
  kc.blockDim = dim3(kEvBlock);
  kc.kernelParams = cmp_args;
  cudaGraphNode_t n_cmp, n_step;
  e = cudaGraphAddKernelNode(&n_cmp, body, nullptr, 0, &kc);
  if (e != cudaSuccess) return e;

  void* step_args[] = {&tp, &cols, &qs, &cctl, &su, &sf};
  cudaKernelNodeParams kp;
  std::memset(&kp, 0, sizeof kp);
  kp.func = ev_fn(det, fmt, true);
  kp.gridDim = dim3(s->grid);
  kp.blockDim = dim3(kEvBlock);
  kp.kernelParams = step_args;
  e = cudaGraphAddKernelNode(&n_step, body, &n_cmp, 1, &kp);
  if (e != cudaSuccess) return e;
  return cudaGraphInstantiate(&s->exec, s->graph, 0);
}

static cudaError_t host_loop(EventState* s, bool det, int fmt, int sm_count, cudaStream_t st,
                             uint32_t& launches) {
  int per_sm_c = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm_c, ev_compact_kernel, kEvBlock, 0);
  if (per_sm_c < 1) per_sm_c = 1;
  const int grid_c = sm_count * (per_sm_c < 4 ? per_sm_c : 4);
  const TrackParams* tp = s->d_tp;
  EvCols cols = s->cols;
  EvQueues qs = s->qs;
  EvCtl* ctl = s->ctl;
  const EvCtl* cctl = s->ctl;
  unsigned long long* su = s->slot_u;
  double* sf = s->slot_f;
  cudaGraphConditionalHandle h = 0;
  int in_graph = 0;
  void* cmp_args[] = {&tp, &cols, &qs, &ctl, &h, &in_graph};
  void* step_args[] = {&tp, &cols, &qs, &cctl, &su, &sf};
  for (;;) {
    for (int k = 0; k < 64; ++k) {
      cudaError_t e = cudaLaunchKernel((void*)ev_compact_kernel, dim3(grid_c), dim3(kEvBlock), cmp_args, 0, st);
      if (e == cudaSuccess)
        e = cudaLaunchKernel(ev_fn(det, fmt, true), dim3(s->grid), dim3(kEvBlock), step_args, 0, st);
      if (e != cudaSuccess) return e;
      launches += 2;
    }
    EvCtl hc;
    cudaError_t e = cudaMemcpyAsync(&hc, s->ctl, sizeof hc, cudaMemcpyDeviceToHost, st);
    if (e == cudaSuccess) e = cudaStreamSynchronize(st);
    if (e != cudaSuccess) return e;
    if (hc.cur[0] + hc.cur[1] + hc.cur[2] == 0u) return cudaSuccess;
  }
}

// One particle range [tp.lo, tp.hi): zero the stat slots, ev_init, the graph loop, and the
// slot reduction into tp.stats_*.
nt_status event_run_range(EventState* s, const TrackParams& tp, bool det, int sm_count,
                          cudaStream_t st, uint32_t& launches, std::string& err) {
  cudaError_t e = ensure_capacity(s, tp.n);
  if (e != cudaSuccess) {
    err = cudaGetErrorString(e);
    return e == cudaErrorMemoryAllocation ? NT_ERR_OOM : NT_ERR_CUDA;
  }
  if (!s->exec || s->graph_det != det || s->graph_fmt != tp.mesh.fmt) {
    e = build_graph(s, det, tp.mesh.fmt, sm_count);
    if (e != cudaSuccess) {
      err = std::string("event graph: ") + cudaGetErrorString(e);
      return NT_ERR_CUDA;
    }
    s->graph_det = det;
    s->graph_fmt = tp.mesh.fmt;
  }
  e = cudaMemcpyAsync(s->d_tp, &tp, sizeof tp, cudaMemcpyHostToDevice, st);
  if (e == cudaSuccess) e = cudaMemsetAsync(s->ctl, 0, sizeof(EvCtl), st);
  if (e == cudaSuccess) e = cudaMemsetAsync(s->slot_u, 0, kStatSlots * SU_COUNT * 8, st);
  if (e == cudaSuccess) e = cudaMemsetAsync(s->slot_f, 0, kStatSlots * SF_COUNT * 8, st);
  if (e != cudaSuccess) { err = cudaGetErrorString(e); return NT_ERR_CUDA; }
  const int64_t span = tp.hi - tp.lo;
  if (span > 0) {
    int64_t blocks = (span + kEvBlock - 1) / kEvBlock;
    if (blocks > (int64_t)sm_count * 16) blocks = (int64_t)sm_count * 16;
    const TrackParams* dtp = s->d_tp;
    EvCols cols = s->cols;
    unsigned long long* su = s->slot_u;
    double* sf = s->slot_f;
    void* args[] = {&dtp, &cols, &su, &sf};
    e = cudaLaunchKernel(ev_fn(det, tp.mesh.fmt, false), dim3((unsigned)blocks), dim3(kEvBlock),
                         args, 0, st);
    ++launches;
    if (std::getenv("NT_EVENT_HOST_LOOP") == nullptr) {
      if (e == cudaSuccess) e = cudaGraphLaunch(s->exec, st);
      launches += 2;   // >= one [ev_compact, ev_step] iteration; the rest run inside the graph
    } else {
      // profiling aid (ncu cannot see kernels inside a conditional graph): the same two
      // kernels launched from the host, 64 iterations between checks of the queue lengths
      e = host_loop(s, det, tp.mesh.fmt, sm_count, st, launches);
    }
    if (e != cudaSuccess) { err = cudaGetErrorString(e); return NT_ERR_CUDA; }
  }
  ev_stats_kernel<<<SU_COUNT + SF_COUNT, 256, 0, st>>>(s->slot_u, s->slot_f, tp.stats_u,
                                                       tp.stats_f);
  ++launches;
  e = cudaGetLastError();
  if (e != cudaSuccess) { err = cudaGetErrorString(e); return NT_ERR_CUDA; }
  return NT_OK;
}

unsigned event_iterations(EventState* s, cudaStream_t st) {
  EvCtl h;
  if (!s || !s->ctl) return 0;
  if (cudaMemcpyAsync(&h, s->ctl, sizeof h, cudaMemcpyDeviceToHost, st) != cudaSuccess) return 0;
  cudaStreamSynchronize(st);
  return h.iter;
}

}  // namespace nt
