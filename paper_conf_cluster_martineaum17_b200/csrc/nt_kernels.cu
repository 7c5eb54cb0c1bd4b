// nt_kernels.cu -- history-based (Over Particles) tracking kernel, source injection,
// deterministic tally application and verification kernels for sm_100a.
//
// DESIGN.md §3 is the arithmetic; §6 is the kernel design.  Paper passages:
//  - Over Particles: one thread follows one particle from birth to census.
//  - Event timers, nearest event wins (Listing 1).
//  - Facet: flush the register-accumulated deposit with one fp64 atomic, load the new
//    cell's density.  Collision: implicit capture + elastic scatter,
//    XS re-lookup, new mean free path.
//  - Census: flush and stop.
#include <cub/device/device_radix_sort.cuh>

#include "nt_internal.h"

namespace nt {

#ifndef NT_SMEM_FSUM
#define NT_SMEM_FSUM 0   // A/B option: per-thread f64 statistic sums in shared memory
#endif
#ifndef NT_XS_EARLY
#define NT_XS_EARLY 0    // A/B option: a collision issues the new energy's XS index loads early
#endif

__device__ __forceinline__ double d_inf() { return __longlong_as_double(0x7ff0000000000000ll); }

#ifndef NT_TIMELINE
#define NT_TIMELINE 0    // dev variant: per-warp start / range-exhausted / end globaltimer stamps
#endif
#if NT_TIMELINE
__device__ unsigned long long g_tl[2][8192][3];
__device__ __forceinline__ unsigned long long gtimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
  return t;
}
#endif

// ---------------------------------------------------------------------------------------
// Mesh edges: edge(i) = (i*W)/n  (DESIGN.md §3 MESH)
__global__ void edges_kernel(double* ex, int32_t nx, double W, double* ey, int32_t ny,
                             double H) {
  const int32_t i = blockIdx.x * blockDim.x + threadIdx.x;
  if (i <= nx) ex[i] = ((double)i * W) / (double)nx;
  if (i <= ny) ey[i] = ((double)i * H) / (double)ny;
}

void launch_edges(double* ex, int32_t nx, double W, double* ey, int32_t ny, double H,
                  cudaStream_t s) {
  const int n = (nx > ny ? nx : ny) + 1;
  edges_kernel<<<(n + 255) / 256, 256, 0, s>>>(ex, nx, W, ey, ny, H);
}

// ---------------------------------------------------------------------------------------
// Source injection: one thread per particle, coalesced SoA stores.
__global__ void __launch_bounds__(256) inject_kernel(const __grid_constant__ InjectParams P) {
  const int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (i >= P.n_local) return;
  const uint64_t pid = (uint64_t)(P.first_id + i);
  const U64x2 r0 = threefry2x64_20(0, 0, pid, P.seed);
  const double x = P.sx + u01(r0.a) * P.sw;
  const double y = P.sy + u01(r0.b) * P.sh;
  const U64x2 r1 = threefry2x64_20(1, 0, pid, P.seed);
  const double theta = kTwoPi * u01(r1.a);
  P.p.x[i] = x;
  P.p.y[i] = y;
  P.p.cx[i] = cell_of(x, P.ex, P.nx, P.W);
  P.p.cy[i] = cell_of(y, P.ey, P.ny, P.H);
  P.p.ox[i] = cos(theta);
  P.p.oy[i] = sin(theta);
  P.p.mfp[i] = -log(u01(r1.b));
  P.p.e[i] = P.e0;
  P.p.w[i] = 1.0;
  P.p.ctr[i] = 2u;
  P.p.status[i] = 1u;
  P.p.nfac[i] = 0u;
  P.p.ncol[i] = 0u;
  P.p.ncen[i] = 0u;
  P.p.dep[i] = 0.0;
  P.p.gid[i] = (int64_t)pid;
}

void launch_inject(const InjectParams& ip, cudaStream_t s) {
  if (ip.n_local <= 0) return;
  const int64_t blocks = (ip.n_local + 255) / 256;
  inject_kernel<<<(unsigned)blocks, 256, 0, s>>>(ip);
}

// ---------------------------------------------------------------------------------------
// History tracking kernel.
//
// Persistent CTAs; each warp claims particles from a global counter with one atomic per
// refill (warp ballot of idle lanes + popc rank), so a lane whose history ends picks up
// a new particle at the next event instead of idling until the warp's longest history
// finishes (the load imbalance of P:344-348).  All of a history's state -- position,
// direction and its reciprocal, energy, weight, mean free paths, census timer, the
// cell's number density, the cached cross sections and the deposit accumulator -- lives
// in registers for the whole history.  Per event the memory traffic is one
// 8 B density gather (facet) and one fp64 RED into the tally (facet / census / kill).
//
// kDet = true: instead of the RED, every flush is written as a (cell, particle, sequence)
// keyed record; the host sorts the records and applies them in the oracle's order.
// kTally (production flushes, tally_mode): 0 one fp64 RED per flush; 1 warp-aggregated;
// 2 the fp64 add emulated with a 64-bit compare-and-swap loop (how fp64 atomics were done
// before native ones); 3 a per-CTA shared-memory copy of a hot window of cells
// (privatisation), merged into the tally with one RED per cell at the end.
//
// kQ (resume_prefetch): a park writes the particle's register state as a queue-ordered record
// (TrackParams::park_rec) instead of the particle store + a queue index, and the resume
// phase streams those records into a per-warp shared-memory ring with cp.async, one batch
// ahead of use, so a refill of parked particles costs shared-memory loads instead of a
// dependent chain of global loads (queue index, then the state, then the XS lookups).
// Measured and rejected as the default (csp 27.0 -> 27.5 ms, split 104.7 -> 107.0 ms,
// profiles/ab/r02_ab20_resume_ring.txt): the resumed phase is not refill-bound -- its time
// goes to the streaming tail of particles scattered back out of dense matter.
template <bool kDet, int kFmt, bool kTiled, bool kBlk, int kMinB, int kTally, bool kXsWalk,
          bool kVar, bool kSlab, bool kAoS = false, bool kFused = false, bool kQ = false>
__global__ void __launch_bounds__(kHistoryBlock, kMinB)
history_kernel(const __grid_constant__ TrackParams P) {
  // particle-store field f of local particle idx: structure of arrays, or -- the
  // AoS ablation (particle_layout 1) -- one 128 B record per particle
#define PP(f, idx) (kAoS ? &P.aos[idx].f : P.p.f + (idx))
  static_assert(!(kSlab && kDet), "slab decomposition: production tally only");
  static_assert(!kBlk || kFmt == kDensU8, "the block map indexes u8 material codes");
  static_assert(!(kTally && kDet), "tally modes reorder the sum: production tally only");
  static_assert(!(kTally == 3 && kSlab), "hot window: replicated meshes only");
  static_assert(!(kAoS && kSlab), "AoS particle store: replicated meshes only");
  static_assert(!(kFused && (kSlab || kDet || kAoS)), "fused phases: production, replicated, SoA");
  static_assert(!(kQ && (kSlab || kDet || kAoS || kFused || kXsWalk)),
                "resume ring: production, replicated, SoA, two launches, table lookups");
  // Statistics: u32 counters per warp in shared memory (native shared atomics); f64 sums in
  // per-thread slots in global memory (touched only when a history ends), so the CTA keeps
  // almost no shared memory and the L1 stays free for the density / edge gathers.
  constexpr int kWarps = kHistoryBlock / 32;
  __shared__ uint32_t s_u[kWarps][SU_COUNT];
  __shared__ double s_nd[kFmt == kDensU8 ? 256 : 1];
  __shared__ __align__(16) uint8_t s_blk[kBlk ? kBlkMax : 1];
  __shared__ double s_wabs[kHistoryBlock];   // weight absorbed by implicit capture, per thread
#if NT_SMEM_FSUM
  // f64 statistic sums per thread in shared memory (a history's end adds 2-3 of them: a
  // shared-memory RMW instead of a global one on the critical path of short histories)
  __shared__ double s_f[SF_COUNT][kHistoryBlock];
#endif
  __shared__ double s_hot[kTally == 3 ? kHotCells : 1];   // privatised hot window (kTally 3)
  const int t = threadIdx.x;
  const int64_t gt = (int64_t)blockIdx.x * kHistoryBlock + t;
  const int64_t sstride = (int64_t)gridDim.x * kHistoryBlock;
  double* __restrict__ sf = P.slot_f + gt;          // sf[k * sstride]: statistic k
#if NT_SMEM_FSUM
#pragma unroll
  for (int k = 0; k < SF_COUNT; ++k) s_f[k][t] = 0.0;
#else
#pragma unroll
  for (int k = 0; k < SF_COUNT; ++k) sf[k * sstride] = 0.0;
#endif
  if (t < kWarps * SU_COUNT) (&s_u[0][0])[t] = 0u;
  if constexpr (kTally == 3)
    for (int k = t; k < kHotCells; k += kHistoryBlock) s_hot[k] = 0.0;
  __syncthreads();
  if constexpr (kFmt == kDensU8) {
    for (int k = t; k < 256; k += kHistoryBlock) s_nd[k] = k < P.mesh.ncodes ? P.mesh.nd_tab[k] : 0.0;
    if constexpr (kBlk) {
      const uint4* src = reinterpret_cast<const uint4*>(P.mesh.blk);
      for (int k = t; k < (P.mesh.nblk + 15) / 16; k += kHistoryBlock)
        reinterpret_cast<uint4*>(s_blk)[k] = __ldg(src + k);
    }
    __syncthreads();
  }
  const int wid = t >> 5;
  auto cnt = [&](int k, uint32_t v) { atomicAdd(&s_u[wid][k], v); };
#if NT_SMEM_FSUM
  auto fsum = [&](int k, double v) { s_f[k][t] += v; };
#else
  auto fsum = [&](int k, double v) { red_add_f64(sf + k * sstride, v); };
#endif
  s_wabs[t] = 0.0;
  const double* __restrict__ ndtab = (kFmt == kDensU8) ? s_nd : P.mesh.nd_tab;

  const int lane = t & 31;
  const unsigned lt_mask = (1u << lane) - 1u;
  const unsigned long long span = (unsigned long long)(P.hi - P.lo);
  const double* __restrict__ ex = P.mesh.ex;
  const double* __restrict__ ey = P.mesh.ey;
  const int32_t nx = P.mesh.gnx, ny = P.mesh.ny;      // reflection bounds (whole mesh)
  const int32_t snx = P.mesh.nx, x0 = P.mesh.x0;      // storage width, first stored column
  const Phys& ph = P.ph;
  const uint32_t strip = (uint32_t)P.mesh.strip;        // tiled: cells per row of tiles
  // storage index of (cx, cy): 4x4 tiles (kTiled) or row-major, as nt_device.cuh cell_index
  // (32-bit: nt_init_mesh guarantees the storage fits 2^32 cells)
  auto cidx_of = [&](int32_t cx_, int32_t cy_) -> uint32_t {
    const uint32_t lx = kSlab ? (uint32_t)(cx_ - x0) : (uint32_t)cx_;   // x-slab storage offset
    if constexpr (kTiled)
      return (uint32_t)(cy_ >> 2) * strip + (lx << 2) + (uint32_t)(cy_ & 3);
    else
      return (uint32_t)cy_ * (uint32_t)snx + lx;
  };
  const uint32_t max_ev = P.max_events < 0xffffffffll ? (uint32_t)P.max_events : 0xffffffffu;
  const uint64_t pol_keep = l2_evict_last();     // tally REDs, density gathers
  const uint64_t pol_stream = l2_evict_first();  // particle store (read / written once)
  // global id of local particle i (the RNG key)
  auto pid_of = [&](int32_t i_) -> uint64_t {
    if constexpr (kSlab) return (uint64_t)__ldg(P.p.gid + i_);
    else return (uint64_t)(P.first_id + i_);
  };
  // density (code) of cell (cx_, cy_) at storage index ci_: issue the gather (with the block
  // map: the block's code from shared memory, the cell's own only in mixed blocks).  Measured
  // and rejected in round 2 (profiles/ab/r02_ab4, r02_ab8): keeping the code while a facet
  // stays inside a uniform block (more spills), and issuing the facet's edge and density
  // loads before its deposit arithmetic (csp +0.5%, split +2%).
  auto dload = [&](int32_t cx_, int32_t cy_, uint32_t ci_) {
    NT_CHECK(ci_ < storage_cells(P.mesh));
    if constexpr (kBlk) {
      const int32_t lx = kSlab ? cx_ - P.mesh.x0 : cx_;
      uint32_t code = s_blk[(cy_ >> P.mesh.bshift) * P.mesh.nbx + (lx >> P.mesh.bshift)];
      if (code == kBlkMixed) code = ldg_u8_hint(P.mesh.rho8 + ci_, pol_keep);
      return code;
    } else {
      return dens_load<kFmt>(P.mesh, ci_, pol_keep);
    }
  };

  bool active = false, exhausted = false;
  int32_t i = 0;                 // local particle index (< 2^31)
#if NT_TIMELINE
  const int tl_w = (int)((blockIdx.x * kHistoryBlock + threadIdx.x) >> 5);
  const int tl_p = P.phase == 2 ? 1 : 0;
  if ((threadIdx.x & 31) == 0 && tl_w < 8192) { g_tl[tl_p][tl_w][0] = gtimer(); g_tl[tl_p][tl_w][1] = 0; }
#endif
  // register-resident history state
  double x = 0, y = 0, ox = 0, oy = 0, iox = 0, ioy = 0, e = 0, w = 0, mfp = 0, dcen = 0;
  typename DensRaw<kFmt>::type draw = 0;  // density (code) of the current cell, as loaded
  double exn = 0, eyn = 0;  // edge each axis is heading to (facet distance, snap value)
  double acc = 0;     // deposit accumulated in the current cell
  double dstep = 0;   // deposits this particle flushed this step
  Mat m{0, 0, 0};
  int32_t cx = 0, cy = 0;
  uint32_t cidx = 0;         // storage index of (cx, cy)
  uint32_t ctr = 0, nf = 0, nc = 0;
  uint32_t seq = 0;          // flush sequence number (deterministic records only)
  // XS clamp counts go straight to the warp's shared counter (rare)
  auto xs_refresh = [&](double e_) {
    uint32_t nr = 0;
    const Mat mm = refresh_xs(P.xs, ph, e_, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    return mm;
  };
  int32_t bin_s = 0, bin_a = 0;   // kXsWalk: the bins of the last lookup

  // Regime parking: phase 1 tracks particles [lo, hi); phase 2 resumes the
  // particles phase 1 parked.  Phase 1 parks a lane whose next event is a collision while
  // fewer than park_coll_below lanes of its warp collide: its state goes to the particle
  // store, its index to the out-queue, and the lane takes a new particle.  So the particles
  // that reach dense matter collide warp-converged in phase 2.  Per-particle results are
  // unchanged.
  const bool resume = P.resume_q != nullptr;
  const unsigned long long span2 = resume ? *P.resume_count : span;
  const int park_coll_below = P.park_coll_below;
  // Fused phases (kFused): one launch; consumer warps resume parked particles while the
  // producers still run phase 1, so the parked collisions' ALU work fills the issue slots
  // the RED-bound streaming leaves free.  Per lane: res = the particle is a resumed one;
  // a consumer lane holds at most one claimed queue position (pend, qpos) and is done (fin)
  // once every producer has finished and its claim lies beyond the final queue length.
  bool consumer = kFused && (int)blockIdx.x < P.coll_ctas;
  // a producer warp turns consumer as soon as its particle range is exhausted, while its
  // own (producer) lanes still run: their idle lanes resume parked particles instead of
  // waiting for the warp's last history (the phase-1 tail).  prod_live: producer lanes may
  // still park -- the warp counts itself done (prod_done) once none is left.
  bool prod_live = kFused && !consumer;
  bool res = resume, pend = false, fin = false;
  uint32_t qpos = 0;
  // Park this lane: the state before its next event to the particle store (status st), the
  // index to queue q (one atomicAdd per group of converged lanes); the lane goes idle and
  // takes a new particle.  Used for regime parking (status 2, park_q) and, with x-slabs,
  // for emigrants (status 4, out_q).
  auto park_to = [&](uint8_t st, int32_t* q, unsigned long long* qn) {
    if constexpr (kQ) {
      // the register state as record k of the queue-ordered park buffer (status stays 1)
      const unsigned am = __activemask();
      const int ld = __ffs(am) - 1;
      unsigned long long k = 0;
      if (lane == ld) k = atomicAdd(qn, (unsigned long long)__popc(am));
      k = __shfl_sync(am, k, ld) + (unsigned long long)__popc(am & lt_mask);
      NT_CHECK(k < (unsigned long long)P.park_cap);
      const int64_t C = P.park_cap;
      double* f = P.park_rec + k;
      uint32_t* u = reinterpret_cast<uint32_t*>(P.park_rec + kParkF64 * C) + k;
      f[0] = x; f[C] = y; f[2 * C] = ox; f[3 * C] = oy; f[4 * C] = exn; f[5 * C] = eyn;
      f[6 * C] = e; f[7 * C] = w; f[8 * C] = mfp; f[9 * C] = dcen; f[10 * C] = acc;
      f[11 * C] = dstep; f[12 * C] = m.st; f[13 * C] = m.pa; f[14 * C] = m.H;
      u[0] = (uint32_t)cx; u[C] = (uint32_t)cy; u[2 * C] = ctr; u[3 * C] = nf; u[4 * C] = nc;
      u[5 * C] = (uint32_t)i;
      (void)st; (void)q;
      active = false;
      return;
    }
    (*PP(x, i)) = x;
    (*PP(y, i)) = y;
    (*PP(ox, i)) = ox;
    (*PP(oy, i)) = oy;
    (*PP(e, i)) = e;
    (*PP(w, i)) = w;
    (*PP(mfp, i)) = mfp;
    (*PP(cx, i)) = cx;
    (*PP(cy, i)) = cy;
    (*PP(ctr, i)) = ctr;
    (*PP(dcen, i)) = dcen;
    (*PP(acc, i)) = acc;
    (*PP(dstep, i)) = dstep;
    (*PP(nf_s, i)) = nf;
    (*PP(nc_s, i)) = nc;
    if constexpr (kDet) (*PP(seq_s, i)) = seq;
    (*PP(status, i)) = st;
    const unsigned am = __activemask();
    const int ld = __ffs(am) - 1;
    unsigned long long k = 0;
    if (lane == ld) k = atomicAdd(qn, (unsigned long long)__popc(am));
    k = __shfl_sync(am, k, ld) + (unsigned long long)__popc(am & lt_mask);
    if constexpr (kFused) {
      // publish to consumers running in this launch: the state, then the entry (index + 1)
      __threadfence();
      st_volatile(q + k, i + 1);
    } else {
      NT_CHECK(k < (unsigned long long)P.n || q == P.out_q);
      q[k] = i;
    }
    active = false;
  };
  auto outside_slab = [&](int32_t cx_) { return cx_ < P.slab_lo || cx_ >= P.slab_hi; };

  // set up the per-history registers of the particle just loaded (x .. ctr, e known)
  auto setup_loaded = [&]() __attribute__((always_inline)) {
    exn = __ldg(ex + cx + (ox > 0.0 ? 1 : 0));
    eyn = __ldg(ey + cy + (oy > 0.0 ? 1 : 0));
    iox = 1.0 / ox;
    ioy = 1.0 / oy;
    if (ox == 0.0) { exn = d_inf(); iox = d_inf(); }
    if (oy == 0.0) { eyn = d_inf(); ioy = d_inf(); }
  };

  // ---- resume ring (kQ, phase 2): per warp two halves of kRingB records in shared memory ----
  // rh: the half being consumed (rpos of rcnt records used); the other half receives the
  // batch claimed at the previous swap (fcnt records, cp.async in flight); cb_raw (lane 0)
  // is the next batch's claim, consumed at the next swap -- so neither the claim's atomic
  // nor the copies stall a refill.
  extern __shared__ __align__(16) unsigned char dsm[];
  unsigned char* ring = dsm + (size_t)wid * 2 * kRingHalfBytes;
  // ring state packed in one register (live through phase 1 too): bit 0 rh, bits 1-7 rpos,
  // 8-15 rcnt, 16-23 fcnt; cb_raw keeps the claim's low word (positions < 2^31)
  uint32_t rstate = 0;
  uint32_t cb_raw = 0;
  auto rvalid = [&](unsigned long long b) -> int {
    return b < span2 ? (int)(span2 - b < (unsigned long long)kRingB ? span2 - b : kRingB) : 0;
  };
  // all 32 lanes: copy records [b, b + kRingB) into half hf (16-byte chunks, coalesced)
  auto ring_issue = [&](unsigned long long b, int hf) __attribute__((always_inline)) {
    const int64_t C = P.park_cap;
    unsigned char* hb = ring + hf * kRingHalfBytes;
    constexpr int kF = kParkF64 * (kRingB / 2), kU = kParkU32 * (kRingB / 4);
    for (int ck = lane; ck < kF + kU; ck += 32) {
      const void* src;
      unsigned char* dst;
      if (ck < kF) {
        const int col = ck / (kRingB / 2), part = ck % (kRingB / 2);
        src = P.park_rec + col * C + (int64_t)b + 2 * part;
        dst = hb + col * (kRingB * 8) + part * 16;
      } else {
        const int c2 = ck - kF, col = c2 / (kRingB / 4), part = c2 % (kRingB / 4);
        src = reinterpret_cast<const uint32_t*>(P.park_rec + kParkF64 * C) + col * C + (int64_t)b + 4 * part;
        dst = hb + kParkF64 * kRingB * 8 + col * (kRingB * 4) + part * 16;
      }
      cp_async16(dst, src);
    }
    cp_async_commit();
  };
  if constexpr (kQ) {
    if (resume) {
      unsigned long long b0 = 0;
      if (lane == 0) b0 = atomicAdd(P.counter, (unsigned long long)kRingB);
      b0 = __shfl_sync(kFull, b0, 0);
      const int rcnt = rvalid(b0);
      if (rcnt > 0) ring_issue(b0, 0);
      unsigned long long b1 = 0;
      if (lane == 0) b1 = atomicAdd(P.counter, (unsigned long long)kRingB);
      b1 = __shfl_sync(kFull, b1, 0);
      const int fcnt = rvalid(b1);
      if (fcnt > 0) {
        ring_issue(b1, 1);
        if (lane == 0) cb_raw = (uint32_t)atomicAdd(P.counter, (unsigned long long)kRingB);
      }
      if (fcnt > 0) cp_async_wait_group1();   // batch b0 has landed (b1 may be in flight)
      else cp_async_wait_all();
      __syncwarp();
      rstate = ((uint32_t)rcnt << 8) | ((uint32_t)fcnt << 16);
    }
  }

  for (;;) {
    if constexpr (kFused) {
      if (prod_live && consumer && !__any_sync(kFull, active && !res)) {
        __threadfence();                     // this warp's parks are published
        if (lane == 0) atomicAdd(P.prod_done, 1u);
        prod_live = false;
      }
      if (consumer) {
        // ---- consumer refill: claim queue positions for idle lanes, take published ones ----
        const unsigned want = __ballot_sync(kFull, !active && !pend && !fin);
        if (want) {
          const int leader = __ffs(want) - 1;
          unsigned long long base = 0;
          if (lane == leader) base = atomicAdd(P.park_taken, (unsigned long long)__popc(want));
          base = __shfl_sync(kFull, base, leader);
          if (!active && !pend && !fin) {
            const unsigned long long q = base + (unsigned long long)__popc(want & lt_mask);
            // a particle is parked at most once, so positions past the store are never filled
            if (q >= (unsigned long long)P.n) fin = true;
            else { qpos = (uint32_t)q; pend = true; }
          }
        }
        if (pend) {
          int32_t v = ld_volatile(P.park_q + qpos);
          if (v == 0 && ld_volatile(P.prod_done) >= P.n_prod) {
            // every producer is done: the queue is final
            if ((unsigned long long)qpos >= ld_volatile(P.park_count)) { fin = true; pend = false; }
            else v = ld_volatile(P.park_q + qpos);
          }
          if (v != 0) {
            // a parked particle (status 2): its state from L2 (written by another CTA before
            // the fence that precedes the entry)
            __threadfence();
            pend = false;
            i = v - 1;
            active = true;
            res = true;
            x = __ldcg(P.p.x + i);
            y = __ldcg(P.p.y + i);
            ox = __ldcg(P.p.ox + i);
            oy = __ldcg(P.p.oy + i);
            e = __ldcg(P.p.e + i);
            w = __ldcg(P.p.w + i);
            mfp = __ldcg(P.p.mfp + i);
            cx = __ldcg(P.p.cx + i);
            cy = __ldcg(P.p.cy + i);
            ctr = __ldcg(P.p.ctr + i);
            dcen = __ldcg(P.p.dcen + i);
            acc = __ldcg(P.p.acc + i);
            dstep = __ldcg(P.p.dstep + i);
            nf = __ldcg(P.p.nf_s + i);
            nc = __ldcg(P.p.nc_s + i);
            setup_loaded();
            uint32_t nr_dummy = 0;              // (the producer counted the XS clamps)
            m = refresh_xs(P.xs, ph, e, nr_dummy);
            cidx = cidx_of(cx, cy);
            draw = dload(cx, cy, cidx);
          }
        }
        if (!__any_sync(kFull, active)) {
          if (__all_sync(kFull, fin)) break;
          __nanosleep(256);
          continue;
        }
      }
    }
    // ---- refill idle lanes with new particles: one atomic per warp ----
    const unsigned idle = __ballot_sync(kFull, !active);
    if (kQ && resume) {
      if (!exhausted && idle != 0u && (__popc(idle) >= P.refill_min || idle == kFull)) {
        int rh = (int)(rstate & 1u), rpos = (int)((rstate >> 1) & 127u);
        int rcnt = (int)((rstate >> 8) & 255u), fcnt = (int)((rstate >> 16) & 255u);
        unsigned need = idle;
        while (need != 0u) {
          if (rpos == rcnt) {                  // the consumed half is used up: swap
            if (fcnt == 0) { exhausted = true; break; }
            cp_async_wait_all();
            __syncwarp();
            rh ^= 1;
            rpos = 0;
            rcnt = fcnt;
            const unsigned long long cb = __shfl_sync(kFull, cb_raw, 0);
            fcnt = rvalid(cb);
            if (fcnt > 0) {
              ring_issue(cb, rh ^ 1);
              if (lane == 0) cb_raw = (uint32_t)atomicAdd(P.counter, (unsigned long long)kRingB);
            }
          }
          const int take = min(rcnt - rpos, __popc(need));
          const int rank = __popc(need & lt_mask);
          const bool mine = ((need >> lane) & 1u) && rank < take;
          if (mine) {
            const int r = rpos + rank;
            NT_CHECK(r < kRingB);
            const unsigned char* hb = ring + rh * kRingHalfBytes;
            const double* f = reinterpret_cast<const double*>(hb) + r;
            const uint32_t* u = reinterpret_cast<const uint32_t*>(hb + kParkF64 * kRingB * 8) + r;
            x = f[0]; y = f[kRingB]; ox = f[2 * kRingB]; oy = f[3 * kRingB];
            exn = f[4 * kRingB]; eyn = f[5 * kRingB]; e = f[6 * kRingB]; w = f[7 * kRingB];
            mfp = f[8 * kRingB]; dcen = f[9 * kRingB]; acc = f[10 * kRingB];
            dstep = f[11 * kRingB]; m.st = f[12 * kRingB]; m.pa = f[13 * kRingB];
            m.H = f[14 * kRingB];
            cx = (int32_t)u[0]; cy = (int32_t)u[kRingB]; ctr = u[2 * kRingB];
            nf = u[3 * kRingB]; nc = u[4 * kRingB]; i = (int32_t)u[5 * kRingB];
            iox = 1.0 / ox;
            ioy = 1.0 / oy;
            if (ox == 0.0) iox = d_inf();
            if (oy == 0.0) ioy = d_inf();
            active = true;
            res = true;
            cidx = cidx_of(cx, cy);
            draw = dload(cx, cy, cidx);
          }
          rpos += take;
          need &= ~__ballot_sync(kFull, mine);
        }
        rstate = (uint32_t)rh | ((uint32_t)rpos << 1) | ((uint32_t)rcnt << 8) | ((uint32_t)fcnt << 16);
      }
    } else if (!consumer && !exhausted && idle != 0u && (__popc(idle) >= P.refill_min || idle == kFull)) {
      const int leader = __ffs(idle) - 1;
      unsigned long long base = 0;
      if (lane == leader) base = atomicAdd(P.counter, (unsigned long long)__popc(idle));
      base = __shfl_sync(kFull, base, leader);
      if (base + (unsigned long long)__popc(idle) >= span2) {
#if NT_TIMELINE
        if (!exhausted && lane == 0 && tl_w < 8192) g_tl[tl_p][tl_w][1] = gtimer();
#endif
        exhausted = true;
        if constexpr (kFused) consumer = true;   // mixed from here on (prod_live until done)
      }
      if (!active) {
        const unsigned long long my = base + (unsigned long long)__popc(idle & lt_mask);
        if (my < span2) {
          i = resume ? P.resume_q[my] : (int32_t)(P.lo + (int64_t)my);
          NT_CHECK(i >= 0 && (int64_t)i < P.n);
          // the state loads are issued together with the status load (one round trip to
          // the particle store instead of two; a skipped particle's loads are wasted)
          const uint32_t st_i = *PP(status, i);
          x = ld_stream(PP(x, i), pol_stream);
          y = ld_stream(PP(y, i), pol_stream);
          ox = ld_stream(PP(ox, i), pol_stream);
          oy = ld_stream(PP(oy, i), pol_stream);
          e = ld_stream(PP(e, i), pol_stream);
          w = ld_stream(PP(w, i), pol_stream);
          mfp = ld_stream(PP(mfp, i), pol_stream);
          cx = ld_stream(PP(cx, i), pol_stream);
          cy = ld_stream(PP(cy, i), pol_stream);
          ctr = ld_stream(PP(ctr, i), pol_stream);
          if (resume) {              // the parked state
            dcen = ld_stream(PP(dcen, i), pol_stream);
            acc = ld_stream(PP(acc, i), pol_stream);
            dstep = ld_stream(PP(dstep, i), pol_stream);
            nf = ld_stream(PP(nf_s, i), pol_stream);
            nc = ld_stream(PP(nc_s, i), pol_stream);
            if constexpr (kDet) seq = ld_stream(PP(seq_s, i), pol_stream);
          }
          if (st_i == (resume ? 2u : 1u)) {
            active = true;
            res = resume;
            setup_loaded();
            if constexpr (kXsWalk) {
              bin_s = xs_bin(P.xs.s, clamp_only(e, P.xs.s));
              bin_a = xs_bin(P.xs.c, clamp_only(e, P.xs.c));
            }
            if (!resume) {
              m = xs_refresh(e);
              dcen = speed(e, ph) * P.dt;
              acc = 0.0;
              dstep = 0.0;
              nf = 0u;
              nc = 0u;
              seq = 0u;
              cnt(SU_ALIVE, 1u);
            } else {                 // parked (loaded above; phase 1 counted the XS clamps)
              uint32_t nr_dummy = 0;
              m = refresh_xs(P.xs, ph, e, nr_dummy);
            }
            // born (or resumed) outside this rank's slab: hand over before any event (and
            // before touching the density, which this rank holds for its columns only)
            bool stay = true;
            if constexpr (kSlab) {
              if (outside_slab(cx)) {
                park_to(4u, P.out_q, P.out_count);
                stay = false;
              }
            }
            if (stay) {
              cidx = cidx_of(cx, cy);
              draw = dload(cx, cy, cidx);
            }
          }
        }
      }
    }
    if (!__any_sync(kFull, active)) {
      if (kFused && consumer) continue;    // the consumer block at the loop top decides
      if (exhausted) {
#if NT_TIMELINE
        if (lane == 0 && tl_w < 8192) g_tl[tl_p][tl_w][2] = gtimer();
#endif
        break;
      }
      continue;
    }

    // ---- events until enough lanes are idle to refill (or none is active) ----
    // event(capped): capped = true handles only the event-cap kill (R27)
    auto event = [&](bool capped) __attribute__((always_inline)) {
        // ---- one event (Listing 1) ----
        // consume the gathers issued by the previous facet (density code, next edge)
        double nd;
        if constexpr (kFmt == kDensU8) nd = s_nd[draw];
        else nd = dens_nd<kFmt>(draw, ndtab, ph.cn);
        const double sig = nd * m.st;
        // An axis with direction cosine 0 carries exn = iox = +inf (set where the direction
        // changes), so (exn - x) * iox = +inf without a select -- the "ω = 0 -> ∞" of §3.
        // §3 clamps tx and ty at 0 and takes X iff clamped tx < clamped ty (tie -> Y).
        // max(tx,0) < max(ty,0) <=> ty > 0 && tx < ty, and the clamped minimum is the
        // minimum clamped, so one clamp of the chosen distance gives the same df (±0 and
        // all; R28).
        const double tx = (exn - x) * iox;
        const double ty = (eyn - y) * ioy;
        const bool ax = ty > 0.0 && tx < ty;
        double df = ax ? tx : ty;
        df = df < 0.0 ? 0.0 : df;
        const double ds = dcen;
        // dc = n_mfp / Sigma_t only matters if a collision is possible: when
        // n_mfp > (min(df, ds) * Sigma_t) * (1 + 2^-20) the rounded quotient provably exceeds
        // min(df, ds), so the event is not a collision and dc is never used.
        // (The relative-error argument needs a normal product: below 2^-960 the division is
        // taken.)  Both constants have a zero low word, so they are instruction immediates.
        const double dmin = df < ds ? df : ds;
        const double dsig = dmin * sig;
        const bool maybe_coll = !(mfp > dsig * 0x1.00001p+0) || dsig < 0x1p-960;
        double dc = d_inf();
        bool coll = false;
        if (__builtin_expect(maybe_coll && sig > 0.0, 0)) {  // branch, not a select
          dc = mfp / sig;
          coll = dc < df && dc < ds;
        }
        int outcome = 0;                      // 0 continue, 1 census, 2 dead
        auto flush = [&]() {
          const uint32_t cell = cidx;                // storage index of the current cell
          NT_CHECK(cell < storage_cells(P.mesh) && (uint32_t)i < (uint32_t)P.n);
          if constexpr (kDet) {
            const unsigned long long slot = atomicAdd(P.rec_count, 1ull);
            if (slot < P.rec_cap) {
              P.rec_key[slot] = ((unsigned long long)cell << 40) |
                                ((unsigned long long)((int64_t)i - P.lo) << 24) |
                                (unsigned long long)(seq & 0xffffffu);
              P.rec_val[slot] = acc;
            }
            if (seq >= (1u << 24)) cnt(SU_REC_OVERFLOW, 1u);
            ++seq;
          } else if constexpr (kTally == 1) {
            red_add_warp(P.mesh.tally, cell, acc, pol_keep);
          } else if constexpr (kTally == 2) {
            // fp64 add by compare-and-swap on the 64-bit word (retried while another thread
            // changed the cell in between)
            unsigned long long* a = reinterpret_cast<unsigned long long*>(P.mesh.tally + cell);
            unsigned long long old = *a, assumed;
            do {
              assumed = old;
              old = atomicCAS(a, assumed,
                              (unsigned long long)__double_as_longlong(__longlong_as_double((long long)assumed) + acc));
            } while (assumed != old);
          } else if constexpr (kTally == 3) {
            const uint32_t hx = (uint32_t)(cx - P.hot_x0), hy = (uint32_t)(cy - P.hot_y0);
            if (hx < (uint32_t)P.hot_nx && hy < (uint32_t)P.hot_ny)
              atomicAdd(&s_hot[hy * (uint32_t)P.hot_nx + hx], acc);     // shared-memory atomic
            else
              red_add_hint(P.mesh.tally + cell, acc, pol_keep);
          } else {
            red_add_hint(P.mesh.tally + cell, acc, pol_keep);   // fire-and-forget fp64 RED at L2
          }
          dstep += acc;
          acc = 0.0;
        };

        if (capped) {
          // guard (R27): count, flush, kill
          cnt(SU_EVENT_CAP, 1u);
          flush();
          cnt(SU_KILLED, 1u);
          fsum(SF_KILLED_E, w * e);
          fsum(SF_KILLED_W, w);
          outcome = 2;
        } else if (coll && !(kFused && res) && __popc(__activemask()) < park_coll_below) {
          park_to(2u, P.park_q, P.park_count);
        } else if (coll) {
          // ---- collision (implicit capture + elastic scatter) ----
          acc += ((w * dc) * sig) * m.H;
          x = x + dc * ox;
          y = y + dc * oy;
          dcen = dcen - dc;
          const U64x2 r = threefry2x64_20((uint64_t)ctr, 0, pid_of(i), P.seed);
          ctr += 1u;
          nc += 1u;
          double mfp_u = u01(r.b);                  // the draw for the new n_mfp
          bool absorbed = false;
          if (!(kVar && ph.analog)) {               // implicit capture
            const double w_old = w;
            w = w * (1.0 - m.pa);
            s_wabs[t] += w_old - w;
          } else if (u01(r.b) < m.pa) {            // sampled absorption (R31)
            absorbed = true;
          } else {                                  // scatter branch: n_mfp from the next counter
            const U64x2 r2 = threefry2x64_20((uint64_t)ctr, 0, pid_of(i), P.seed);
            ctr += 1u;
            mfp_u = u01(r2.a);
          }
          if (absorbed) {
            flush();
            s_wabs[t] += w;
            fsum(SF_ABSORBED_E, w * e);
            cnt(SU_ABSORBED, 1u);
            outcome = 2;
          } else {
            const double mu = 1.0 - 2.0 * u01(r.a);
            const double e2 = e * (((ph.AA + ph.twoA * mu) + 1.0) / ph.Ap1sq);
#if NT_XS_EARLY
            // the new energy's table bins: issue the index loads now, so their latency
            // overlaps the scatter arithmetic (used only if the particle survives)
            const MatPre mpre = refresh_begin(P.xs, e2);
#endif
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
            if (kVar && kill && ph.roulette && !(e < ph.e_min)) {
              // Russian roulette (R32): survive with probability w / w_s at weight w_s
              const U64x2 r3 = threefry2x64_20((uint64_t)ctr, 0, pid_of(i), P.seed);
              ctr += 1u;
              if (u01(r3.a) < w / ph.w_roul) {
                fsum(SF_ROULETTE, ph.w_roul - w);
                w = ph.w_roul;
                kill = false;
              }
            }
            if (kill) {
              flush();
              fsum(SF_KILLED_E, w * e);
              fsum(SF_KILLED_W, w);
              cnt(SU_KILLED, 1u);
              outcome = 2;
            } else {
              exn = __ldg(ex + cx + (ox > 0.0 ? 1 : 0));
              eyn = __ldg(ey + cy + (oy > 0.0 ? 1 : 0));
              dcen = tcen * speed(e, ph);
              if constexpr (kXsWalk) {
                uint32_t nr = 0;
                m = refresh_xs_walk(P.xs, ph, e, nr, bin_s, bin_a);
                if (nr) cnt(SU_XS_RANGE, nr);
              } else {
#if NT_XS_EARLY
                if (mpre.nr) cnt(SU_XS_RANGE, mpre.nr);
                m = refresh_end(P.xs, ph, mpre);
#else
                m = xs_refresh(e);
#endif
              }
              iox = 1.0 / ox;
              ioy = 1.0 / oy;
              if (ox == 0.0) { exn = d_inf(); iox = d_inf(); }
              if (oy == 0.0) { eyn = d_inf(); ioy = d_inf(); }
              mfp = -log(mfp_u);
            }
          }
        } else if (df < ds) {
          // ---- facet: one code path for both axes (no X/Y divergence) ----
          acc += ((w * df) * sig) * m.H;
          mfp = clamp0(mfp - df * sig);
          dcen = dcen - df;
          const double xm = x + df * ox, ym = y + df * oy;
          x = ax ? exn : xm;                          // snap the crossed coordinate
          y = ax ? ym : eyn;
          flush();                                    // deposit of the cell being left
          const int32_t c = ax ? cx : cy;
          const bool pos = ax ? (ox > 0.0) : (oy > 0.0);
          // step, and reflect if the stepped index leaves [0, n): one unsigned compare
          const int32_t cs = c + (pos ? 1 : -1);
          const bool refl = (uint32_t)cs >= (uint32_t)(ax ? nx : ny);   // reflective
          const int32_t c2 = refl ? c : cs;
          cx = ax ? c2 : cx;
          cy = ax ? cy : c2;
          if (refl) {                               // rare: a branch beats 8 selects
            if (kVar && ph.vacuum) {                // vacuum boundary (R30): escape
              cnt(SU_ESCAPED, 1u);
              fsum(SF_ESCAPED_E, w * e);
              fsum(SF_ESCAPED_W, w);
              outcome = 3;
            } else if (ax) {
              ox = -ox;
              iox = -iox;
            } else {
              oy = -oy;
              ioy = -ioy;
            }
          }
          // next edge on the crossed axis and the new cell's density: two independent loads,
          // consumed at the next event
          const bool pos2 = refl ? !pos : pos;
          const int32_t ke = pos2 ? c2 + 1 : c2;
          if (ax) exn = __ldg(ex + ke); else eyn = __ldg(ey + ke);
          cidx = cidx_of(cx, cy);
          draw = dload(cx, cy, cidx);                 // new cell's density
          nf += 1u;
          if constexpr (kSlab) {
            // entered the neighbour's slab: the facet is done, the neighbour continues
            if (ax && !refl && outside_slab(cx)) park_to(4u, P.out_q, P.out_count);
          }
        } else {
          // ---- census ----
          acc += ((w * ds) * sig) * m.H;
          x = x + ds * ox;
          y = y + ds * oy;
          const double nm = mfp - ds * sig;
          mfp = nm > 0.0 ? nm : 0.0;
          flush();
          cnt(SU_CENSUS, 1u);
          fsum(SF_CENSUS_E, w * e);
          fsum(SF_CENSUS_W, w);
          outcome = 1;
        }

        if (outcome != 0) {
          if (!(isfinite(x) && isfinite(y) && isfinite(e) && isfinite(w)))
            cnt(SU_NONFINITE, 1u);
          st_stream(PP(x, i), x, pol_stream);
          st_stream(PP(y, i), y, pol_stream);
          st_stream(PP(ox, i), ox, pol_stream);
          st_stream(PP(oy, i), oy, pol_stream);
          st_stream(PP(e, i), e, pol_stream);
          st_stream(PP(w, i), w, pol_stream);
          st_stream(PP(mfp, i), mfp, pol_stream);
          red_add_f64(PP(dep, i), dstep);           // the particle's ledgers: no load here
          st_stream(PP(cx, i), cx, pol_stream);
          st_stream(PP(cy, i), cy, pol_stream);
          st_stream(PP(ctr, i), ctr, pol_stream);
          red_add_u32(PP(nfac, i), nf);
          red_add_u32(PP(ncol, i), nc);
          if (outcome == 1) {
            red_add_u32(PP(ncen, i), 1u);
            if (res) (*PP(status, i)) = 1u;              // was parked (2)
          } else {
            (*PP(status, i)) = 0u;
          }
          cnt(SU_FACETS, nf);
          cnt(SU_COLLISIONS, nc);
          fsum(SF_TALLY, dstep);
          active = false;
        }
    };
    // Each lane runs up to kInnerEvents events between two warp votes; the per-lane bound
    // lim = min(events so far + kInnerEvents, max_events) also enforces the event cap (R27),
    // whose kill is handled by event(true) once the bound is the cap.
    // (with the resume ring's cheap refills, 4-64 events per vote in the resumed phase were
    // measured too: all slower, csp +0.9-2.6%, split +1-9%; profiles/ab/r02_ab20_resume_ring.txt)
    constexpr uint32_t inner = (uint32_t)kInnerEvents;
    auto run_lane = [&]() __attribute__((always_inline)) {
      if (active) {
        const uint32_t ne = nf + nc;
        const uint32_t lim =
            (ne < max_ev && max_ev - ne > inner) ? ne + inner : max_ev;
        while (nf + nc < lim) {
          event(false);
          if (!active) break;
        }
        if (active && nf + nc >= max_ev) event(true);
      }
    };
    if (kFused && consumer) {
      // refill as soon as enough lanes can take a parked particle
      for (;;) {
        run_lane();
        if (__popc(__ballot_sync(kFull, !active && !fin)) >= P.refill_min || !__any_sync(kFull, active))
          break;
      }
    } else if (!exhausted) {
      for (;;) {
        run_lane();
        if (__popc(__ballot_sync(kFull, !active)) >= P.refill_min) break;
      }
    } else {
      for (;;) {
        run_lane();
        if (!__any_sync(kFull, active)) break;
      }
    }
  }
  // ---- CTA reduction of the statistics, one atomic per statistic per CTA ----
  fsum(SF_ABSORBED_W, s_wabs[t]);
  __syncthreads();
  if constexpr (kTally == 3) {        // merge the privatised window: one RED per touched cell
    for (int k = t; k < P.hot_nx * P.hot_ny; k += kHistoryBlock) {
      const double v = s_hot[k];
      if (v != 0.0) {
        const int32_t hx = k % P.hot_nx, hy = k / P.hot_nx;
        red_add_hint(P.mesh.tally + cidx_of(P.hot_x0 + hx, P.hot_y0 + hy), v, pol_keep);
      }
    }
  }
  const int lane2 = t & 31;
  for (int k = wid; k < SU_COUNT + SF_COUNT; k += kWarps) {
    if (k < SU_COUNT) {
      unsigned long long v = lane2 < kWarps ? s_u[lane2][k] : 0u;
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
      if (lane2 == 0 && v != 0) atomicAdd(P.stats_u + k, v);
    } else {
      const int kf = k - SU_COUNT;
      double v = 0.0;
      for (int j = lane2; j < kHistoryBlock; j += 32)
#if NT_SMEM_FSUM
        v += s_f[kf][j];
#else
        v += P.slot_f[(int64_t)blockIdx.x * kHistoryBlock + j + kf * sstride];
#endif
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
      if (lane2 == 0 && v != 0.0) atomicAdd(P.stats_f + kf, v);
    }
  }
}

#undef PP

// Instantiations: deterministic/production x density format x layout x block map x physics
// variants (kVar: the code paths of DESIGN.md R30-R32, compiled only into the kernels used
// when a variant is switched on, so the default kernels carry none of it); the u8 +
// block-map kernels also come with the cached-bin linear XS walk (xs_search 2), and the
// production ones with a 72-register cap (7 CTAs per SM, ctas_per_sm = 7; the default is 80
// registers, 6 CTAs per SM) and with warp-aggregated flushes (tally_mode 1).
#ifndef NT_HIST_MINB
#define NT_HIST_MINB 6   // resident CTAs per SM the default kernel is compiled for (A/B ab11)
#endif
template <bool kDet, bool kTiled, bool kVar>
static void* history_fn(int fmt, bool blk, int minb, int tally, int xs, bool aos, bool fused,
                        bool q = false) {
  if (fmt == kDensU8) {
    if (!blk) return (void*)history_kernel<kDet, kDensU8, kTiled, false, 6, 0, false, kVar, false>;
    if constexpr (!kVar) {
      if (aos) return (void*)history_kernel<kDet, kDensU8, kTiled, true, NT_HIST_MINB, 0, false, false, false, true>;
      if (xs == 2) return (void*)history_kernel<kDet, kDensU8, kTiled, true, 6, 0, true, false, false>;
      if constexpr (!kDet) {
        if (minb >= 7) return (void*)history_kernel<kDet, kDensU8, kTiled, true, 7, 0, false, false, false>;
        if (tally == 1) return (void*)history_kernel<kDet, kDensU8, kTiled, true, 6, 1, false, false, false>;
        if (tally == 2) return (void*)history_kernel<kDet, kDensU8, kTiled, true, 6, 2, false, false, false>;
        if (tally == 3) return (void*)history_kernel<kDet, kDensU8, kTiled, true, 6, 3, false, false, false>;
        // resume ring (resume_prefetch): the default kernel with record parking
        if (q) return (void*)history_kernel<kDet, kDensU8, kTiled, true, NT_HIST_MINB, 0, false, false, false, false, false, true>;
        // fused phases: the default kernel otherwise (nt_api.cu history_fused mirrors this)
        if (fused) return (void*)history_kernel<kDet, kDensU8, kTiled, true, NT_HIST_MINB, 0, false, false, false, false, true>;
      }
    }
    return (void*)history_kernel<kDet, kDensU8, kTiled, true, NT_HIST_MINB, 0, false, kVar, false>;
  }
  if (fmt == kDensU16) return (void*)history_kernel<kDet, kDensU16, kTiled, false, 6, 0, false, kVar, false>;
  return (void*)history_kernel<kDet, kDensF64, kTiled, false, 6, 0, false, kVar, false>;
}

// x-slab decomposition kernels: production tally, physics variants compiled in.
template <bool kTiled>
static void* history_slab_fn(int fmt, bool blk) {
  if (fmt == kDensU8)
    return blk ? (void*)history_kernel<false, kDensU8, kTiled, true, 6, 0, false, true, true>
               : (void*)history_kernel<false, kDensU8, kTiled, false, 6, 0, false, true, true>;
  if (fmt == kDensU16) return (void*)history_kernel<false, kDensU16, kTiled, false, 6, 0, false, true, true>;
  return (void*)history_kernel<false, kDensF64, kTiled, false, 6, 0, false, true, true>;
}

template <bool kVar>
static void* history_select_v(bool det, int fmt, bool tiled, bool blk, int minb, int tally, int xs,
                              bool aos, bool fused, bool q) {
  if (det) return tiled ? history_fn<true, true, kVar>(fmt, blk, minb, tally, xs, aos, false)
                        : history_fn<true, false, kVar>(fmt, blk, minb, tally, xs, aos, false);
  return tiled ? history_fn<false, true, kVar>(fmt, blk, minb, tally, xs, aos, fused, q)
               : history_fn<false, false, kVar>(fmt, blk, minb, tally, xs, aos, fused, q);
}

static void* history_select(bool det, int fmt, bool tiled, bool blk, int minb, int tally, int xs,
                            bool var, bool slab = false, bool aos = false, bool fused = false,
                            bool q = false) {
  if (slab) return tiled ? history_slab_fn<true>(fmt, blk) : history_slab_fn<false>(fmt, blk);
  return var ? history_select_v<true>(det, fmt, tiled, blk, minb, tally, xs, false, false, false)
             : history_select_v<false>(det, fmt, tiled, blk, minb, tally, xs, aos, fused, q);
}

void launch_history(const TrackParams& tp, bool det, int grid, int minb, int tally_mode,
                    int xs_search, bool slab, cudaStream_t s) {
  const bool var = tp.ph.vacuum || tp.ph.analog || tp.ph.roulette;
  const bool q = tp.park_rec != nullptr;     // resume_prefetch (the host checked the conditions)
  void* fn = history_select(det, tp.mesh.fmt, tp.mesh.tiled != 0, tp.mesh.blk != nullptr, minb,
                            tally_mode, xs_search, var, slab, tp.aos != nullptr, tp.park_taken != nullptr, q);
  void* args[] = {const_cast<TrackParams*>(&tp)};
  // the resume phase of a kQ kernel holds the record ring in dynamic shared memory (phase 1
  // launches without it, keeping the larger L1 for the density and edge gathers)
  const size_t dyn = (q && tp.resume_q != nullptr) ? (size_t)kRingCtaBytes : 0;
  cudaLaunchKernel(fn, dim3(grid), dim3(kHistoryBlock), args, dyn, s);
}

int history_ring_ctas_per_sm(bool tiled) {
  int n = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(
      &n, history_select(false, kDensU8, tiled, true, 6, 0, 0, false, false, false, false, true),
      kHistoryBlock, kRingCtaBytes);
  return n;
}

int history_max_ctas_per_sm(bool det, int fmt, bool tiled, bool blk, int minb, int tally) {
  int n = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&n, history_select(det, fmt, tiled, blk, minb, tally, 0, false),
                                                kHistoryBlock, 0);
  return n;
}

// ---------------------------------------------------------------------------------------
// Deterministic tally: records sorted by (cell, particle, sequence); one thread per cell
// segment adds the segment serially onto the running tally -- the oracle's order.
__global__ void det_apply_kernel(const unsigned long long* __restrict__ keys,
                                 const double* __restrict__ vals, unsigned long long n,
                                 double* __restrict__ tally) {
  for (unsigned long long j = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x; j < n;
       j += (unsigned long long)gridDim.x * blockDim.x) {
    const unsigned long long cell = keys[j] >> 40;
    if (j != 0 && (keys[j - 1] >> 40) == cell) continue;
    double s = tally[cell];
    for (unsigned long long k = j; k < n && (keys[k] >> 40) == cell; ++k) s += vals[k];
    tally[cell] = s;
  }
}

void launch_det_apply(const unsigned long long* keys, const double* vals,
                      unsigned long long n, double* tally, cudaStream_t s) {
  if (n == 0) return;
  unsigned long long blocks = (n + 255) / 256;
  if (blocks > 65535ull * 8) blocks = 65535ull * 8;
  det_apply_kernel<<<(unsigned)blocks, 256, 0, s>>>(keys, vals, n, tally);
}

cudaError_t sort_pairs(void* temp, size_t& temp_bytes, const unsigned long long* kin,
                       unsigned long long* kout, const double* vin, double* vout,
                       unsigned long long n, int end_bit, cudaStream_t s) {
  return cub::DeviceRadixSort::SortPairs(temp, temp_bytes, kin, kout, vin, vout,
                                         (int64_t)n, 0, end_bit, s);
}

// ---------------------------------------------------------------------------------------
// x-slab decomposition: emigrant records.
__global__ void slab_pack_kernel(const __grid_constant__ TrackParams P, const int32_t* __restrict__ out_q,
                                 int64_t n, SlabRec* __restrict__ dst, unsigned long long* cnt) {
  const int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (k >= n) return;
  const int32_t i = out_q[k];
  const bool left = P.p.cx[i] < P.slab_lo;
  const unsigned long long slot = atomicAdd(cnt + (left ? 0 : 1), 1ull);
  SlabRec& r = dst[left ? (int64_t)slot : n - 1 - (int64_t)slot];
  r.gid = P.p.gid[i];
  r.x = P.p.x[i]; r.y = P.p.y[i]; r.ox = P.p.ox[i]; r.oy = P.p.oy[i];
  r.e = P.p.e[i]; r.w = P.p.w[i]; r.mfp = P.p.mfp[i];
  r.dcen = P.p.dcen[i]; r.acc = P.p.acc[i]; r.dstep = P.p.dstep[i]; r.dep = P.p.dep[i];
  r.cx = P.p.cx[i]; r.cy = P.p.cy[i]; r.ctr = P.p.ctr[i];
  // (x-slabs run the production tally only: the flush sequence is not kept -- compute-
  // sanitizer initcheck flagged the read of the never-written column)
  r.nf = P.p.nf_s[i]; r.nc = P.p.nc_s[i]; r.seq = 0u;
  r.nfac = P.p.nfac[i]; r.ncol = P.p.ncol[i]; r.ncen = P.p.ncen[i]; r.pad = 0u;
}

__global__ void slab_unpack_kernel(const Soa p, const SlabRec* __restrict__ src, int64_t n,
                                   const int32_t* __restrict__ free_slots, int64_t n_free,
                                   int64_t base, int32_t* __restrict__ arr_q) {
  const int64_t k = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (k >= n) return;
  const SlabRec& r = src[k];
  const int64_t i = k < n_free ? (int64_t)free_slots[k] : base + (k - n_free);
  p.gid[i] = r.gid;
  p.x[i] = r.x; p.y[i] = r.y; p.ox[i] = r.ox; p.oy[i] = r.oy;
  p.e[i] = r.e; p.w[i] = r.w; p.mfp[i] = r.mfp;
  p.dcen[i] = r.dcen; p.acc[i] = r.acc; p.dstep[i] = r.dstep; p.dep[i] = r.dep;
  p.cx[i] = r.cx; p.cy[i] = r.cy; p.ctr[i] = r.ctr;
  p.nf_s[i] = r.nf; p.nc_s[i] = r.nc; p.seq_s[i] = r.seq;
  p.nfac[i] = r.nfac; p.ncol[i] = r.ncol; p.ncen[i] = r.ncen;
  p.status[i] = 2u;
  arr_q[k] = (int32_t)i;
}

void launch_slab_pack(const TrackParams& tp, const int32_t* out_q, int64_t n, SlabRec* dst,
                      unsigned long long* cnt, cudaStream_t s) {
  if (n <= 0) return;
  slab_pack_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(tp, out_q, n, dst, cnt);
}

void launch_slab_unpack(const Soa& p, const SlabRec* src, int64_t n, const int32_t* free_slots,
                        int64_t n_free, int64_t base, int32_t* arr_q, cudaStream_t s) {
  if (n <= 0) return;
  slab_unpack_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(p, src, n, free_slots, n_free,
                                                                  base, arr_q);
}

// ---------------------------------------------------------------------------------------
// particle_layout 1 (AoS ablation): the particle store into 128 B records and back.
__global__ void aos_copy_kernel(const Soa p, ParticleAoS* __restrict__ a, int64_t n, int to_aos) {
  const int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (i >= n) return;
  ParticleAoS& r = a[i];
  if (to_aos) {
    r.x = p.x[i]; r.y = p.y[i]; r.ox = p.ox[i]; r.oy = p.oy[i]; r.e = p.e[i]; r.w = p.w[i];
    r.mfp = p.mfp[i]; r.dep = p.dep[i]; r.cx = p.cx[i]; r.cy = p.cy[i]; r.ctr = p.ctr[i];
    r.nfac = p.nfac[i]; r.ncol = p.ncol[i]; r.ncen = p.ncen[i]; r.status = p.status[i];
  } else {
    p.x[i] = r.x; p.y[i] = r.y; p.ox[i] = r.ox; p.oy[i] = r.oy; p.e[i] = r.e; p.w[i] = r.w;
    p.mfp[i] = r.mfp; p.dep[i] = r.dep; p.cx[i] = r.cx; p.cy[i] = r.cy; p.ctr[i] = r.ctr;
    p.nfac[i] = r.nfac; p.ncol[i] = r.ncol; p.ncen[i] = r.ncen; p.status[i] = r.status;
  }
}

void launch_aos_copy(const Soa& p, ParticleAoS* aos, int64_t n, bool to_aos, cudaStream_t s) {
  if (n <= 0) return;
  aos_copy_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(p, aos, n, to_aos ? 1 : 0);
}

// ---------------------------------------------------------------------------------------
// Step statistics as one f64 vector (the NCCL allreduce and the single D2H read).
__global__ void stats_to_f64_kernel(const unsigned long long* __restrict__ su,
                                    const double* __restrict__ sf, double* __restrict__ out) {
  const int k = threadIdx.x;
  if (k < SU_COUNT) out[k] = (double)su[k];
  else if (k < SU_COUNT + SF_COUNT) out[k] = sf[k - SU_COUNT];
}

void launch_stats_to_f64(const unsigned long long* su, const double* sf, double* out,
                         cudaStream_t s) {
  stats_to_f64_kernel<<<1, 32, 0, s>>>(su, sf, out);
}

// ---------------------------------------------------------------------------------------
// Verification kernels.
__global__ void threefry_debug_kernel(const uint64_t* __restrict__ in, int64_t n,
                                      uint64_t* __restrict__ out) {
  const int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (i >= n) return;
  const U64x2 r = threefry2x64_20(in[4 * i], in[4 * i + 1], in[4 * i + 2], in[4 * i + 3]);
  out[2 * i] = r.a;
  out[2 * i + 1] = r.b;
}

void launch_threefry_debug(const uint64_t* in, int64_t n, uint64_t* out, cudaStream_t s) {
  if (n <= 0) return;
  threefry_debug_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(in, n, out);
}

#if NT_TIMELINE
extern "C" int nt_dev_timeline(unsigned long long* out) {   // [2][8192][3]
  return (int)cudaMemcpyFromSymbol(out, g_tl, sizeof(g_tl));
}
#endif

// ---- cross-section table preparation (nt_load_cross_sections) ----
// interleaved (key, value) pairs [n + 1], the last pair repeated as padding
__global__ void xs_pairs_kernel(const double* __restrict__ k, const double* __restrict__ v,
                                int64_t n, double2* __restrict__ kv) {
  const int64_t j = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (j > n) return;
  const int64_t q = j < n ? j : n - 1;
  kv[j] = make_double2(k[q], v[q]);
}

// bucket index: idx[b] = max{i in [0, n-2] : k[i] <= value with bits base + (b << shift)}
// (+inf past the finite range), b in [0, nb]
__global__ void xs_index_kernel(const double* __restrict__ k, int64_t n, uint64_t base, int shift,
                                int64_t nb, uint32_t* __restrict__ idx) {
  const int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (b > nb) return;
  const uint64_t bits = base + ((uint64_t)b << shift);
  const double v = bits >= 0x7ff0000000000000ull ? __longlong_as_double(0x7ff0000000000000ll)
                                                 : __longlong_as_double((long long)bits);
  int64_t lo = 0, hi = n - 1;                 // k[lo] <= v (k[0] is bucket 0's first value)
  while (hi - lo > 1) {
    const int64_t mid = (lo + hi) >> 1;
    if (k[mid] <= v) lo = mid; else hi = mid;
  }
  idx[b] = (uint32_t)lo;
}

// direct bucket rows: row[3b .. 3b+2] = kv[idx[b] .. idx[b]+2]; *wide != 0 if some bucket
// spans more than one key (then the rows are not used)
__global__ void xs_rows_kernel(const double2* __restrict__ kv, const uint32_t* __restrict__ idx,
                               int64_t nb, double2* __restrict__ row, unsigned int* wide) {
  const int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (b >= nb) return;
  const uint32_t i0 = idx[b];
  if (idx[b + 1] - i0 > 1u) atomicOr(wide, 1u);
  const double2* src = kv + i0;
  row[3 * b] = src[0];
  row[3 * b + 1] = src[1];
  row[3 * b + 2] = src[2];
}

// unionised grid (xs_search 0): per bucket of the union index, each table's three pairs
// (scatter then capture); *wide != 0 if some bucket spans more than one key of a table
__device__ __forceinline__ int64_t xs_bin_of(const double* __restrict__ k, int64_t n, double v) {
  if (!(k[0] <= v)) return 0;                 // below the table: its first bin (e is clamped)
  int64_t lo = 0, hi = n - 1;
  while (hi - lo > 1) {
    const int64_t mid = (lo + hi) >> 1;
    if (k[mid] <= v) lo = mid; else hi = mid;
  }
  return lo;
}
__device__ __forceinline__ double xs_bucket_value(uint64_t base, int shift, int64_t b) {
  const uint64_t bits = base + ((uint64_t)b << shift);
  return bits >= 0x7ff0000000000000ull ? __longlong_as_double(0x7ff0000000000000ll)
                                       : __longlong_as_double((long long)bits);
}
__global__ void xs_urow_kernel(const double* __restrict__ ks, const double2* __restrict__ kvs, int64_t ns,
                               const double* __restrict__ kc, const double2* __restrict__ kvc, int64_t nc,
                               uint64_t base, int shift, int64_t nb, double2* __restrict__ row,
                               unsigned int* wide) {
  const int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (b >= nb) return;
  const double v0 = xs_bucket_value(base, shift, b), v1 = xs_bucket_value(base, shift, b + 1);
  const int64_t s0 = xs_bin_of(ks, ns, v0), s1 = xs_bin_of(ks, ns, v1);
  const int64_t c0 = xs_bin_of(kc, nc, v0), c1 = xs_bin_of(kc, nc, v1);
  if (s1 - s0 > 1 || c1 - c0 > 1) atomicOr(wide, 1u);
  for (int j = 0; j < 3; ++j) {
    row[6 * b + j] = kvs[s0 + j];
    row[6 * b + 3 + j] = kvc[c0 + j];
  }
}

void launch_xs_urows(const double* ks, const double2* kvs, int64_t ns, const double* kc,
                     const double2* kvc, int64_t nc, uint64_t base, int shift, int64_t nb,
                     double2* row, unsigned int* wide, cudaStream_t s) {
  if (nb <= 0) return;
  xs_urow_kernel<<<(unsigned)((nb + 255) / 256), 256, 0, s>>>(ks, kvs, ns, kc, kvc, nc, base, shift,
                                                               nb, row, wide);
}

void launch_xs_prepare(const double* k, const double* v, int64_t n, uint64_t base, int shift,
                       int64_t nb, bool rows, uint32_t* idx, double2* kv, double2* row,
                       unsigned int* wide, cudaStream_t s) {
  xs_pairs_kernel<<<(unsigned)((n + 256) / 256), 256, 0, s>>>(k, v, n, kv);
  if (nb <= 0) return;
  xs_index_kernel<<<(unsigned)((nb + 256) / 256), 256, 0, s>>>(k, n, base, shift, nb, idx);
  if (rows) xs_rows_kernel<<<(unsigned)((nb + 255) / 256), 256, 0, s>>>(kv, idx, nb, row, wide);
}

__global__ void xs_debug_kernel(const Tables T, const double* __restrict__ e, int64_t n,
                                double* __restrict__ os, double* __restrict__ oa) {
  const int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  if (i >= n) return;
  uint32_t dummy = 0;
  const double es = clamp_count(e[i], T.s, dummy);
  const double ea = clamp_count(e[i], T.c, dummy);
  if (T.urow != nullptr && es == ea && es < T.ulast) {       // the unionised grid (xs_search 0)
    const uint64_t b = ((uint64_t)__double_as_longlong(es) - T.ubase) >> T.ushift;
    os[i] = xs_urow_lerp(T.urow + 6 * b, es);
    oa[i] = xs_urow_lerp(T.urow + 6 * b + 3, ea);
    return;
  }
  os[i] = xs_lookup(T.s, es);
  oa[i] = xs_lookup(T.c, ea);
}

void launch_xs_debug(const Tables& T, const double* e, int64_t n, double* os, double* oa,
                     cudaStream_t s) {
  if (n <= 0) return;
  xs_debug_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(T, e, n, os, oa);
}

}  // namespace nt
