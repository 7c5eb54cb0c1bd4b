// nt_event.cu -- event-based (Over Events) variant of the tracker, P:358-390 (§V-B).
//
// Listing 2 advances every particle by one event per iteration: compute the time to each
// event, determine the next one, then handle collisions, facets and census in separate
// loops.  Particles are independent, so here every CTA runs that loop on its
// own set of at most kACap active particles -- no grid-wide synchronisation -- and refills
// the set from a global counter whenever a block-size of slots is free (the Over Events
// analogue of the history kernel's refill), so every CTA stays busy until the
// particle range is exhausted.
//
// State.  Over Events cannot keep a history's cached state in registers.  A CTA
// owns kACap particle slots whose state lives in global memory as structure-of-arrays
// columns -- column f of slot s at slots[(cta * kCols + f) * kACap + s].  The
// three event queues hold slot numbers in increasing order, so the warps handling a queue
// read and write runs of consecutive slots: coalesced column accesses, ≈ 15 columns read and
// 8 written per facet.
//
// Iteration.  (1) Refill free slots with new particles (one atomicAdd per refill).  (2) One
// thread per queued event: the collisions, then the facets, then the census events, then
// the new particles' first classification, as one concatenated range so each warp handles
// one event type; every handler classifies its particle's next event into the
// slot's type byte in shared memory.  (3) Compaction: a scan over the slots' type bytes --
// per-thread counts, warp prefix sums with shuffles, a prefix over the warps -- rebuilds the
// three queues and the free list in slot order.
//
// Arithmetic: DESIGN.md §3, identical to the history kernel, so per-particle results match
// it (and the oracle) bit for bit; the next-event distances are recomputed by the handler
// from the same inputs, so the classification and the handling agree exactly.
#include <cstdlib>
#include <cstring>

#include "nt_event.h"

namespace nt {

constexpr int kEvBlock = 256;
#ifndef NT_EV_ACAP
#define NT_EV_ACAP 1024
#endif
#ifndef NT_EV_MINB
#define NT_EV_MINB 4
#endif
constexpr int kACap = NT_EV_ACAP;           // particle slots per CTA
constexpr int kSlotsPerThread = kACap / kEvBlock;
constexpr unsigned kAccBit = 4u;            // type-byte flag: the slot's C_ACC is non-zero

static_assert(kACap % kEvBlock == 0 && kACap / kEvBlock <= 8, "slots per thread");

// slot columns (8-byte words)
enum Col : int {
  C_X = 0, C_Y, C_MFP, C_DCEN, C_ACC, C_DSTEP,   // every event
  C_OX, C_OY, C_IOX, C_IOY,                      // reflections and collisions
  C_W, C_ST, C_H, C_E, C_PA,                     // collisions
  C_CXY,                                         // cell (cx, cy): facets
  C_NFC,                                         // facet and collision counts this step
  C_CTR,                                         // RNG counter, flush sequence
  C_PID,                                         // local particle index
  kCols
};

struct EvCtl {
  unsigned long long counter;   // particles of [lo, hi) handed out to the CTAs
  unsigned int iter;            // most iterations a CTA ran
  unsigned int pad;
};

struct EventState {
  int64_t slot_blocks = 0;
  double* slots = nullptr;  // [grid][kCols][kACap]
  EvCtl* ctl = nullptr;
  double* slot_f = nullptr; // [SF_COUNT][grid * block] per-thread f64 statistic slots
  int64_t slot_cap = 0;
};

struct EvParams {
  TrackParams P;
  double* slots;
  EvCtl* ctl;
};

__device__ __forceinline__ double ev_inf() { return __longlong_as_double(0x7ff0000000000000ll); }

// One particle's state in registers while its event is handled.
struct St {
  double x, y, mfp, dcen, acc, dstep, ox, oy, iox, ioy, w, st, H, e;
  int32_t cx, cy;
  uint32_t nf, nc;
};

template <bool kDet, int kFmt, bool kBlk>
struct EvKernel {
  const TrackParams& P;
  const Phys& ph;
  const double* s_nd;
  const uint8_t* s_blk;
  unsigned long long* s_u;  // per-CTA statistics (shared atomics)
  double* sf;               // this thread's f64 statistic slots, stride sstride
  int64_t sstride;
  uint64_t pol;             // L2 evict_last: tally REDs and density gathers
  double* cols;             // this CTA's slot columns
  int slot;                 // the slot being handled
  const uint8_t* s_type;    // slot type bytes (bit 2: the slot's deposit accumulator is non-zero)

  __device__ double& c(int f) { return cols[f * kACap + slot]; }
  __device__ int2 ci2(int f) { return reinterpret_cast<int2*>(cols + f * kACap)[slot]; }
  __device__ void si2(int f, int2 v) { reinterpret_cast<int2*>(cols + f * kACap)[slot] = v; }

  __device__ void cnt(int k, uint32_t v) { atomicAdd(s_u + k, (unsigned long long)v); }
  __device__ void fsum(int k, double v) { sf[k * sstride] += v; }

  __device__ double nd_of(int32_t cx, int32_t cy) {
    const uint32_t cidx = (uint32_t)cell_index(P.mesh, cx, cy);
    if constexpr (kBlk) return s_nd[dens_load_blk(P.mesh, s_blk, cx, cy, cidx, pol)];
    else if constexpr (kFmt == kDensU8) return s_nd[ldg_u8_hint(P.mesh.rho8 + cidx, pol)];
    else return number_density<kFmt>(P.mesh, P.mesh.nd_tab, cidx, ph.cn);
  }

  // the flush of DESIGN.md §3: production RED or deterministic record
  __device__ void flush(St& s) {
    const int64_t cell = cell_index(P.mesh, s.cx, s.cy);
    if constexpr (kDet) {
      const int32_t i = ci2(C_PID).x;
      int2 cs = ci2(C_CTR);
      const uint32_t seq = (uint32_t)cs.y;
      const unsigned long long rs = atomicAdd(P.rec_count, 1ull);
      if (rs < P.rec_cap) {
        P.rec_key[rs] = ((unsigned long long)cell << 40) |
                        ((unsigned long long)((int64_t)i - P.lo) << 24) |
                        (unsigned long long)(seq & 0xffffffu);
        P.rec_val[rs] = s.acc;
      }
      if (seq >= (1u << 24)) cnt(SU_REC_OVERFLOW, 1u);
      cs.y = (int)(seq + 1u);
      si2(C_CTR, cs);
    } else {
      red_add_hint(P.mesh.tally + cell, s.acc, pol);
    }
    s.dstep += s.acc;
    s.acc = 0.0;
  }

  // A history ended here: write the particle store (census: alive; otherwise dead).
  __device__ void finish(const St& s, uint32_t ctr, bool alive) {
    const int32_t i = ci2(C_PID).x;
    if (!(isfinite(s.x) && isfinite(s.y) && isfinite(s.e) && isfinite(s.w))) cnt(SU_NONFINITE, 1u);
    P.p.x[i] = s.x;
    P.p.y[i] = s.y;
    P.p.ox[i] = s.ox;
    P.p.oy[i] = s.oy;
    P.p.e[i] = s.e;
    P.p.w[i] = s.w;
    P.p.mfp[i] = s.mfp;
    P.p.dep[i] += s.dstep;
    P.p.cx[i] = s.cx;
    P.p.cy[i] = s.cy;
    P.p.ctr[i] = ctr;
    P.p.nfac[i] += s.nf;
    P.p.ncol[i] += s.nc;
    if (alive) P.p.ncen[i] += 1u; else P.p.status[i] = 0u;
    cnt(SU_FACETS, s.nf);
    cnt(SU_COLLISIONS, s.nc);
    fsum(SF_TALLY, s.dstep);
  }

  // Distances to the three events.
  struct Dist { double df, dc, ds; bool ax; };
  __device__ Dist dist(const St& s, double nd) {
    const double exn = __ldg(P.mesh.ex + s.cx + (s.ox > 0.0 ? 1 : 0));
    const double eyn = __ldg(P.mesh.ey + s.cy + (s.oy > 0.0 ? 1 : 0));
    const double sig = nd * s.st;
    double tx = (exn - s.x) * s.iox;
    tx = tx < 0.0 ? 0.0 : tx;
    tx = s.ox != 0.0 ? tx : ev_inf();          // no crossing along an axis with ω = 0
    double ty = (eyn - s.y) * s.ioy;
    ty = ty < 0.0 ? 0.0 : ty;
    ty = s.oy != 0.0 ? ty : ev_inf();
    Dist d;
    d.ax = tx < ty;
    d.df = d.ax ? tx : ty;
    d.ds = s.dcen;
    d.dc = sig > 0.0 ? s.mfp / sig : ev_inf();
    return d;
  }

  // determine_next_event (Listing 2): 0 collision, 1 facet, 2 census; the event cap
  // (R27) ends the history here (3).
  __device__ int classify(St& s) {
    if ((int64_t)(s.nf + s.nc) >= P.max_events) {
      cnt(SU_EVENT_CAP, 1u);
      flush(s);
      cnt(SU_KILLED, 1u);
      fsum(SF_KILLED_E, s.w * s.e);
      fsum(SF_KILLED_W, s.w);
      finish(s, (uint32_t)ci2(C_CTR).x, false);
      return 3;
    }
    const Dist d = dist(s, nd_of(s.cx, s.cy));
    const int ab = s.acc != 0.0 ? (int)kAccBit : 0;   // the slot's type bit for load_common
    if (d.dc < d.df && d.dc < d.ds) return 0 | ab;
    return (d.df < d.ds ? 1 : 2) | ab;
  }

  __device__ void load_common(St& s) {
    s.x = c(C_X); s.y = c(C_Y); s.mfp = c(C_MFP); s.dcen = c(C_DCEN);
    s.acc = (s_type[slot] & kAccBit) ? c(C_ACC) : 0.0;   // most events start with acc == 0
    s.dstep = c(C_DSTEP);
    s.ox = c(C_OX); s.oy = c(C_OY); s.iox = c(C_IOX); s.ioy = c(C_IOY);
    s.w = c(C_W); s.st = c(C_ST); s.H = c(C_H);
    const int2 cxy = ci2(C_CXY);
    s.cx = cxy.x; s.cy = cxy.y;
    const int2 nfc = ci2(C_NFC);
    s.nf = (uint32_t)nfc.x; s.nc = (uint32_t)nfc.y;
  }
  __device__ void store_moved(const St& s) {     // what every event changes
    c(C_X) = s.x; c(C_Y) = s.y; c(C_MFP) = s.mfp; c(C_DCEN) = s.dcen;
    if (s.acc != 0.0) c(C_ACC) = s.acc;          // read back only while the type bit is set
    c(C_DSTEP) = s.dstep;
    si2(C_CXY, make_int2(s.cx, s.cy));
    si2(C_NFC, make_int2((int)s.nf, (int)s.nc));
  }

  // ---- collision ----
  __device__ int collision() {
    St s;
    load_common(s);
    s.e = c(C_E);
    const double pa = c(C_PA);
    int2 cs = ci2(C_CTR);
    uint32_t ctr = (uint32_t)cs.x;
    const int32_t i = ci2(C_PID).x;
    const double nd = nd_of(s.cx, s.cy);
    const Dist dd = dist(s, nd);
    const double d = dd.dc;
    const double sig = nd * s.st;
    s.acc += ((s.w * d) * sig) * s.H;
    s.x = s.x + d * s.ox;
    s.y = s.y + d * s.oy;
    s.dcen = s.dcen - d;
    const uint64_t pid = (uint64_t)(P.first_id + i);
    const U64x2 r = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
    ctr += 1u;
    s.nc += 1u;
    double mfp_u = u01(r.b);
    bool absorbed = false;
    const double w0 = s.w;
    if (!ph.analog) {                           // implicit capture
      s.w = s.w * (1.0 - pa);
      fsum(SF_ABSORBED_W, w0 - s.w);
    } else if (u01(r.b) < pa) {                // sampled absorption (R31)
      absorbed = true;
    } else {                                    // scatter: n_mfp from the next counter
      const U64x2 r2 = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
      ctr += 1u;
      mfp_u = u01(r2.a);
    }
    if (absorbed) {
      flush(s);
      fsum(SF_ABSORBED_W, s.w);
      fsum(SF_ABSORBED_E, s.w * s.e);
      cnt(SU_ABSORBED, 1u);
      finish(s, ctr, false);
      return 3;
    }
    const double e = s.e;
    const double mu = 1.0 - 2.0 * u01(r.a);
    const double e2 = e * (((ph.AA + ph.twoA * mu) + 1.0) / ph.Ap1sq);
    const double ct = 0.5 * (ph.Ap1 * sqrt(e2 / e) - ph.Am1 * sqrt(e / e2));
    const double sgn = (r.a & 1ull) ? -1.0 : 1.0;
    const double q = 1.0 - ct * ct;
    const double stt = sgn * sqrt(q > 0.0 ? q : 0.0);
    const double nox = s.ox * ct - s.oy * stt;
    const double noy = s.ox * stt + s.oy * ct;
    s.ox = nox;
    s.oy = noy;
    const double tcen = s.dcen / speed(e, ph);
    s.e = e2;
    bool kill = s.e < ph.e_min || s.w < ph.w_min;   // termination
    if (kill && ph.roulette && !(s.e < ph.e_min)) {
      // Russian roulette (R32): survive with probability w / w_s at weight w_s
      const U64x2 r3 = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
      ctr += 1u;
      if (u01(r3.a) < s.w / ph.w_roul) {
        fsum(SF_ROULETTE, ph.w_roul - s.w);
        s.w = ph.w_roul;
        kill = false;
      }
    }
    if (kill) {
      flush(s);
      fsum(SF_KILLED_E, s.w * s.e);
      fsum(SF_KILLED_W, s.w);
      cnt(SU_KILLED, 1u);
      finish(s, ctr, false);
      return 3;
    }
    s.dcen = tcen * speed(s.e, ph);
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, s.e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    s.st = m.st;
    s.H = m.H;
    s.iox = 1.0 / s.ox;
    s.ioy = 1.0 / s.oy;
    s.mfp = -log(mfp_u);
    store_moved(s);
    c(C_OX) = s.ox; c(C_OY) = s.oy; c(C_IOX) = s.iox; c(C_IOY) = s.ioy;
    c(C_W) = s.w; c(C_ST) = s.st; c(C_H) = s.H; c(C_E) = s.e; c(C_PA) = m.pa;
    cs = ci2(C_CTR);                            // (the flush sequence is unchanged here)
    cs.x = (int)ctr;
    si2(C_CTR, cs);
    return classify(s);
  }

  // ---- facet ----
  __device__ int facet() {
    St s;
    load_common(s);
    const double nd = nd_of(s.cx, s.cy);
    const Dist dd = dist(s, nd);
    const double d = dd.df;
    const bool ax = dd.ax;
    const double sig = nd * s.st;
    s.acc += ((s.w * d) * sig) * s.H;
    const double nm = s.mfp - d * sig;
    s.mfp = nm > 0.0 ? nm : 0.0;
    s.dcen = s.dcen - d;
    const double xm = s.x + d * s.ox, ym = s.y + d * s.oy;
    const bool pos = ax ? (s.ox > 0.0) : (s.oy > 0.0);
    const int32_t c0 = ax ? s.cx : s.cy;
    // snap the crossed coordinate onto the edge being crossed
    const double edge = ax ? __ldg(P.mesh.ex + c0 + (pos ? 1 : 0)) : __ldg(P.mesh.ey + c0 + (pos ? 1 : 0));
    s.x = ax ? edge : xm;
    s.y = ax ? ym : edge;
    flush(s);
    const int32_t last = (ax ? P.mesh.nx : P.mesh.ny) - 1;
    const bool refl = pos ? (c0 == last) : (c0 == 0);
    s.nf += 1u;
    if (refl && ph.vacuum) {
      // vacuum boundary (R30): the facet ends the history (escape)
      s.e = c(C_E);
      cnt(SU_ESCAPED, 1u);
      fsum(SF_ESCAPED_E, s.w * s.e);
      fsum(SF_ESCAPED_W, s.w);
      finish(s, (uint32_t)ci2(C_CTR).x, false);
      return 3;
    }
    const int32_t c2 = refl ? c0 : (pos ? c0 + 1 : c0 - 1);
    if (ax) s.cx = c2; else s.cy = c2;
    if (refl) {
      if (ax) {
        s.ox = -s.ox; s.iox = -s.iox;
        c(C_OX) = s.ox; c(C_IOX) = s.iox;
      } else {
        s.oy = -s.oy; s.ioy = -s.ioy;
        c(C_OY) = s.oy; c(C_IOY) = s.ioy;
      }
    }
    store_moved(s);
    if ((int64_t)(s.nf + s.nc) >= P.max_events) s.e = c(C_E);   // the cap's kill needs E
    // the new cell's density is gathered by classify
    return classify(s);
  }

  // ---- census ----
  __device__ void census() {
    St s;
    load_common(s);
    s.e = c(C_E);
    const double d = s.dcen;
    const double sig = nd_of(s.cx, s.cy) * s.st;
    s.acc += ((s.w * d) * sig) * s.H;
    s.x = s.x + d * s.ox;
    s.y = s.y + d * s.oy;
    const double nm = s.mfp - d * sig;
    s.mfp = nm > 0.0 ? nm : 0.0;
    flush(s);
    cnt(SU_CENSUS, 1u);
    fsum(SF_CENSUS_E, s.w * s.e);
    fsum(SF_CENSUS_W, s.w);
    finish(s, (uint32_t)ci2(C_CTR).x, true);
  }

  // ---- a new particle: its slot state and first event ----
  __device__ int birth(int32_t i) {
    if (P.p.status[i] != 1u) return 3;
    St s;
    s.x = P.p.x[i];
    s.y = P.p.y[i];
    s.ox = P.p.ox[i];
    s.oy = P.p.oy[i];
    s.w = P.p.w[i];
    s.mfp = P.p.mfp[i];
    s.cx = P.p.cx[i];
    s.cy = P.p.cy[i];
    s.e = P.p.e[i];
    const uint32_t ctr = P.p.ctr[i];
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, s.e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    s.st = m.st;
    s.H = m.H;
    s.dcen = speed(s.e, ph) * P.dt;
    s.iox = 1.0 / s.ox;
    s.ioy = 1.0 / s.oy;
    s.acc = 0.0;
    s.dstep = 0.0;
    s.nf = 0u;
    s.nc = 0u;
    cnt(SU_ALIVE, 1u);
    store_moved(s);
    c(C_OX) = s.ox; c(C_OY) = s.oy; c(C_IOX) = s.iox; c(C_IOY) = s.ioy;
    c(C_W) = s.w; c(C_ST) = s.st; c(C_H) = s.H; c(C_E) = s.e; c(C_PA) = m.pa;
    si2(C_CTR, make_int2((int)ctr, 0));
    si2(C_PID, make_int2(i, 0));
    return classify(s);
  }
};

template <bool kDet, int kFmt, bool kBlk>
__global__ void __launch_bounds__(kEvBlock, NT_EV_MINB) ev_loop_kernel(const __grid_constant__ EvParams E) {
  const TrackParams& P = E.P;
  __shared__ unsigned long long s_u[SU_COUNT];
  __shared__ double s_nd[kFmt == kDensU8 ? 256 : 1];
  __shared__ __align__(16) uint8_t s_blk[kBlk ? kBlkMax : 1];
  __shared__ uint8_t s_type[kACap];            // next event of each slot; 3 = free
  __shared__ uint16_t s_q[4][kACap];           // collision, facet, census queues; free list
  __shared__ unsigned s_n[4];                  // their lengths
  __shared__ unsigned s_wsum[kEvBlock / 32][4];
  __shared__ unsigned s_nnew;                  // particles fetched for this iteration
  __shared__ unsigned long long s_newbase;     // their first position in [lo, hi)
  __shared__ int s_exhausted;
  const int t = threadIdx.x;
  const int lane = t & 31, wid = t >> 5;
  const int bidx = (int)blockIdx.x;
  const int64_t gt = (int64_t)bidx * kEvBlock + t;
  const int64_t sstride = (int64_t)gridDim.x * kEvBlock;
  if (t < SU_COUNT) s_u[t] = 0u;
  for (int k = t; k < kACap; k += kEvBlock) {
    s_type[k] = 3u;
    s_q[3][k] = (uint16_t)k;
  }
  if (t == 0) {
    s_n[0] = s_n[1] = s_n[2] = 0u;
    s_n[3] = kACap;
    s_exhausted = 0;
  }
#pragma unroll
  for (int k = 0; k < SF_COUNT; ++k) P.slot_f[gt + k * sstride] = 0.0;
  if constexpr (kFmt == kDensU8) {
    for (int k = t; k < 256; k += kEvBlock) s_nd[k] = k < P.mesh.ncodes ? P.mesh.nd_tab[k] : 0.0;
    if constexpr (kBlk) {
      const uint4* src = reinterpret_cast<const uint4*>(P.mesh.blk);
      for (int k = t; k < (P.mesh.nblk + 15) / 16; k += kEvBlock)
        reinterpret_cast<uint4*>(s_blk)[k] = __ldg(src + k);
    }
  }
  __syncthreads();
  EvKernel<kDet, kFmt, kBlk> K{P, P.ph, s_nd, s_blk, s_u, P.slot_f + gt, sstride,
                              l2_evict_last(), E.slots + (int64_t)bidx * kCols * kACap, 0, s_type};
  const unsigned long long span = (unsigned long long)(P.hi - P.lo);

  // (1) refill: new particles for the free slots once a block-size of them is free (one
  // thread; published by the barrier that follows.  Folding it into the compaction's
  // barriers measured 11% slower: profiles/ab/r01_ab7_event_refill.md)
  auto refill = [&](unsigned nfree) {
    unsigned nnew = 0;
    if (!s_exhausted && (nfree >= (unsigned)kEvBlock || nfree == (unsigned)kACap)) {
      const unsigned long long base = atomicAdd(&E.ctl->counter, (unsigned long long)nfree);
      if (base >= span) {
        s_exhausted = 1;
      } else {
        nnew = (unsigned)(span - base < nfree ? span - base : nfree);
        if (base + nfree >= span) s_exhausted = 1;
        s_newbase = base;
      }
    }
    s_nnew = nnew;
  };
  for (unsigned it = 0;; ++it) {
    if (t == 0) refill(s_n[3]);
    __syncthreads();
    const unsigned n0 = s_n[0], n1 = s_n[1], n2 = s_n[2], nnew = s_nnew;
    const unsigned n012 = n0 + n1 + n2, total = n012 + nnew;
    if (total == 0u) break;                       // no active particle and none left
    const unsigned long long newbase = s_newbase;
    // ---- (2) one event of every active particle (Listing 2), then the new particles ----
    for (unsigned j = t; j < total; j += kEvBlock) {
      int type;
      if (j < n012) {
        const int seg = j < n0 ? 0 : (j < n0 + n1 ? 1 : 2);
        K.slot = s_q[seg][j - (seg == 0 ? 0u : (seg == 1 ? n0 : n0 + n1))];
        if (seg == 0) type = K.collision();
        else if (seg == 1) type = K.facet();
        else { K.census(); type = 3; }
      } else {
        K.slot = s_q[3][j - n012];
        type = K.birth((int32_t)(P.lo + (int64_t)(newbase + (j - n012))));
      }
      s_type[K.slot] = (uint8_t)type;
    }
    __syncthreads();
    // ---- (3) compaction: the queues and the free list in slot order ----
    {
      unsigned long long tys = 0ull;              // this thread's kSlotsPerThread (<= 8) type bytes
      unsigned c01 = 0u, c23 = 0u;                // per-type counts, two 16-bit fields each
#pragma unroll
      for (int k = 0; k < kSlotsPerThread; ++k) {
        const unsigned ty = s_type[t * kSlotsPerThread + k] & 3u;
        tys |= (unsigned long long)ty << (8 * k);
        if (ty < 2u) c01 += 1u << (16 * ty); else c23 += 1u << (16 * (ty - 2u));
      }
      unsigned i01 = c01, i23 = c23;              // inclusive warp scans
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const unsigned a = __shfl_up_sync(kFull, i01, o), b = __shfl_up_sync(kFull, i23, o);
        if (lane >= o) { i01 += a; i23 += b; }
      }
      if (lane == 31) {
        s_wsum[wid][0] = i01 & 0xffffu; s_wsum[wid][1] = i01 >> 16;
        s_wsum[wid][2] = i23 & 0xffffu; s_wsum[wid][3] = i23 >> 16;
      }
      __syncthreads();
      if (t < 4) {
        unsigned run = 0;
#pragma unroll
        for (int w = 0; w < kEvBlock / 32; ++w) {
          const unsigned v = s_wsum[w][t];
          s_wsum[w][t] = run;
          run += v;
        }
        s_n[t] = run;
      }
      __syncthreads();
      unsigned p0 = s_wsum[wid][0] + ((i01 - c01) & 0xffffu);
      unsigned p1 = s_wsum[wid][1] + ((i01 - c01) >> 16);
      unsigned p2 = s_wsum[wid][2] + ((i23 - c23) & 0xffffu);
      unsigned p3 = s_wsum[wid][3] + ((i23 - c23) >> 16);
#pragma unroll
      for (int k = 0; k < kSlotsPerThread; ++k) {
        const unsigned ty = (unsigned)(tys >> (8 * k)) & 0xffu;
        const unsigned p = ty == 0u ? p0++ : (ty == 1u ? p1++ : (ty == 2u ? p2++ : p3++));
        s_q[ty][p] = (uint16_t)(t * kSlotsPerThread + k);
      }
    }
    __syncthreads();
    if (t == 0 && it + 1u > E.ctl->iter) atomicMax(&E.ctl->iter, it + 1u);
  }

  // ---- statistics: one atomic per statistic per CTA ----
  __syncthreads();
  if (t < SU_COUNT && s_u[t]) atomicAdd(P.stats_u + t, s_u[t]);
  for (int k = wid; k < SF_COUNT; k += kEvBlock / 32) {
    double v = 0.0;
    for (int jj = lane; jj < kEvBlock; jj += 32)
      v += P.slot_f[(int64_t)bidx * kEvBlock + jj + k * sstride];
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if (lane == 0 && v != 0.0) atomicAdd(P.stats_f + k, v);
  }
}

// ---------------------------------------------------------------------------------------
static void* ev_fn(bool det, int fmt, bool blk) {
#define NT_EV(D, F, B) return (void*)ev_loop_kernel<D, F, B>
  if (det) {
    if (fmt == kDensU8) { if (blk) NT_EV(true, kDensU8, true); NT_EV(true, kDensU8, false); }
    if (fmt == kDensU16) NT_EV(true, kDensU16, false);
    NT_EV(true, kDensF64, false);
  }
  if (fmt == kDensU8) { if (blk) NT_EV(false, kDensU8, true); NT_EV(false, kDensU8, false); }
  if (fmt == kDensU16) NT_EV(false, kDensU16, false);
  NT_EV(false, kDensF64, false);
#undef NT_EV
}

EventState* event_state_create() { return new EventState(); }

void event_state_destroy(EventState* s) {
  if (!s) return;
  if (s->slots) cudaFree(s->slots);
  if (s->ctl) cudaFree(s->ctl);
  if (s->slot_f) cudaFree(s->slot_f);
  delete s;
}

void event_state_invalidate(EventState* s) { (void)s; }

// One particle range [tp.lo, tp.hi): the persistent per-CTA event loops, statistics into
// tp.stats_*.
nt_status event_run_range(EventState* s, const TrackParams& tp, bool det, int sm_count,
                          cudaStream_t st, uint32_t& launches, std::string& err) {
  const bool blk = tp.mesh.fmt == kDensU8 && tp.mesh.blk != nullptr;
  void* fn = ev_fn(det, tp.mesh.fmt, blk);
  int per_sm = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, fn, kEvBlock, 0);
  if (per_sm < 1) per_sm = 1;
  const int grid = sm_count * per_sm;
  cudaError_t e = cudaSuccess;
  if (!s->ctl) {
    e = device_malloc(reinterpret_cast<void**>(&s->ctl), sizeof(EvCtl));
    if (e != cudaSuccess) { s->ctl = nullptr; err = cudaGetErrorString(e); return NT_ERR_OOM; }
  }
  if (grid > s->slot_blocks) {
    if (s->slots) cudaFree(s->slots);
    s->slots = nullptr;
    s->slot_blocks = 0;
    e = device_malloc(reinterpret_cast<void**>(&s->slots), (size_t)grid * kCols * kACap * 8);
    if (e != cudaSuccess) { s->slots = nullptr; err = cudaGetErrorString(e); return NT_ERR_OOM; }
    s->slot_blocks = grid;
  }
  const int64_t nslot = (int64_t)grid * kEvBlock * SF_COUNT;
  if (nslot > s->slot_cap) {
    if (s->slot_f) cudaFree(s->slot_f);
    s->slot_f = nullptr;
    s->slot_cap = 0;
    e = device_malloc(reinterpret_cast<void**>(&s->slot_f), (size_t)nslot * 8);
    if (e != cudaSuccess) { s->slot_f = nullptr; err = cudaGetErrorString(e); return NT_ERR_OOM; }
    s->slot_cap = nslot;
  }
  EvParams ep;
  ep.P = tp;
  ep.P.slot_f = s->slot_f;
  ep.slots = s->slots;
  ep.ctl = s->ctl;
  e = cudaMemsetAsync(s->ctl, 0, sizeof(EvCtl), st);
  if (e != cudaSuccess) { err = cudaGetErrorString(e); return NT_ERR_CUDA; }
  if (tp.hi > tp.lo) {
    void* args[] = {&ep};
    e = cudaLaunchKernel(fn, dim3(grid), dim3(kEvBlock), args, 0, st);
    ++launches;
    if (e != cudaSuccess) { err = std::string("event loop: ") + cudaGetErrorString(e); return NT_ERR_CUDA; }
  }
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
