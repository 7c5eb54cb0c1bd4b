// nt_event.cu -- event-based (Over Events) variant of the tracker, P:358-390 (§V-B).
//
// Listing 2 advances every particle by one event per iteration: compute the time to each
// event and determine the next one, then handle all collisions, all facets and all census
// events in separate loops.  Here the particle set is split into per-warp sets
// of kWSlots slots, and each warp runs Listing 2 on its own set with warp-level event
// queues: per iteration the warp snapshots its slots' next-event types, and for each type
// in turn (collisions, facets, census, new particles) compacts the slots of that type into
// a queue with one __ballot_sync per slot half and __popc(mask & lanemask_lt) ranks, then
// handles the queue with all lanes on the same event type (converged code, the Over Events
// advantage).  No CTA-wide barrier runs inside the loop: warps proceed
// independently, and a warp refills its free slots from a global counter (one atomicAdd
// per refill) whenever enough are free, so every warp stays busy until the id range is
// exhausted (the load balancing of P:344-348).
//
// State.  Over Events cannot keep a history's cached state in registers across events
// (P:377-383): every handler loads the particle's state, updates it and stores it back.
// On B200 that state lives in shared memory, not HBM: one CTA per SM owns kSlots slots
// whose fields are structure-of-arrays columns in ~190 KB of shared memory,
// so a handler's loads and stores are conflict-free LDS/STS instead of L2 round trips.
// The classification at the end of every handler stores what the next handler needs --
// the event type, its distance, the facet axis and the cell's number density -- so
// nothing is computed or gathered twice (Listing 2's calculate-then-handle split).
//
// Arithmetic: DESIGN.md §3, the same expressions as the history kernel, so per-particle
// results match it (and the oracle) bit for bit.
#include <cstdlib>
#include <cstring>

#include "nt_event.h"

namespace nt {

#ifndef NT_EV_WARPS
#define NT_EV_WARPS 16
#endif
#ifndef NT_EV_REFILL
#define NT_EV_REFILL 16
#endif
constexpr int kEvWarps = NT_EV_WARPS;        // warps per CTA (one CTA per SM)
constexpr int kEvBlock = kEvWarps * 32;
constexpr int kWSlots = 64;                  // slots per warp: two per lane
constexpr int kSlots = kEvWarps * kWSlots;   // slots per CTA
constexpr int kEvRefill = NT_EV_REFILL;      // a warp refills once this many slots are free

// event types (low 3 bits of a slot's type byte); bit 3: the facet crosses an X edge
enum : uint32_t { T_COLL = 0, T_FACET = 1, T_CENSUS = 2, T_BIRTH = 3, T_FREE = 4, T_AXBIT = 8 };

// f64 slot columns
enum Col8 : int {
  C_X = 0, C_Y, C_OX, C_OY, C_IOX, C_IOY, C_EXN, C_EYN, C_MFP, C_DCEN, C_ACC, C_DSTEP,
  C_W, C_E, C_ST, C_H, C_PA, C_ND, C_D, kCol8
};
// i32 slot columns
enum Col4 : int { C_CX = 0, C_CY, C_NF, C_NC, C_CTR, C_SEQ, C_PID, kCol4 };

constexpr size_t kSmemCols = (size_t)kSlots * (kCol8 * 8 + kCol4 * 4);
constexpr size_t ev_smem_bytes(bool blk) {
  return kSmemCols + 2 * (size_t)kSlots /* types, per-warp queues */ + (blk ? (size_t)kBlkMax : 0);
}

struct EvCtl {
  unsigned long long counter;   // particles of [lo, hi) handed out to the warps
  unsigned int iter;            // most iterations a warp ran
  unsigned int pad;
};

struct EventState {
  EvCtl* ctl = nullptr;
  double* slot_f = nullptr;     // [SF_COUNT][grid * block] per-thread f64 statistic slots
  int64_t slot_cap = 0;
};

struct EvParams {
  TrackParams P;
  EvCtl* ctl;
};

__device__ __forceinline__ double ev_inf() { return __longlong_as_double(0x7ff0000000000000ll); }

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
  double* c8;               // [kCol8][kSlots]
  int32_t* c4;              // [kCol4][kSlots]

  __device__ double& d(int f, int s) { return c8[f * kSlots + s]; }
  __device__ int32_t& i(int f, int s) { return c4[f * kSlots + s]; }

  __device__ void cnt(int k, uint32_t v) { atomicAdd(s_u + k, (unsigned long long)v); }
  __device__ void fsum(int k, double v) { sf[k * sstride] += v; }

  __device__ uint32_t cidx(int32_t cx, int32_t cy) { return (uint32_t)cell_index(P.mesh, cx, cy); }

  // number density of cell (cx, cy)
  __device__ double nd_of(int32_t cx, int32_t cy) {
    const uint32_t ci = cidx(cx, cy);
    if constexpr (kBlk) return s_nd[dens_load_blk(P.mesh, s_blk, cx, cy, ci, pol)];
    else if constexpr (kFmt == kDensU8) return s_nd[ldg_u8_hint(P.mesh.rho8 + ci, pol)];
    else return number_density<kFmt>(P.mesh, P.mesh.nd_tab, ci, ph.cn);
  }

  // the flush of DESIGN.md §3: production RED or deterministic record
  __device__ void flush(int s, int32_t cx, int32_t cy, double& acc, double& dstep) {
    const uint32_t cell = cidx(cx, cy);
    if constexpr (kDet) {
      const int32_t pi = i(C_PID, s);
      const uint32_t seq = (uint32_t)i(C_SEQ, s);
      const unsigned long long rs = atomicAdd(P.rec_count, 1ull);
      if (rs < P.rec_cap) {
        P.rec_key[rs] = ((unsigned long long)cell << 40) |
                        ((unsigned long long)((int64_t)pi - P.lo) << 24) |
                        (unsigned long long)(seq & 0xffffffu);
        P.rec_val[rs] = acc;
      }
      if (seq >= (1u << 24)) cnt(SU_REC_OVERFLOW, 1u);
      i(C_SEQ, s) = (int32_t)(seq + 1u);
    } else {
      red_add_hint(P.mesh.tally + cell, acc, pol);
    }
    dstep += acc;
    acc = 0.0;
  }

  // A history ended in slot s: write the particle store (census: alive; otherwise dead).
  __device__ uint32_t finish(int s, double x, double y, double ox, double oy, double e, double w,
                             double mfp, double dstep, int32_t cx, int32_t cy, uint32_t ctr,
                             uint32_t nf, uint32_t nc, bool alive) {
    const int32_t pi = i(C_PID, s);
    if (!(isfinite(x) && isfinite(y) && isfinite(e) && isfinite(w))) cnt(SU_NONFINITE, 1u);
    P.p.x[pi] = x;
    P.p.y[pi] = y;
    P.p.ox[pi] = ox;
    P.p.oy[pi] = oy;
    P.p.e[pi] = e;
    P.p.w[pi] = w;
    P.p.mfp[pi] = mfp;
    P.p.dep[pi] += dstep;
    P.p.cx[pi] = cx;
    P.p.cy[pi] = cy;
    P.p.ctr[pi] = ctr;
    P.p.nfac[pi] += nf;
    P.p.ncol[pi] += nc;
    if (alive) P.p.ncen[pi] += 1u; else P.p.status[pi] = 0u;
    cnt(SU_FACETS, nf);
    cnt(SU_COLLISIONS, nc);
    fsum(SF_TALLY, dstep);
    return T_FREE;
  }

  // calculate_time_to_events + determine_next_event (Listing 2) for the
  // state in slot s (whose x, y, exn, eyn, iox, ioy, mfp, dcen, st, nd are stored): the
  // next event's type and distance go to the slot.  The event cap (R27) ends the
  // history here.  Same expressions as the history kernel (R28 clamps).
  __device__ uint32_t classify(int s, uint32_t nf, uint32_t nc) {
    if ((int64_t)(nf + nc) >= P.max_events) {
      double acc = d(C_ACC, s), dstep = d(C_DSTEP, s);
      const int32_t cx = i(C_CX, s), cy = i(C_CY, s);
      const double w = d(C_W, s), e = d(C_E, s);
      cnt(SU_EVENT_CAP, 1u);
      flush(s, cx, cy, acc, dstep);
      cnt(SU_KILLED, 1u);
      fsum(SF_KILLED_E, w * e);
      fsum(SF_KILLED_W, w);
      return finish(s, d(C_X, s), d(C_Y, s), d(C_OX, s), d(C_OY, s), e, w, d(C_MFP, s), dstep, cx,
                    cy, (uint32_t)i(C_CTR, s), nf, nc, false);
    }
    const double sig = d(C_ND, s) * d(C_ST, s);
    const double tx = (d(C_EXN, s) - d(C_X, s)) * d(C_IOX, s);
    const double ty = (d(C_EYN, s) - d(C_Y, s)) * d(C_IOY, s);
    const bool ax = ty > 0.0 && tx < ty;
    double df = ax ? tx : ty;
    df = df < 0.0 ? 0.0 : df;
    const double ds = d(C_DCEN, s);
    const double mfp = d(C_MFP, s);
    // n_mfp / Sigma_t only when a collision is possible (the history kernel's screen)
    const double dmin = df < ds ? df : ds;
    const double dsig = dmin * sig;
    const bool maybe_coll = !(mfp > dsig * 0x1.00001p+0) || dsig < 0x1p-960;
    if (maybe_coll && sig > 0.0) {
      const double dc = mfp / sig;
      if (dc < df && dc < ds) {
        d(C_D, s) = dc;
        return T_COLL;
      }
    }
    if (df < ds) {
      d(C_D, s) = df;
      return T_FACET | (ax ? T_AXBIT : 0u);
    }
    d(C_D, s) = ds;
    return T_CENSUS;
  }

  // ---- collision ----
  __device__ uint32_t collision(int s) {
    double x = d(C_X, s), y = d(C_Y, s), ox = d(C_OX, s), oy = d(C_OY, s);
    double w = d(C_W, s), e = d(C_E, s), acc = d(C_ACC, s), dstep = d(C_DSTEP, s);
    double dcen = d(C_DCEN, s);
    const double dd = d(C_D, s), nd = d(C_ND, s);
    const double sig = nd * d(C_ST, s);
    const double pa = d(C_PA, s);
    const int32_t cx = i(C_CX, s), cy = i(C_CY, s);
    uint32_t ctr = (uint32_t)i(C_CTR, s);
    const uint32_t nf = (uint32_t)i(C_NF, s);
    const uint32_t nc = (uint32_t)i(C_NC, s) + 1u;
    acc += ((w * dd) * sig) * d(C_H, s);
    x = x + dd * ox;
    y = y + dd * oy;
    dcen = dcen - dd;
    const uint64_t pid = (uint64_t)(P.first_id + i(C_PID, s));
    const U64x2 r = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
    ctr += 1u;
    double mfp_u = u01(r.b);
    bool absorbed = false;
    if (!ph.analog) {                           // implicit capture
      const double w0 = w;
      w = w * (1.0 - pa);
      fsum(SF_ABSORBED_W, w0 - w);
    } else if (u01(r.b) < pa) {                // sampled absorption (R31)
      absorbed = true;
    } else {                                    // scatter: n_mfp from the next counter
      const U64x2 r2 = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
      ctr += 1u;
      mfp_u = u01(r2.a);
    }
    if (absorbed) {
      flush(s, cx, cy, acc, dstep);
      fsum(SF_ABSORBED_W, w);
      fsum(SF_ABSORBED_E, w * e);
      cnt(SU_ABSORBED, 1u);
      return finish(s, x, y, ox, oy, e, w, d(C_MFP, s), dstep, cx, cy, ctr, nf, nc, false);
    }
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
      const U64x2 r3 = threefry2x64_20((uint64_t)ctr, 0, pid, P.seed);
      ctr += 1u;
      if (u01(r3.a) < w / ph.w_roul) {
        fsum(SF_ROULETTE, ph.w_roul - w);
        w = ph.w_roul;
        kill = false;
      }
    }
    if (kill) {
      flush(s, cx, cy, acc, dstep);
      fsum(SF_KILLED_E, w * e);
      fsum(SF_KILLED_W, w);
      cnt(SU_KILLED, 1u);
      return finish(s, x, y, ox, oy, e, w, d(C_MFP, s), dstep, cx, cy, ctr, nf, nc, false);
    }
    double exn = __ldg(P.mesh.ex + cx + (ox > 0.0 ? 1 : 0));
    double eyn = __ldg(P.mesh.ey + cy + (oy > 0.0 ? 1 : 0));
    dcen = tcen * speed(e, ph);
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    double iox = 1.0 / ox, ioy = 1.0 / oy;
    if (ox == 0.0) { exn = ev_inf(); iox = ev_inf(); }
    if (oy == 0.0) { eyn = ev_inf(); ioy = ev_inf(); }
    d(C_X, s) = x; d(C_Y, s) = y; d(C_OX, s) = ox; d(C_OY, s) = oy;
    d(C_IOX, s) = iox; d(C_IOY, s) = ioy; d(C_EXN, s) = exn; d(C_EYN, s) = eyn;
    d(C_MFP, s) = -log(mfp_u); d(C_DCEN, s) = dcen; d(C_ACC, s) = acc;
    d(C_W, s) = w; d(C_E, s) = e; d(C_ST, s) = m.st; d(C_H, s) = m.H; d(C_PA, s) = m.pa;
    i(C_NC, s) = (int32_t)nc;
    i(C_CTR, s) = (int32_t)ctr;
    return classify(s, nf, nc);
  }

  // ---- facet ----
  __device__ uint32_t facet(int s, bool ax) {
    double x = d(C_X, s), y = d(C_Y, s);
    double acc = d(C_ACC, s), dstep = d(C_DSTEP, s);
    const double dd = d(C_D, s), w = d(C_W, s);
    const double sig = d(C_ND, s) * d(C_ST, s);
    int32_t cx = i(C_CX, s), cy = i(C_CY, s);
    const uint32_t nf = (uint32_t)i(C_NF, s) + 1u;
    acc += ((w * dd) * sig) * d(C_H, s);
    d(C_MFP, s) = clamp0(d(C_MFP, s) - dd * sig);
    d(C_DCEN, s) = d(C_DCEN, s) - dd;
    const double ox = d(C_OX, s), oy = d(C_OY, s);
    const double xm = x + dd * ox, ym = y + dd * oy;
    x = ax ? d(C_EXN, s) : xm;                  // snap the crossed coordinate
    y = ax ? ym : d(C_EYN, s);
    flush(s, cx, cy, acc, dstep);               // deposit of the cell being left
    const int32_t c = ax ? cx : cy;
    const bool pos = ax ? (ox > 0.0) : (oy > 0.0);
    const int32_t cs = c + (pos ? 1 : -1);
    const bool refl = (uint32_t)cs >= (uint32_t)(ax ? P.mesh.nx : P.mesh.ny);
    const int32_t c2 = refl ? c : cs;
    if (refl) {
      if (ph.vacuum) {                          // vacuum boundary (R30): escape
        cnt(SU_ESCAPED, 1u);
        const double e = d(C_E, s);
        fsum(SF_ESCAPED_E, w * e);
        fsum(SF_ESCAPED_W, w);
        return finish(s, x, y, ox, oy, e, w, d(C_MFP, s), dstep, cx, cy, (uint32_t)i(C_CTR, s), nf,
                      (uint32_t)i(C_NC, s), false);
      }
      if (ax) { d(C_OX, s) = -ox; d(C_IOX, s) = -d(C_IOX, s); }
      else    { d(C_OY, s) = -oy; d(C_IOY, s) = -d(C_IOY, s); }
    }
    const bool pos2 = refl ? !pos : pos;
    const int32_t ke = pos2 ? c2 + 1 : c2;
    if (ax) { cx = c2; d(C_EXN, s) = __ldg(P.mesh.ex + ke); i(C_CX, s) = cx; }
    else    { cy = c2; d(C_EYN, s) = __ldg(P.mesh.ey + ke); i(C_CY, s) = cy; }
    d(C_X, s) = x;
    d(C_Y, s) = y;
    d(C_ACC, s) = acc;
    d(C_DSTEP, s) = dstep;
    d(C_ND, s) = nd_of(cx, cy);                 // the new cell's density
    i(C_NF, s) = (int32_t)nf;
    return classify(s, nf, (uint32_t)i(C_NC, s));
  }

  // ---- census ----
  __device__ uint32_t census(int s) {
    double acc = d(C_ACC, s), dstep = d(C_DSTEP, s);
    const double dd = d(C_D, s), w = d(C_W, s), e = d(C_E, s);
    const double ox = d(C_OX, s), oy = d(C_OY, s);
    const double sig = d(C_ND, s) * d(C_ST, s);
    const int32_t cx = i(C_CX, s), cy = i(C_CY, s);
    acc += ((w * dd) * sig) * d(C_H, s);
    const double x = d(C_X, s) + dd * ox;
    const double y = d(C_Y, s) + dd * oy;
    const double nm = d(C_MFP, s) - dd * sig;
    const double mfp = nm > 0.0 ? nm : 0.0;
    flush(s, cx, cy, acc, dstep);
    cnt(SU_CENSUS, 1u);
    fsum(SF_CENSUS_E, w * e);
    fsum(SF_CENSUS_W, w);
    return finish(s, x, y, ox, oy, e, w, mfp, dstep, cx, cy, (uint32_t)i(C_CTR, s),
                  (uint32_t)i(C_NF, s), (uint32_t)i(C_NC, s), true);
  }

  // ---- a new particle (local index in C_PID): its slot state and first event ----
  __device__ uint32_t birth(int s) {
    const int32_t pi = i(C_PID, s);
    if (P.p.status[pi] != 1u) return T_FREE;
    const double ox = P.p.ox[pi], oy = P.p.oy[pi];
    const double e = P.p.e[pi];
    const int32_t cx = P.p.cx[pi], cy = P.p.cy[pi];
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    double exn = __ldg(P.mesh.ex + cx + (ox > 0.0 ? 1 : 0));
    double eyn = __ldg(P.mesh.ey + cy + (oy > 0.0 ? 1 : 0));
    double iox = 1.0 / ox, ioy = 1.0 / oy;
    if (ox == 0.0) { exn = ev_inf(); iox = ev_inf(); }
    if (oy == 0.0) { eyn = ev_inf(); ioy = ev_inf(); }
    d(C_X, s) = P.p.x[pi]; d(C_Y, s) = P.p.y[pi]; d(C_OX, s) = ox; d(C_OY, s) = oy;
    d(C_IOX, s) = iox; d(C_IOY, s) = ioy; d(C_EXN, s) = exn; d(C_EYN, s) = eyn;
    d(C_MFP, s) = P.p.mfp[pi]; d(C_DCEN, s) = speed(e, ph) * P.dt;
    d(C_ACC, s) = 0.0; d(C_DSTEP, s) = 0.0;
    d(C_W, s) = P.p.w[pi]; d(C_E, s) = e; d(C_ST, s) = m.st; d(C_H, s) = m.H; d(C_PA, s) = m.pa;
    d(C_ND, s) = nd_of(cx, cy);
    i(C_CX, s) = cx; i(C_CY, s) = cy; i(C_NF, s) = 0; i(C_NC, s) = 0;
    i(C_CTR, s) = (int32_t)P.p.ctr[pi]; i(C_SEQ, s) = 0;
    cnt(SU_ALIVE, 1u);
    return classify(s, 0u, 0u);
  }
};

template <bool kDet, int kFmt, bool kBlk>
__global__ void __launch_bounds__(kEvBlock, 1) ev_loop_kernel(const __grid_constant__ EvParams E) {
  const TrackParams& P = E.P;
  extern __shared__ __align__(16) unsigned char smem[];
  __shared__ unsigned long long s_u[SU_COUNT];
  __shared__ double s_nd[kFmt == kDensU8 ? 256 : 1];
  double* c8 = reinterpret_cast<double*>(smem);
  int32_t* c4 = reinterpret_cast<int32_t*>(c8 + (size_t)kCol8 * kSlots);
  uint8_t* s_type = reinterpret_cast<uint8_t*>(c4 + (size_t)kCol4 * kSlots);
  uint8_t* s_wq = s_type + kSlots;             // per-warp event queue (slot offsets)
  uint8_t* s_blk = s_wq + kSlots;              // block map (kBlk)
  const int t = threadIdx.x;
  const int lane = t & 31, wid = t >> 5;
  const unsigned lt = (1u << lane) - 1u;
  const int bidx = (int)blockIdx.x;
  const int64_t gt = (int64_t)bidx * kEvBlock + t;
  const int64_t sstride = (int64_t)gridDim.x * kEvBlock;
  if (t < SU_COUNT) s_u[t] = 0u;
  for (int k = t; k < kSlots; k += kEvBlock) s_type[k] = (uint8_t)T_FREE;
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
  EvKernel<kDet, kFmt, kBlk> K{P, P.ph, s_nd, s_blk, s_u, P.slot_f + gt, sstride, l2_evict_last(), c8, c4};
  const unsigned long long span = (unsigned long long)(P.hi - P.lo);
  const int sb = wid * kWSlots;                // this warp's slots [sb, sb + 64)
  uint8_t* wq = s_wq + sb;
  bool exhausted = false;
  unsigned iter = 0;
  for (;; ++iter) {
    __syncwarp();
    uint32_t ta = s_type[sb + lane], tb = s_type[sb + 32 + lane];
    // ---- refill: new particles for the free slots (one atomicAdd per warp) ----
    const unsigned fa = __ballot_sync(kFull, ta == T_FREE), fb = __ballot_sync(kFull, tb == T_FREE);
    const unsigned nfree = (unsigned)(__popc(fa) + __popc(fb));
    if (!exhausted && nfree >= (unsigned)kEvRefill) {
      unsigned long long base = 0;
      if (lane == 0) base = atomicAdd(&E.ctl->counter, (unsigned long long)nfree);
      base = __shfl_sync(kFull, base, 0);
      const unsigned long long avail = base < span ? (span - base < nfree ? span - base : nfree) : 0ull;
      if (base + nfree >= span) exhausted = true;
      const unsigned ra = (unsigned)__popc(fa & lt), rb = (unsigned)(__popc(fa) + __popc(fb & lt));
      if (ta == T_FREE && ra < avail) {
        K.i(C_PID, sb + lane) = (int32_t)(P.lo + (int64_t)(base + ra));
        ta = T_BIRTH;
      }
      if (tb == T_FREE && rb < avail) {
        K.i(C_PID, sb + 32 + lane) = (int32_t)(P.lo + (int64_t)(base + rb));
        tb = T_BIRTH;
      }
    }
    if (!__any_sync(kFull, ta != T_FREE || tb != T_FREE)) {
      if (exhausted) break;
      continue;
    }
    // ---- Listing 2: all collisions, then all facets, then all census, then the births ----
#pragma unroll 1
    for (uint32_t T = 0; T < 4; ++T) {
      const bool a = (ta & 7u) == T, b = (tb & 7u) == T;
      const unsigned ma = __ballot_sync(kFull, a), mb = __ballot_sync(kFull, b);
      const int na = __popc(ma), n = na + __popc(mb);
      if (n == 0) continue;
      if (a) wq[__popc(ma & lt)] = (uint8_t)lane;
      if (b) wq[na + __popc(mb & lt)] = (uint8_t)(32 + lane);
      __syncwarp();
      for (int k = lane; k < n; k += 32) {
        const int s = sb + wq[k];
        uint32_t nt;
        if (T == T_COLL) nt = K.collision(s);
        else if (T == T_FACET) nt = K.facet(s, (s_type[s] & T_AXBIT) != 0);
        else if (T == T_CENSUS) nt = K.census(s);
        else nt = K.birth(s);
        s_type[s] = (uint8_t)nt;
      }
      __syncwarp();
    }
  }
  if (lane == 0 && iter > 0) atomicMax(&E.ctl->iter, iter);

  // ---- statistics: one atomic per statistic per CTA ----
  __syncthreads();
  if (t < SU_COUNT && s_u[t]) atomicAdd(P.stats_u + t, s_u[t]);
  for (int k = wid; k < SF_COUNT; k += kEvWarps) {
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
  if (s->ctl) cudaFree(s->ctl);
  if (s->slot_f) cudaFree(s->slot_f);
  delete s;
}

// One particle range [tp.lo, tp.hi): the per-warp event loops of one CTA per SM,
// statistics into tp.stats_*.
nt_status event_run_range(EventState* s, const TrackParams& tp, bool det, int sm_count,
                          cudaStream_t st, uint32_t& launches, std::string& err) {
  const bool blk = tp.mesh.fmt == kDensU8 && tp.mesh.blk != nullptr;
  void* fn = ev_fn(det, tp.mesh.fmt, blk);
  const size_t smem = ev_smem_bytes(blk);
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) { err = std::string("event loop smem: ") + cudaGetErrorString(e); return NT_ERR_CUDA; }
  int per_sm = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, fn, kEvBlock, smem);
  if (per_sm < 1) { err = "event loop: no resident CTA (shared memory)"; return NT_ERR_CUDA; }
  const int grid = sm_count * per_sm;
  if (!s->ctl) {
    e = device_malloc(reinterpret_cast<void**>(&s->ctl), sizeof(EvCtl));
    if (e != cudaSuccess) { s->ctl = nullptr; err = cudaGetErrorString(e); return NT_ERR_OOM; }
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
  ep.ctl = s->ctl;
  e = cudaMemsetAsync(s->ctl, 0, sizeof(EvCtl), st);
  if (e != cudaSuccess) { err = cudaGetErrorString(e); return NT_ERR_CUDA; }
  if (tp.hi > tp.lo) {
    void* args[] = {&ep};
    e = cudaLaunchKernel(fn, dim3(grid), dim3(kEvBlock), args, smem, st);
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
