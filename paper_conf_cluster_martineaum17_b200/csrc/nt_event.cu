// nt_event.cu -- event-based (Over Events) variant of the tracker, P:358-390 (§V-B).
//
// Listing 2 advances every particle by one event per iteration: compute the time to each
// event and determine the next one, then handle all collisions, all facets and all census
// events in separate loops.  Here the particle set is split into per-warp sets
// of 64 slots, and each warp runs Listing 2 on its own set with warp-level per-type
// queues: lane k owns slots k and k + 32 and keeps their next-event types in registers; per
// iteration one REDUX finds the types present, and each present type (collisions, facets,
// census, new particles) is handled in at most two rounds -- round 1 one event of every lane
// holding one, round 2 the second event of lanes holding two (one vote) -- so every round
// runs one event type across the warp (converged code, the Over Events advantage,
// P:384-390) and touches one slot per bank pair per half-warp (bank-conflict free).  No
// CTA-wide barrier runs inside the loop: warps proceed independently, and a warp refills its
// free slots from a global counter (one atomicAdd per refill) whenever enough are free, so
// every warp stays busy until the id range is exhausted (the load balancing of P:344-348).
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
#define NT_EV_REFILL 4
#endif
constexpr int kEvWarps = NT_EV_WARPS;        // warps per CTA (one CTA per SM)
constexpr int kEvBlock = kEvWarps * 32;
constexpr int kWSlots = 64;                  // slots per warp: two per lane
constexpr int kSlots = kEvWarps * kWSlots;   // slots per CTA
constexpr int kEvRefill = NT_EV_REFILL;      // a warp refills once this many slots are free

// Type byte of a slot (kept in the owning lane's registers): bits 0-2 the next event (or
// free / birth), bit 3 the facet crosses an X edge, bit 4 the slot's deposit accumulator is
// non-zero (it is zero after every flush, so most events neither load nor store it), bit 5
// the current cell's block (of the block map) is uniform, so a facet that stays in the
// block keeps the stored number density (every cell of the block has it).
enum : uint32_t { T_COLL = 0, T_FACET = 1, T_CENSUS = 2, T_BIRTH = 3, T_FREE = 4, T_AXBIT = 8,
                  T_ACCBIT = 16, T_UNIBIT = 32 };

// Slot columns, 16 bytes each: fields that are read (and mostly written) together share a
// column, so one LDS.128 / STS.128 moves both (a lane touches slot k or k + 32 only, so a
// quarter-warp's 16-byte accesses never share a bank group).
enum Col : int {
  P_XY = 0,   // x, y
  P_O,        // omega_x, omega_y
  P_IO,       // 1/omega_x, 1/omega_y
  P_EN,       // heading edges x, y
  P_MD,       // n_mfp, census distance
  P_AD,       // deposit accumulator, deposits flushed this step
  P_WH,       // weight, heating response H
  P_SN,       // sigma_t (m^2), number density of the cell
  P_EP,       // energy, p_a
  P_CN,       // int4: cx, cy, facets, collisions (this step)
  P_CS,       // int4: RNG counter, flush sequence, local particle index, -
  kCols
};

constexpr size_t ev_smem_bytes(bool blk) {
  return (size_t)kSlots * kCols * 16 + (blk ? (size_t)kBlkMax : 0);
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

// A particle's state in registers while one of its events is handled.
struct St {
  double x, y, ox, oy, iox, ioy, exn, eyn, mfp, dcen, acc, dstep, w, e, st, H, nd, pa;
  int32_t cx, cy;
  uint32_t nf, nc, ctr;
  uint32_t uni;             // T_UNIBIT when the cell's block is uniform
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
  double2* cols;            // [kCols][kSlots] 16-byte entries

  __device__ double2& c(int f, int s) { return cols[f * kSlots + s]; }
  __device__ int4& ci(int f, int s) { return reinterpret_cast<int4*>(cols + f * kSlots)[s]; }
  // one 8-byte half of a 16-byte entry
  __device__ double& h(int f, int s, int k) { return reinterpret_cast<double*>(cols + f * kSlots + s)[k]; }
  __device__ int32_t pid(int s) { return ci(P_CS, s).z; }

  __device__ void cnt(int k, uint32_t v) { atomicAdd(s_u + k, (unsigned long long)v); }
  __device__ void fsum(int k, double v) { red_add_f64(sf + k * sstride, v); }

  __device__ uint32_t cidx(int32_t cx, int32_t cy) {
    const uint32_t c = (uint32_t)cell_index(P.mesh, cx, cy);
    NT_CHECK(c < storage_cells(P.mesh));
    return c;
  }

  __device__ double edge_x(int32_t k) { return __ldg(P.mesh.ex + k); }
  __device__ double edge_y(int32_t k) { return __ldg(P.mesh.ey + k); }

  // number density of cell (cx, cy); uni: its block is uniform (block map)
  __device__ double nd_of(int32_t cx, int32_t cy, bool& uni) {
    const uint32_t ci_ = cidx(cx, cy);
    uni = false;
    if constexpr (kBlk) {
      uint32_t code = s_blk[(cy >> P.mesh.bshift) * P.mesh.nbx + (cx >> P.mesh.bshift)];
      uni = code != kBlkMixed;
      if (!uni) code = ldg_u8_hint(P.mesh.rho8 + ci_, pol);
      return s_nd[code];
    } else if constexpr (kFmt == kDensU8) {
      return s_nd[ldg_u8_hint(P.mesh.rho8 + ci_, pol)];
    } else {
      return number_density<kFmt>(P.mesh, P.mesh.nd_tab, ci_, ph.cn);
    }
  }

  // the flush of DESIGN.md §3: production RED or deterministic record
  __device__ void flush(int s, St& v) {
    const uint32_t cell = cidx(v.cx, v.cy);
    if constexpr (kDet) {
      int4 cs = ci(P_CS, s);
      const uint32_t seq = (uint32_t)cs.y;
      const unsigned long long rs = atomicAdd(P.rec_count, 1ull);
      if (rs < P.rec_cap) {
        P.rec_key[rs] = ((unsigned long long)cell << 40) |
                        ((unsigned long long)((int64_t)cs.z - P.lo) << 24) |
                        (unsigned long long)(seq & 0xffffffu);
        P.rec_val[rs] = v.acc;
      }
      if (seq >= (1u << 24)) cnt(SU_REC_OVERFLOW, 1u);
      cs.y = (int)(seq + 1u);
      ci(P_CS, s) = cs;
    } else {
      red_add_hint(P.mesh.tally + cell, v.acc, pol);
    }
    v.dstep += v.acc;
    v.acc = 0.0;
  }

  // A history ended in slot s: write the particle store (census: alive; otherwise dead).
  __device__ uint32_t finish(int s, const St& v, bool alive) {
    const int32_t pi = pid(s);
    if (!(isfinite(v.x) && isfinite(v.y) && isfinite(v.e) && isfinite(v.w))) cnt(SU_NONFINITE, 1u);
    P.p.x[pi] = v.x;
    P.p.y[pi] = v.y;
    P.p.ox[pi] = v.ox;
    P.p.oy[pi] = v.oy;
    P.p.e[pi] = v.e;
    P.p.w[pi] = v.w;
    P.p.mfp[pi] = v.mfp;
    red_add_f64(P.p.dep + pi, v.dstep);         // the particle's ledgers: no load here
    P.p.cx[pi] = v.cx;
    P.p.cy[pi] = v.cy;
    P.p.ctr[pi] = v.ctr;
    red_add_u32(P.p.nfac + pi, v.nf);
    red_add_u32(P.p.ncol + pi, v.nc);
    if (alive) red_add_u32(P.p.ncen + pi, 1u); else P.p.status[pi] = 0u;
    cnt(SU_FACETS, v.nf);
    cnt(SU_COLLISIONS, v.nc);
    fsum(SF_TALLY, v.dstep);
    return T_FREE;
  }

  // The event cap (R27): flush, count, kill.  v.e, v.ox, v.oy, v.ctr must be loaded.
  __device__ uint32_t cap_kill(int s, St& v) {
    cnt(SU_EVENT_CAP, 1u);
    flush(s, v);
    cnt(SU_KILLED, 1u);
    fsum(SF_KILLED_E, v.w * v.e);
    fsum(SF_KILLED_W, v.w);
    return finish(s, v, false);
  }

  // calculate_time_to_events + determine_next_event (Listing 2) from the
  // state in registers: the type bits are returned (the handler re-derives the event's
  // distance from the state it loads anyway -- the same expressions, so the same value --
  // instead of a stored distance column).  Same expressions as the history kernel
  // (R28 clamps).
  __device__ uint32_t classify(const St& v) {
    const double sig = v.nd * v.st;
    const double tx = (v.exn - v.x) * v.iox;
    const double ty = (v.eyn - v.y) * v.ioy;
    const bool ax = ty > 0.0 && tx < ty;
    double df = ax ? tx : ty;
    df = df < 0.0 ? 0.0 : df;
    const double ds = v.dcen;
    const uint32_t accb = (v.acc != 0.0 ? T_ACCBIT : 0u) | v.uni;
    // n_mfp / Sigma_t only when a collision is possible (the history kernel's screen)
    const double dmin = df < ds ? df : ds;
    const double dsig = dmin * sig;
    const bool maybe_coll = !(v.mfp > dsig * 0x1.00001p+0) || dsig < 0x1p-960;
    if (maybe_coll && sig > 0.0) {
      const double dc = v.mfp / sig;
      if (dc < df && dc < ds) return T_COLL | accb;
    }
    if (df < ds) return T_FACET | (ax ? T_AXBIT : 0u) | accb;
    return T_CENSUS | accb;
  }

  __device__ void load_cn(int s, St& v) {
    const int4 a = ci(P_CN, s);
    v.cx = a.x; v.cy = a.y; v.nf = (uint32_t)a.z; v.nc = (uint32_t)a.w;
  }
  __device__ void store_cn(int s, const St& v) {
    ci(P_CN, s) = make_int4(v.cx, v.cy, (int)v.nf, (int)v.nc);
  }
  // acc (only while its type bit says it is non-zero) and dstep
  __device__ void load_ad(int s, uint32_t ty, St& v) {
    if (ty & T_ACCBIT) {
      const double2 a = c(P_AD, s);
      v.acc = a.x; v.dstep = a.y;
    } else {
      v.acc = 0.0; v.dstep = h(P_AD, s, 1);
    }
  }

  // ---- collision ----
  __device__ uint32_t collision(int s, uint32_t ty) {
    St v;
    { const double2 a = c(P_XY, s); v.x = a.x; v.y = a.y; }
    { const double2 a = c(P_O, s); v.ox = a.x; v.oy = a.y; }
    { const double2 a = c(P_MD, s); v.mfp = a.x; v.dcen = a.y; }
    load_ad(s, ty, v);
    { const double2 a = c(P_WH, s); v.w = a.x; v.H = a.y; }
    { const double2 a = c(P_EP, s); v.e = a.x; v.pa = a.y; }
    { const double2 a = c(P_SN, s); v.st = a.x; v.nd = a.y; }
    v.uni = ty & T_UNIBIT;
    load_cn(s, v);
    int4 cs = ci(P_CS, s);
    v.ctr = (uint32_t)cs.x;
    const double sig = v.nd * v.st;
    const double dd = v.mfp / sig;               // the collision distance classify compared
    v.nc += 1u;
    v.acc += ((v.w * dd) * sig) * v.H;
    v.x = v.x + dd * v.ox;
    v.y = v.y + dd * v.oy;
    v.dcen = v.dcen - dd;
    const uint64_t pidg = (uint64_t)(P.first_id + cs.z);
    const U64x2 r = threefry2x64_20((uint64_t)v.ctr, 0, pidg, P.seed);
    v.ctr += 1u;
    double mfp_u = u01(r.b);
    bool absorbed = false;
    if (!ph.analog) {                           // implicit capture
      const double w0 = v.w;
      v.w = v.w * (1.0 - v.pa);
      fsum(SF_ABSORBED_W, w0 - v.w);
    } else if (u01(r.b) < v.pa) {              // sampled absorption (R31)
      absorbed = true;
    } else {                                    // scatter: n_mfp from the next counter
      const U64x2 r2 = threefry2x64_20((uint64_t)v.ctr, 0, pidg, P.seed);
      v.ctr += 1u;
      mfp_u = u01(r2.a);
    }
    if (absorbed) {
      flush(s, v);
      fsum(SF_ABSORBED_W, v.w);
      fsum(SF_ABSORBED_E, v.w * v.e);
      cnt(SU_ABSORBED, 1u);
      return finish(s, v, false);
    }
    const double e = v.e;
    const double mu = 1.0 - 2.0 * u01(r.a);
    const double e2 = e * (((ph.AA + ph.twoA * mu) + 1.0) / ph.Ap1sq);
    const double ct = 0.5 * (ph.Ap1 * sqrt(e2 / e) - ph.Am1 * sqrt(e / e2));
    const double sgn = (r.a & 1ull) ? -1.0 : 1.0;
    const double q = 1.0 - ct * ct;
    const double stt = sgn * sqrt(q > 0.0 ? q : 0.0);
    const double nox = v.ox * ct - v.oy * stt;
    const double noy = v.ox * stt + v.oy * ct;
    v.ox = nox;
    v.oy = noy;
    const double tcen = v.dcen / speed(e, ph);
    v.e = e2;
    bool kill = v.e < ph.e_min || v.w < ph.w_min;   // termination
    if (kill && ph.roulette && !(v.e < ph.e_min)) {
      // Russian roulette (R32): survive with probability w / w_s at weight w_s
      const U64x2 r3 = threefry2x64_20((uint64_t)v.ctr, 0, pidg, P.seed);
      v.ctr += 1u;
      if (u01(r3.a) < v.w / ph.w_roul) {
        fsum(SF_ROULETTE, ph.w_roul - v.w);
        v.w = ph.w_roul;
        kill = false;
      }
    }
    if (kill) {
      flush(s, v);
      fsum(SF_KILLED_E, v.w * v.e);
      fsum(SF_KILLED_W, v.w);
      cnt(SU_KILLED, 1u);
      return finish(s, v, false);
    }
    v.exn = edge_x(v.cx + (v.ox > 0.0 ? 1 : 0));
    v.eyn = edge_y(v.cy + (v.oy > 0.0 ? 1 : 0));
    v.dcen = tcen * speed(v.e, ph);
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, v.e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    v.st = m.st;
    v.H = m.H;
    v.pa = m.pa;
    v.iox = 1.0 / v.ox;
    v.ioy = 1.0 / v.oy;
    if (v.ox == 0.0) { v.exn = ev_inf(); v.iox = ev_inf(); }
    if (v.oy == 0.0) { v.eyn = ev_inf(); v.ioy = ev_inf(); }
    v.mfp = -log(mfp_u);
    cs.x = (int)v.ctr;
    ci(P_CS, s) = cs;
    store_cn(s, v);
    if ((int64_t)(v.nf + v.nc) >= P.max_events) return cap_kill(s, v);
    c(P_XY, s) = make_double2(v.x, v.y);
    c(P_O, s) = make_double2(v.ox, v.oy);
    c(P_IO, s) = make_double2(v.iox, v.ioy);
    c(P_EN, s) = make_double2(v.exn, v.eyn);
    c(P_MD, s) = make_double2(v.mfp, v.dcen);
    c(P_AD, s) = make_double2(v.acc, v.dstep);
    c(P_WH, s) = make_double2(v.w, v.H);
    c(P_EP, s) = make_double2(v.e, v.pa);
    c(P_SN, s) = make_double2(v.st, v.nd);
    return classify(v);
  }

  // ---- facet ----
  // Three stages: pre (state loads; the next cell, its heading edge and its density depend
  // only on the cell and the direction, so those loads go first), math (deposit, timers,
  // snap, flush -- no branch), post (reflection, stores, event cap, classification).  (A
  // lane holding two facets handling both interleaved, for twice the ILP, was measured and
  // rejected: csp 70.5 -> 91.2 ms, profiles/ab/r02_ab9.)
  struct Fct {
    St v;
    double om, enew, ndn;
    int32_t c, c2, ncx, ncy;
    uint32_t uni;
    bool ax, refl, keep;
  };

  __device__ void facet_pre(int s, uint32_t ty, Fct& f) {
    St& v = f.v;
    f.ax = (ty & T_AXBIT) != 0;
    load_cn(s, v);
    { const double2 a = c(P_IO, s); v.iox = a.x; v.ioy = a.y; }
    f.c = f.ax ? v.cx : v.cy;
    const bool pos = (f.ax ? v.iox : v.ioy) > 0.0;  // crossed axis' direction: sign of 1/omega
    const int32_t cs = f.c + (pos ? 1 : -1);
    f.refl = (uint32_t)cs >= (uint32_t)(f.ax ? P.mesh.gnx : P.mesh.ny);
    f.c2 = f.refl ? f.c : cs;
    const int32_t ke = (f.refl ? !pos : pos) ? f.c2 + 1 : f.c2;
    f.enew = f.ax ? edge_x(ke) : edge_y(ke);
    f.ncx = f.ax ? f.c2 : v.cx;
    f.ncy = f.ax ? v.cy : f.c2;
    // the new cell's density: unchanged when the facet stays inside a uniform
    // block of the block map (a reflection keeps the cell)
    f.uni = ty & T_UNIBIT;
    f.keep = false;
    if constexpr (kBlk) f.keep = f.uni && ((f.c2 >> P.mesh.bshift) == (f.c >> P.mesh.bshift));
    f.ndn = 0.0;
    if (!f.keep) {
      bool u;
      f.ndn = nd_of(f.ncx, f.ncy, u);
      f.uni = u ? T_UNIBIT : 0u;
    }
    { const double2 a = c(P_XY, s); v.x = a.x; v.y = a.y; }
    { const double2 a = c(P_EN, s); v.exn = a.x; v.eyn = a.y; }
    // the direction cosine of the coordinate that moves (the other is snapped to the edge)
    f.om = h(P_O, s, f.ax ? 1 : 0);
    { const double2 a = c(P_MD, s); v.mfp = a.x; v.dcen = a.y; }
    load_ad(s, ty, v);
    { const double2 a = c(P_WH, s); v.w = a.x; v.H = a.y; }
    { const double2 a = c(P_SN, s); v.st = a.x; v.nd = a.y; }
  }

  __device__ void facet_math(int s, Fct& f) {
    St& v = f.v;
    const double sig = v.nd * v.st;
    // the facet distance classify chose (axis from the type byte), clamped at 0 (R28)
    double dd = f.ax ? (v.exn - v.x) * v.iox : (v.eyn - v.y) * v.ioy;
    dd = dd < 0.0 ? 0.0 : dd;
    v.nf += 1u;
    v.acc += ((v.w * dd) * sig) * v.H;
    v.mfp = clamp0(v.mfp - dd * sig);
    v.dcen = v.dcen - dd;
    const double moved = (f.ax ? v.y : v.x) + dd * f.om;
    v.x = f.ax ? v.exn : moved;                 // snap the crossed coordinate
    v.y = f.ax ? moved : v.eyn;
    flush(s, v);                                // deposit of the cell being left
  }

  __device__ uint32_t facet_post(int s, Fct& f) {
    St& v = f.v;
    if (f.refl) {
      { const double2 a = c(P_O, s); v.ox = a.x; v.oy = a.y; }
      if (ph.vacuum) {                          // vacuum boundary (R30): escape
        v.e = h(P_EP, s, 0);
        v.ctr = (uint32_t)ci(P_CS, s).x;
        cnt(SU_ESCAPED, 1u);
        fsum(SF_ESCAPED_E, v.w * v.e);
        fsum(SF_ESCAPED_W, v.w);
        return finish(s, v, false);
      }
      if (f.ax) { v.ox = -v.ox; v.iox = -v.iox; }
      else      { v.oy = -v.oy; v.ioy = -v.ioy; }
      c(P_O, s) = make_double2(v.ox, v.oy);
      c(P_IO, s) = make_double2(v.iox, v.ioy);
    }
    v.cx = f.ncx;
    v.cy = f.ncy;
    if (f.ax) v.exn = f.enew; else v.eyn = f.enew;
    c(P_EN, s) = make_double2(v.exn, v.eyn);
    v.uni = f.uni;
    if (!f.keep) {
      v.nd = f.ndn;
      h(P_SN, s, 1) = v.nd;
    }
    store_cn(s, v);
    if ((int64_t)(v.nf + v.nc) >= P.max_events) {
      v.e = h(P_EP, s, 0);
      { const double2 a = c(P_O, s); v.ox = a.x; v.oy = a.y; }
      v.ctr = (uint32_t)ci(P_CS, s).x;
      return cap_kill(s, v);
    }
    c(P_XY, s) = make_double2(v.x, v.y);
    c(P_MD, s) = make_double2(v.mfp, v.dcen);
    h(P_AD, s, 1) = v.dstep;                    // acc == 0 after the flush
    return classify(v);
  }

  __device__ uint32_t facet(int s, uint32_t ty) {
    Fct f;
    facet_pre(s, ty, f);
    facet_math(s, f);
    return facet_post(s, f);
  }

  // ---- census ----
  __device__ uint32_t census(int s, uint32_t ty) {
    St v;
    { const double2 a = c(P_O, s); v.ox = a.x; v.oy = a.y; }
    load_ad(s, ty, v);
    { const double2 a = c(P_WH, s); v.w = a.x; v.H = a.y; }
    v.e = h(P_EP, s, 0);
    load_cn(s, v);
    v.ctr = (uint32_t)ci(P_CS, s).x;
    const double2 md = c(P_MD, s);
    const double dd = md.y;                     // census: the remaining census distance
    const double2 sn = c(P_SN, s);
    const double sig = sn.y * sn.x;
    v.acc += ((v.w * dd) * sig) * v.H;
    const double2 xy = c(P_XY, s);
    v.x = xy.x + dd * v.ox;
    v.y = xy.y + dd * v.oy;
    const double nm = md.x - dd * sig;
    v.mfp = nm > 0.0 ? nm : 0.0;
    flush(s, v);
    cnt(SU_CENSUS, 1u);
    fsum(SF_CENSUS_E, v.w * v.e);
    fsum(SF_CENSUS_W, v.w);
    return finish(s, v, true);
  }

  // ---- a new particle (local index in P_CS.z): its slot state and first event ----
  __device__ uint32_t birth(int s) {
    const int32_t pi = pid(s);
    // the state loads go out with the status load (one round trip instead of two)
    const uint32_t st_i = ld_volatile_u8(P.p.status + pi);
    St v;
    v.ox = __ldcs(P.p.ox + pi); v.oy = __ldcs(P.p.oy + pi);
    v.e = __ldcs(P.p.e + pi);
    v.cx = __ldcs(P.p.cx + pi); v.cy = __ldcs(P.p.cy + pi);
    v.x = __ldcs(P.p.x + pi); v.y = __ldcs(P.p.y + pi);
    v.mfp = __ldcs(P.p.mfp + pi); v.w = __ldcs(P.p.w + pi);
    v.ctr = __ldcs(P.p.ctr + pi);
    if (st_i != 1u) return T_FREE;
    uint32_t nr = 0;
    const Mat m = refresh_xs(P.xs, ph, v.e, nr);
    if (nr) cnt(SU_XS_RANGE, nr);
    v.exn = edge_x(v.cx + (v.ox > 0.0 ? 1 : 0));
    v.eyn = edge_y(v.cy + (v.oy > 0.0 ? 1 : 0));
    v.iox = 1.0 / v.ox;
    v.ioy = 1.0 / v.oy;
    if (v.ox == 0.0) { v.exn = ev_inf(); v.iox = ev_inf(); }
    if (v.oy == 0.0) { v.eyn = ev_inf(); v.ioy = ev_inf(); }
    v.dcen = speed(v.e, ph) * P.dt;
    v.acc = 0.0; v.dstep = 0.0;
    v.st = m.st; v.H = m.H; v.pa = m.pa;
    bool u;
    v.nd = nd_of(v.cx, v.cy, u);
    v.uni = u ? T_UNIBIT : 0u;
    v.nf = 0u; v.nc = 0u;
    cnt(SU_ALIVE, 1u);
    c(P_XY, s) = make_double2(v.x, v.y);
    c(P_O, s) = make_double2(v.ox, v.oy);
    c(P_IO, s) = make_double2(v.iox, v.ioy);
    c(P_EN, s) = make_double2(v.exn, v.eyn);
    c(P_MD, s) = make_double2(v.mfp, v.dcen);
    c(P_AD, s) = make_double2(0.0, 0.0);
    c(P_WH, s) = make_double2(v.w, v.H);
    c(P_EP, s) = make_double2(v.e, v.pa);
    c(P_SN, s) = make_double2(v.st, v.nd);
    store_cn(s, v);
    ci(P_CS, s) = make_int4((int)v.ctr, 0, pi, 0);
    if (P.max_events <= 0) return cap_kill(s, v);
    return classify(v);
  }
};

template <bool kDet, int kFmt, bool kBlk>
__global__ void __launch_bounds__(kEvBlock, 1) ev_loop_kernel(const __grid_constant__ EvParams E) {
  const TrackParams& P = E.P;
  extern __shared__ __align__(16) unsigned char smem[];
  __shared__ unsigned long long s_u[SU_COUNT];
  __shared__ double s_nd[kFmt == kDensU8 ? 256 : 1];
  double2* cols = reinterpret_cast<double2*>(smem);
  uint8_t* s_blk = reinterpret_cast<uint8_t*>(cols + (size_t)kCols * kSlots);   // block map (kBlk)
  const int t = threadIdx.x;
  const int lane = t & 31, wid = t >> 5;
  const unsigned lt = (1u << lane) - 1u;
  const int bidx = (int)blockIdx.x;
  const int64_t gt = (int64_t)bidx * kEvBlock + t;
  const int64_t sstride = (int64_t)gridDim.x * kEvBlock;
  if (t < SU_COUNT) s_u[t] = 0u;
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
  EvKernel<kDet, kFmt, kBlk> K{P, P.ph, s_nd, s_blk, s_u, P.slot_f + gt, sstride, l2_evict_last(), cols};
  const unsigned long long span = (unsigned long long)(P.hi - P.lo);
  const int sb = wid * kWSlots;                // this warp's slots [sb, sb + 64)
  bool exhausted = false;
  unsigned iter = 0;
  // Lane k owns slots sb + k and sb + 32 + k; their type bytes live in its registers.
  uint32_t ta = T_FREE, tb = T_FREE;
  for (;; ++iter) {
    // the event types present in the warp's slots (one REDUX): absent types cost nothing,
    // and the refill votes run only when a slot is free
    unsigned present = __reduce_or_sync(kFull, (1u << (ta & 7u)) | (1u << (tb & 7u)));
    if (!exhausted && (present & (1u << T_FREE))) {
      // ---- refill: new particles for the free slots (one atomicAdd per warp) ----
      const unsigned fa = __ballot_sync(kFull, ta == T_FREE), fb = __ballot_sync(kFull, tb == T_FREE);
      const unsigned nfree = (unsigned)(__popc(fa) + __popc(fb));
      if (nfree >= (unsigned)kEvRefill) {
        unsigned long long base = 0;
        if (lane == 0) base = atomicAdd(&E.ctl->counter, (unsigned long long)nfree);
        base = __shfl_sync(kFull, base, 0);
        const unsigned long long avail = base < span ? (span - base < nfree ? span - base : nfree) : 0ull;
        if (base + nfree >= span) exhausted = true;
        const unsigned ra = (unsigned)__popc(fa & lt), rb = (unsigned)(__popc(fa) + __popc(fb & lt));
        if (ta == T_FREE && ra < avail) {
          K.ci(P_CS, sb + lane).z = (int32_t)(P.lo + (int64_t)(base + ra));
          ta = T_BIRTH;
        }
        if (tb == T_FREE && rb < avail) {
          K.ci(P_CS, sb + 32 + lane).z = (int32_t)(P.lo + (int64_t)(base + rb));
          tb = T_BIRTH;
        }
        if (avail > 0ull) present |= 1u << T_BIRTH;
      }
    }
    if (!(present & 0xfu)) {                   // every slot free
      if (exhausted) break;
      continue;
    }
    // ---- Listing 2: all collisions, then all facets, then all census, then the births ----
    // Lane-paired per-type queues: a type's events run in at most two rounds -- round 1 one
    // event of every lane holding one, round 2 the second of lanes holding two -- so a round
    // touches slot k or k + 32 only: conflict-free shared-memory accesses.  Only the present
    // types are visited (find-first-set over the REDUX), in Listing 2's order.
#pragma unroll 1
    for (unsigned pm = present & 0xfu; pm != 0u; pm &= pm - 1u) {
      const uint32_t T = (uint32_t)(__ffs(pm) - 1);
      bool pa = (ta & 7u) == T, pb = (tb & 7u) == T;
#pragma unroll 1
      do {                                      // (the type is present: round 1 always runs)
        if (pa || pb) {
          const bool first = pa;
          const int s = sb + (first ? lane : 32 + lane);
          const uint32_t ty = first ? ta : tb;
          uint32_t nt;
          if (T == T_COLL) nt = K.collision(s, ty);
          else if (T == T_FACET) nt = K.facet(s, ty);
          else if (T == T_CENSUS) nt = K.census(s, ty);
          else nt = K.birth(s);
          if (first) { ta = nt; pa = false; } else { tb = nt; pb = false; }
        }
      } while (__any_sync(kFull, pa || pb));
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
