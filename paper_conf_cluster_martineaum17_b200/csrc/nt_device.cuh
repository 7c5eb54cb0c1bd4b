// nt_device.cuh -- device-side building blocks of the tracker (sm_100a).
//
// Everything here implements DESIGN.md §3 (the paper's method as read in DESIGN.md §4)
// and is written independently of oracle/ (no shared code).  The library is compiled
// with -fmad=false so every expression rounds exactly as parenthesised.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace nt {

// ---- physical constants (DESIGN.md §4 R4) -------------------------------------------
constexpr double kAvogadro = 6.02214076e23;     // mol^-1
constexpr double kEv = 1.602176634e-19;         // J
constexpr double kNeutronMass = 1.67492749804e-27;  // kg
constexpr double kBarn = 1.0e-28;               // m^2
constexpr double kTwoPi = 6.283185307179586;
constexpr unsigned kFull = 0xffffffffu;

// ---- data layout -----------------------------------------------------------------------
// Particle store: structure of arrays, one column per field, indexed by local index.
// Coalesced 8 B / 4 B / 1 B column accesses for a warp handling consecutive particles.
struct Soa {
  double *x, *y, *ox, *oy, *e, *w, *mfp, *dep;
  int32_t *cx, *cy;
  uint32_t *ctr, *nfac, *ncol, *ncen;
  uint8_t *status;             // 1 alive (at census), 0 dead, 2 parked mid-step (deferral)
  // mid-step state of a particle parked by the history kernel's collision deferral
  double *dcen, *acc, *dstep;  // census distance left, pending deposit, deposits flushed
  uint32_t *nf_s, *nc_s, *seq_s;   // facets, collisions, flush records so far this step
  int64_t *gid;                // global id (RNG key); = first_id + local index unless slabs
};

// Array-of-structures particle record (the particle_layout 1 ablation, §VI-D: the
// paper measured SoA vs AoS on CPUs only; on its GPU it used SoA).  Same fields as Soa
// (without the global id), 128 B per particle.
struct ParticleAoS {
  double x, y, ox, oy, e, w, mfp, dep, dcen, acc, dstep;
  int32_t cx, cy;
  uint32_t ctr, nfac, ncol, ncen, nf_s, nc_s, seq_s;
  uint8_t status;
  uint8_t pad[3];
};
static_assert(sizeof(ParticleAoS) == 128, "AoS record size");

// A particle migrating between x-slabs (decomposition 1): its store fields plus the
// mid-step state of a parked particle.
struct SlabRec {
  int64_t gid;
  double x, y, ox, oy, e, w, mfp, dcen, acc, dstep, dep;
  int32_t cx, cy;
  uint32_t ctr, nf, nc, seq, nfac, ncol, ncen, pad;
};

// Density storage (lossless): the f64 map, or -- when the map holds <= 256 (65536) distinct
// values -- a u8 (u16) material code per cell plus a table of each code's number density
// rho_k * cn (the product DESIGN.md §3 forms first, computed on the host with the same
// single rounding).  Either way the kernel obtains nd = rho[cell] * cn bit-identically.
enum DensFmt { kDensF64 = 0, kDensU16 = 1, kDensU8 = 2 };

struct Mesh {
  const double* __restrict__ rho;     // [ny][nx] kg/m^3            (kDensF64)
  const uint8_t* __restrict__ rho8;   // [ny][nx] material code     (kDensU8)
  const uint16_t* __restrict__ rho16; // [ny][nx] material code     (kDensU16)
  const double* __restrict__ nd_tab;  // [codes] rho_k * cn, atoms/m^3
  double* __restrict__ tally;         // [ny][nx] eV*weight
  const double* __restrict__ ex;      // [gnx+1] edge(i) = (i*W)/gnx
  const double* __restrict__ ey;      // [ny+1]
  int32_t nx, ny;                     // cells in storage (the columns this rank holds x rows)
  int32_t gnx;                        // cells per row of the whole mesh (reflection bound)
  int32_t x0;                         // whole-mesh column of storage column 0 (x-slabs: the
                                      // rank's first column minus a one-column halo; else 0)
  double wx, wy;                      // mesh extents W, H: edge(i) = (i*W)/gnx in place of a
                                      // load (bit-identical to ex[i], DESIGN.md §3 MESH)
  int32_t fmt, ncodes;
  int32_t tiled;                      // 1: 4x4-cell tiles (one 128 B tally line per tile)
  int32_t ntx;                        // tiles per row = ceil(nx / 4)
  // Block map (kDensU8 only, lossless): blocks of 2^bshift x 2^bshift cells, row-major
  // [nby][nbx]; entry = the block's material code when every cell of the block has that
  // code, kBlkMixed otherwise.  The history kernel keeps it in shared memory, so a facet
  // into a uniform block needs no global gather.  blk == nullptr: no block map.
  const uint8_t* __restrict__ blk;
  int32_t bshift, nbx, nblk;
  int32_t strip;                      // 16 * ntx: cells per row of tiles (tiled layout)
};

constexpr uint32_t kBlkMixed = 255u;   // block-map entry: block holds more than one code

// NT_CHECKS (dev variant, scripts/gpu_r02_chk.sh): device-side bounds checks of the indices
// the kernels compute -- storage cells, table buckets, queue and ring positions -- run under
// the GPU parity suite in place of compute-sanitizer (closed on this pool).
#ifndef NT_CHECKS
#define NT_CHECKS 0
#endif
#if NT_CHECKS
#include <cassert>
#define NT_CHECK(c) assert(c)
#else
#define NT_CHECK(c) ((void)0)
#endif
__device__ __forceinline__ uint32_t storage_cells(const Mesh& M) {
  return M.tiled ? (uint32_t)M.strip * (uint32_t)((M.ny + 3) / 4) : (uint32_t)M.nx * (uint32_t)M.ny;
}
constexpr int kBlkMax = 16384;         // max block-map entries (bytes of shared memory)

// Storage index of cell (cx, cy) in the tally and density arrays.  Tiled layout: 4x4-cell
// tiles in row-major tile order, column-major inside a tile -- index
// (cy/4)*(16*ntx) + 4*cx + cy%4 -- so the 16 f64 tally cells of a tile fill one 128 B line
// and a particle's consecutive facets (x or y) mostly stay in it; the index costs one shift
// and two integer multiply-adds.
// kOff (x-slab storage): cx is a whole-mesh column, the storage column is cx - x0; without
// it cx is the storage column (x0 = 0: replicated meshes and mesh preparation).
template <bool kOff = false>
__device__ __forceinline__ int64_t cell_index(const Mesh& M, int32_t cx, int32_t cy) {
  const int64_t lx = kOff ? (int64_t)(cx - M.x0) : (int64_t)cx;
  if (M.tiled)
    return (int64_t)(cy >> 2) * (16 * (int64_t)M.ntx) + (lx << 2) + (int64_t)(cy & 3);
  return (int64_t)cy * M.nx + lx;
}

// One microscopic cross-section table with its bucket index: bucket b covers the IEEE bit
// patterns [base + (b << shift), base + ((b+1) << shift)) of positive energies (monotone in
// the value), and idx[b] is the bin holding the bucket's first value, so the bin of any
// energy in bucket b lies in [idx[b], idx[b+1]].  nb = 0 disables the index (keys <= 0).
struct Table {
  const double* __restrict__ k;     // keys, eV, strictly increasing
  const double* __restrict__ v;     // values, barns
  const double2* __restrict__ kv;   // (k[i], v[i]) interleaved, [n + 1] (last entry repeats
                                    // n - 1): one 48 B run holds the two bins a bucket spans
  const uint32_t* __restrict__ idx; // [nb + 1]
  const double2* __restrict__ row;  // xs_search 0/4: per bucket b the three pairs kv[idx[b]],
                                    // kv[idx[b] + 1], kv[idx[b] + 2] (48 B), or nullptr
  uint64_t base;
  int32_t n, nb, shift, pad;
  double kfirst, klast;             // k[0] and k[n-1], as kernel parameters (no load latency)
};

struct Tables {
  Table s;   // scatter
  Table c;   // capture
  // xs_search 0, unionised grid: one bucket index over both tables' keys (bucket b covers
  // the bit patterns [ubase + (b << ushift), ...)); row b = the three scatter pairs, then the
  // three capture pairs its energies can need (96 B), or urow == nullptr
  const double2* __restrict__ urow;
  uint64_t ubase;
  int32_t ushift, unb;
  double ulast;               // min(klast of both tables): energies below it use urow
};

// Sub-expressions of DESIGN.md §3 that depend only on run constants.  Each is computed
// on the host with exactly the parenthesisation §3 writes, so using the stored value
// rounds identically to evaluating it in place.
struct Phys {
  double A;        // A
  double AA;       // A*A
  double twoA;     // 2.0*A
  double Ap1;      // A + 1.0
  double Am1;      // A - 1.0
  double Ap1sq;    // (A + 1.0)*(A + 1.0)
  double f;        // (A*A + 1.0) / ((A + 1.0)*(A + 1.0))
  double cn;       // N_A / M
  double kv;       // (2.0*EV) / M_N
  double e_min, w_min;
  double w_roul;   // roulette survivor weight
  int32_t vacuum;  // physics variants (R30-R32): vacuum boundary,
  int32_t analog;  //   sampled absorption,
  int32_t roulette;//   Russian roulette
  int32_t pad;
};

// Step statistics slots (u64 and f64 arrays in global memory).
enum StatU { SU_ALIVE = 0, SU_FACETS, SU_COLLISIONS, SU_CENSUS, SU_KILLED, SU_XS_RANGE,
             SU_NONFINITE, SU_EVENT_CAP, SU_REC_OVERFLOW, SU_ESCAPED, SU_ABSORBED, SU_COUNT };
enum StatF { SF_TALLY = 0, SF_CENSUS_E, SF_CENSUS_W, SF_KILLED_E, SF_KILLED_W,
             SF_ABSORBED_W, SF_ESCAPED_E, SF_ESCAPED_W, SF_ABSORBED_E, SF_ROULETTE, SF_COUNT };

// ---- Threefry-2x64-20 (Random123 Threefry) -----------------------------------
__device__ __forceinline__ uint64_t rotl64(uint64_t x, int r) {
  return (x << r) | (x >> (64 - r));
}

struct U64x2 { uint64_t a, b; };

__device__ __forceinline__ U64x2 threefry2x64_20(uint64_t c0, uint64_t c1, uint64_t k0,
                                                 uint64_t k1) {
  const uint64_t k2 = 0x1BD11BDAA9FC1A22ull ^ k0 ^ k1;
  const uint64_t ks[3] = {k0, k1, k2};
  constexpr int R[8] = {16, 42, 12, 31, 16, 32, 24, 21};
  uint64_t x0 = c0 + k0, x1 = c1 + k1;
#pragma unroll
  for (int r = 0; r < 20; ++r) {
    x0 += x1;
    x1 = rotl64(x1, R[r & 7]);
    x1 ^= x0;
    if ((r & 3) == 3) {
      const int s = (r + 1) >> 2;
      x0 += ks[s % 3];
      x1 += ks[(s + 1) % 3] + (uint64_t)s;
    }
  }
  return {x0, x1};
}

// u(x) = ((x >> 11) | 1) * 2^-53 : odd multiple of 2^-53, exact (R13)
__device__ __forceinline__ double u01(uint64_t x) {
  return (double)((x >> 11) | 1ull) * 0x1.0p-53;
}

// ---- mesh --------------------------------------------------------------------------------
// The unique i in [0,n-1] with edge[i] <= q < edge[i+1] (q >= edge[n] -> n-1), from a guess.
__device__ __forceinline__ int32_t cell_of(double q, const double* __restrict__ edge,
                                           int32_t n, double extent) {
  if (!(q >= 0.0)) return 0;
  if (q >= edge[n]) return n - 1;
  int32_t i = (int32_t)(q / extent * (double)n);
  i = i < 0 ? 0 : (i > n - 1 ? n - 1 : i);
  while (i > 0 && edge[i] > q) --i;
  while (i < n - 1 && edge[i + 1] <= q) ++i;
  return i;
}

// Number density of a cell: rho[cell] * cn.
template <int kFmt>
__device__ __forceinline__ double number_density(const Mesh& M, const double* __restrict__ tab,
                                                 int64_t cell, double cn) {
  if constexpr (kFmt == kDensU8) {
    return tab[__ldg(M.rho8 + cell)];
  } else if constexpr (kFmt == kDensU16) {
    return __ldg(tab + __ldg(M.rho16 + cell));
  } else {
    return __ldg(M.rho + cell) * cn;
  }
}

// max(v, 0) on the sign bit: +0 for negative v and -0 (R28: differs from
// v > 0 ? v : 0 only for a NaN with the sign bit clear, which stays NaN).
__device__ __forceinline__ double clamp0(double v) {
  const long long b = __double_as_longlong(v);
  return __longlong_as_double(b & ~(b >> 63));
}

// ---- L2 residency hints ----------------------------------------------------------------
// The tally (128 MB at 4000^2) and the density map compete for the 126 MB L2 with the
// particle store, which is read and written once per step: tally REDs and density gathers
// carry an evict_last policy, particle-store traffic evict_first.
__device__ __forceinline__ uint64_t l2_evict_last() {
  uint64_t p;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
  return p;
}
__device__ __forceinline__ uint64_t l2_evict_first() {
  uint64_t p;
  asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
  return p;
}
// The tally is never read by the tracking kernels, so the RED needs no "memory" clobber:
// without it the compiler may schedule the particle's other loads and stores across the
// flush (NT_RED_CLOBBER=1 restores the compiler barrier; A/B option).
#ifndef NT_RED_CLOBBER
#define NT_RED_CLOBBER 0
#endif
__device__ __forceinline__ void red_add_hint(double* a, double v, uint64_t pol) {
#if NT_RED_CLOBBER
  asm volatile("red.global.add.L2::cache_hint.f64 [%0], %1, %2;" ::"l"(a), "d"(v), "l"(pol)
               : "memory");
#else
  asm volatile("red.global.add.L2::cache_hint.f64 [%0], %1, %2;" ::"l"(a), "d"(v), "l"(pol));
#endif
}
// Fire-and-forget adds to locations a single thread owns (a particle's ledgers, a thread's
// statistic slots): no load on the critical path at the end of a history.  A thread's own
// adds to one address apply in program order, so the sums round as the load-add-store did.
__device__ __forceinline__ void red_add_f64(double* a, double v) {
  asm volatile("red.global.add.f64 [%0], %1;" ::"l"(a), "d"(v));
}
__device__ __forceinline__ void red_add_u32(uint32_t* a, uint32_t v) {
  asm volatile("red.global.add.u32 [%0], %1;" ::"l"(a), "r"(v));
}
// Warp-aggregated flush (tally_mode 1): the lanes executing this call that flush into the
// same cell are grouped with __match_any_sync; the group's lowest lane adds the group's
// values (its own first, then the others in lane order) and issues the one RED.  Lanes
// without a peer (the usual case away from hot spots) take the plain RED after one vote.
__device__ __forceinline__ void red_add_warp(double* tally, uint32_t cell, double v, uint64_t pol) {
  const unsigned act = __activemask();
  const unsigned peers = __match_any_sync(act, cell);
  const unsigned gmax = __reduce_max_sync(act, (unsigned)__popc(peers));
  if (gmax > 1u) {
    const int lane = threadIdx.x & 31;
    const unsigned g = (unsigned)__popc(peers);
    const bool leader = (__ffs(peers) - 1) == lane;
    double sum = v;
    for (unsigned k = 1; k < gmax; ++k) {
      const int src = k < g ? (int)__fns(peers, 0, (int)k + 1) : lane;
      const double o = __shfl_sync(act, v, src);
      if (leader && k < g) sum += o;
    }
    if (leader) red_add_hint(tally + cell, sum, pol);
  } else {
    red_add_hint(tally + cell, v, pol);
  }
}

__device__ __forceinline__ uint32_t ldg_u8_hint(const uint8_t* p, uint64_t pol) {
  unsigned short v;
  asm volatile("ld.global.nc.L2::cache_hint.u8 %0, [%1], %2;" : "=h"(v) : "l"(p), "l"(pol));
  return v;
}
template <class T>
__device__ __forceinline__ T ld_stream(const T* p, uint64_t pol);
template <>
__device__ __forceinline__ double ld_stream<double>(const double* p, uint64_t pol) {
  double v;
  asm volatile("ld.global.L1::no_allocate.L2::cache_hint.f64 %0, [%1], %2;"
               : "=d"(v) : "l"(p), "l"(pol));
  return v;
}
template <>
__device__ __forceinline__ int32_t ld_stream<int32_t>(const int32_t* p, uint64_t pol) {
  int32_t v;
  asm volatile("ld.global.L1::no_allocate.L2::cache_hint.s32 %0, [%1], %2;"
               : "=r"(v) : "l"(p), "l"(pol));
  return v;
}
template <>
__device__ __forceinline__ uint32_t ld_stream<uint32_t>(const uint32_t* p, uint64_t pol) {
  uint32_t v;
  asm volatile("ld.global.L1::no_allocate.L2::cache_hint.u32 %0, [%1], %2;"
               : "=r"(v) : "l"(p), "l"(pol));
  return v;
}
__device__ __forceinline__ void st_stream(double* p, double v, uint64_t pol) {
  asm volatile("st.global.L2::cache_hint.f64 [%0], %1, %2;" ::"l"(p), "d"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void st_stream(int32_t* p, int32_t v, uint64_t pol) {
  asm volatile("st.global.L2::cache_hint.s32 [%0], %1, %2;" ::"l"(p), "r"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void st_stream(uint32_t* p, uint32_t v, uint64_t pol) {
  asm volatile("st.global.L2::cache_hint.u32 [%0], %1, %2;" ::"l"(p), "r"(v), "l"(pol) : "memory");
}

// Split form of number_density for latency hiding: dens_load issues the gather (raw code or
// raw density), dens_nd consumes it later -- the history kernel issues the load at a facet
// and consumes it at the start of the next event, so the gather overlaps the loop overhead.
template <int kFmt> struct DensRaw { using type = uint32_t; };
template <> struct DensRaw<kDensF64> { using type = double; };

template <int kFmt>
__device__ __forceinline__ typename DensRaw<kFmt>::type dens_load(const Mesh& M, uint32_t cell,
                                                                  uint64_t pol) {
  if constexpr (kFmt == kDensU8) return ldg_u8_hint(M.rho8 + cell, pol);
  else if constexpr (kFmt == kDensU16) return (uint32_t)__ldg(M.rho16 + cell);
  else return __ldg(M.rho + cell);
}

// u8 code of cell (cx, cy) via the shared-memory block map: the block's code when the block
// is uniform, else the cell's own code from the global map (storage index cidx).
template <bool kOff = false>
__device__ __forceinline__ uint32_t dens_load_blk(const Mesh& M, const uint8_t* s_blk,
                                                  int32_t cx, int32_t cy, uint32_t cidx,
                                                  uint64_t pol) {
  const int32_t lx = kOff ? cx - M.x0 : cx;
  uint32_t code = s_blk[(cy >> M.bshift) * M.nbx + (lx >> M.bshift)];
  if (code == kBlkMixed) code = ldg_u8_hint(M.rho8 + cidx, pol);
  return code;
}

// Cross-CTA hand-over within one launch (fused phases): volatile / L2-only accesses.
// cp.async (Ampere+ LDGSTS): 16 bytes global -> shared, L2 only (.cg), completion tracked per
// thread by commit groups
__device__ __forceinline__ void cp_async16(void* smem, const void* gmem) {
  const unsigned sa = (unsigned)__cvta_generic_to_shared(smem);
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" :: "r"(sa), "l"(gmem) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
__device__ __forceinline__ void cp_async_wait_all() { asm volatile("cp.async.wait_all;" ::: "memory"); }
__device__ __forceinline__ void cp_async_wait_group1() { asm volatile("cp.async.wait_group 1;" ::: "memory"); }

__device__ __forceinline__ uint32_t ld_volatile_u8(const uint8_t* p) {
  uint32_t v;
  asm volatile("ld.volatile.global.u8 %0, [%1];" : "=r"(v) : "l"(p));
  return v;
}
__device__ __forceinline__ int32_t ld_volatile(const int32_t* p) {
  return *reinterpret_cast<const volatile int32_t*>(p);
}
__device__ __forceinline__ uint32_t ld_volatile(const unsigned int* p) {
  return *reinterpret_cast<const volatile unsigned int*>(p);
}
__device__ __forceinline__ unsigned long long ld_volatile(const unsigned long long* p) {
  return *reinterpret_cast<const volatile unsigned long long*>(p);
}
__device__ __forceinline__ void st_volatile(int32_t* p, int32_t v) {
  *reinterpret_cast<volatile int32_t*>(p) = v;
}

__device__ __forceinline__ void prefetch_l1(const void* p) {
  asm volatile("prefetch.global.L1 [%0];" ::"l"(p));
}

template <int kFmt>
__device__ __forceinline__ void dens_prefetch(const Mesh& M, int64_t cell) {
  if constexpr (kFmt == kDensU8) prefetch_l1(M.rho8 + cell);
  else if constexpr (kFmt == kDensU16) prefetch_l1(M.rho16 + cell);
  else prefetch_l1(M.rho + cell);
}

template <int kFmt>
__device__ __forceinline__ double dens_nd(typename DensRaw<kFmt>::type raw,
                                          const double* __restrict__ tab, double cn) {
  if constexpr (kFmt == kDensU8) return tab[raw];
  else if constexpr (kFmt == kDensU16) return __ldg(tab + raw);
  else return raw * cn;
}

// ---- microscopic cross sections -----------------------------------------------
// Table loads.  NT_XS_HINT=1 (A/B option) gives them an L2 evict_last policy, the priority
// of the tally lines, so the 128 MB tally cannot push the (~5 MB) tables out of L2.
#ifndef NT_XS_HINT
#define NT_XS_HINT 0
#endif
__device__ __forceinline__ double2 xs_ld2(const double2* p) {
#if NT_XS_HINT
  double2 v;
  asm volatile("{ .reg .b64 pol; createpolicy.fractional.L2::evict_last.b64 pol, 1.0;\n\t"
               "ld.global.nc.L2::cache_hint.v2.f64 {%0, %1}, [%2], pol; }"
               : "=d"(v.x), "=d"(v.y) : "l"(p));
  return v;
#else
  return __ldg(p);
#endif
}
__device__ __forceinline__ uint32_t xs_ldu(const uint32_t* p) {
#if NT_XS_HINT
  uint32_t v;
  asm volatile("{ .reg .b64 pol; createpolicy.fractional.L2::evict_last.b64 pol, 1.0;\n\t"
               "ld.global.nc.L2::cache_hint.u32 %0, [%1], pol; }" : "=r"(v) : "l"(p));
  return v;
#else
  return __ldg(p);
#endif
}

// Bin i = max{i in [0,N-2]: k[i] <= e} for e already in [k0, k_{N-1}] (the energy-bin
// search), then linear interpolation.  The bucket index is fine enough (about four buckets
// per key, nt_load_cross_sections) that a bucket nearly always spans at most one key: then
// the bin is idx[b] or idx[b] + 1, decided by one compare against k[idx[b] + 1], and the
// three (key, value) pairs that can be needed come from one 48 B run of the interleaved
// table -- two dependent loads per lookup (the index pair, then the run).  A bucket holding
// more keys falls back to a binary search inside it.  Same bin as a full binary search by
// construction.
// Split in two so a caller can issue the first dependent load (the bucket's index pair)
// early and finish the lookup later: xs_begin (bin bounds) and xs_end (pairs + lerp).
struct XsPre {
  double e;
  int32_t lo, hi;                             // k[lo] <= e < k[hi]
};
__device__ __forceinline__ XsPre xs_begin(const Table& T, double e) {
  XsPre r;
  r.e = e;
  if (e >= T.klast) {
    r.lo = T.n - 2;
    r.hi = T.n - 1;
  } else if (T.nb > 0) {
    const uint64_t b = ((uint64_t)__double_as_longlong(e) - T.base) >> T.shift;
    NT_CHECK(b < (uint64_t)T.nb);
    r.lo = (int32_t)xs_ldu(T.idx + b);
    r.hi = (int32_t)xs_ldu(T.idx + b + 1) + 1;
  } else {
    r.lo = 0;
    r.hi = T.n - 1;
  }
  return r;
}

__device__ __forceinline__ double xs_end(const Table& T, XsPre r) {
  const double e = r.e;
  int32_t lo = r.lo, hi = r.hi;
  double k0, k1, v0, v1;
  if (hi - lo <= 2) {
    const double2 a = xs_ld2(T.kv + lo), b = xs_ld2(T.kv + lo + 1), c = xs_ld2(T.kv + lo + 2);
    const bool up = hi - lo == 2 && b.x <= e;
    k0 = up ? b.x : a.x;
    v0 = up ? b.y : a.y;
    k1 = up ? c.x : b.x;
    v1 = up ? c.y : b.y;
  } else {
    while (hi - lo > 1) {
      const int32_t mid = (lo + hi) >> 1;
      if (__ldg(T.k + mid) <= e) lo = mid; else hi = mid;
    }
    const double2 a = __ldg(T.kv + lo), b = __ldg(T.kv + lo + 1);
    k0 = a.x;
    v0 = a.y;
    k1 = b.x;
    v1 = b.y;
  }
  const double t = (e - k0) / (k1 - k0);
  return v0 + t * (v1 - v0);
}

// Direct bucket rows (xs_search 4, and 0 where the unionised grid does not apply): the loader copies, for every bucket b, the three pairs a
// bucket spanning at most one key can need into row[3b .. 3b+2], and builds rows only when
// every bucket spans at most one key.  Then the lookup is ONE dependent load (the 48 B row)
// instead of two (the index pair, then the run): the index and the pairs are "staged" into
// one L2-resident structure addressed by the energy's bits (scatter history 8.26 -> 7.42 ms,
// scatter event 17.8 -> 15.4 ms; profiles/ab/r02_ab19_xs_rows.txt).  Same bin and the same
// lerp expression as xs_end, hence the same result.
__device__ __forceinline__ double xs_row(const Table& T, double e) {
  const uint64_t b = ((uint64_t)__double_as_longlong(e) - T.base) >> T.shift;
  NT_CHECK(b < (uint64_t)T.nb);
  const double2* r = T.row + 3 * b;
  const double2 a = __ldg(r), m = __ldg(r + 1), c = __ldg(r + 2);
  const bool up = m.x <= e;
  const double k0 = up ? m.x : a.x, v0 = up ? m.y : a.y;
  const double k1 = up ? c.x : m.x, v1 = up ? c.y : m.y;
  const double t = (e - k0) / (k1 - k0);
  return v0 + t * (v1 - v0);
}

__device__ __forceinline__ double xs_lookup(const Table& T, double e) {
  if (T.row != nullptr && e < T.klast) return xs_row(T, e);   // uniform branch (kernel param)
  return xs_end(T, xs_begin(T, e));
}

struct Mat {
  double st;   // (sigma_s + sigma_a) * barn, m^2
  double pa;   // sigma_a / sigma_t
  double H;    // E - (sigma_s/sigma_t) * (E*f): expected heating response
};

__device__ __forceinline__ double clamp_count(double e, const Table& T, uint32_t& nrange) {
  if (e < T.kfirst) { ++nrange; return T.kfirst; }
  if (e > T.klast) { ++nrange; return T.klast; }
  return e;
}

// refresh_xs in two halves (the XS-range count of the clamps is returned by the first and
// committed by the caller only if the refresh is used)
struct MatPre {
  XsPre s, c;
  double e;
  uint32_t nr;
};
__device__ __forceinline__ MatPre refresh_begin(const Tables& T, double e) {
  MatPre p;
  p.nr = 0;
  p.e = e;
  p.s = xs_begin(T.s, clamp_count(e, T.s, p.nr));
  p.c = xs_begin(T.c, clamp_count(e, T.c, p.nr));
  return p;
}

// one row of the unionised grid: the same bin selection and lerp as xs_row, per table
__device__ __forceinline__ double xs_urow_lerp(const double2* r, double e) {
  const double2 a = __ldg(r), m = __ldg(r + 1), c = __ldg(r + 2);
  const bool up = m.x <= e;
  const double k0 = up ? m.x : a.x, v0 = up ? m.y : a.y;
  const double k1 = up ? c.x : m.x, v1 = up ? c.y : m.y;
  const double t = (e - k0) / (k1 - k0);
  return v0 + t * (v1 - v0);
}

__device__ __forceinline__ Mat refresh_xs(const Tables& T, const Phys& ph, double e,
                                          uint32_t& nrange) {
  const double es = clamp_count(e, T.s, nrange);
  const double ea = clamp_count(e, T.c, nrange);
  double ss, sa;
  if (T.urow != nullptr && es == ea && es < T.ulast) {     // uniform branch on T.urow
    const uint64_t b = ((uint64_t)__double_as_longlong(es) - T.ubase) >> T.ushift;
    NT_CHECK(b < (uint64_t)T.unb);
    const double2* r = T.urow + 6 * b;
    ss = xs_urow_lerp(r, es);
    sa = xs_urow_lerp(r + 3, ea);
  } else {
    ss = xs_lookup(T.s, es);
    sa = xs_lookup(T.c, ea);
  }
  const double t = ss + sa;
  Mat m;
  m.st = t * kBarn;
  m.pa = t > 0.0 ? sa / t : 0.0;
  const double rs = t > 0.0 ? ss / t : 0.0;
  m.H = e - rs * (e * ph.f);
  return m;
}

__device__ __forceinline__ Mat refresh_end(const Tables& T, const Phys& ph, const MatPre& p) {
  const double ss = xs_end(T.s, p.s);
  const double sa = xs_end(T.c, p.c);
  const double t = ss + sa;
  const double e = p.e;
  Mat m;
  m.st = t * kBarn;
  m.pa = t > 0.0 ? sa / t : 0.0;
  const double rs = t > 0.0 ? ss / t : 0.0;
  m.H = e - rs * (e * ph.f);
  return m;
}

// ---- the paper's cached-index search: the bin of the last lookup is kept and
// the new bin is found by a linear walk from it (energies only fall in elastic scatter
// off a target at rest, so the walk goes down).  Same bin as xs_lookup by definition.
__device__ __forceinline__ double clamp_only(double e, const Table& T) {
  return e < T.kfirst ? T.kfirst : (e > T.klast ? T.klast : e);
}

// Bin of e (already in [k0, k_{N-1}]) by the bucketed binary search of xs_lookup.
__device__ __forceinline__ int32_t xs_bin(const Table& T, double e) {
  const double* __restrict__ k = T.k;
  const int32_t n = T.n;
  if (e >= T.klast) return n - 2;
  int32_t lo = 0, hi = n - 1;
  if (T.nb > 0) {
    const uint64_t b = ((uint64_t)__double_as_longlong(e) - T.base) >> T.shift;
    lo = (int32_t)__ldg(T.idx + b);
    hi = (int32_t)__ldg(T.idx + b + 1) + 1;
  }
  while (hi - lo > 1) {
    const int32_t mid = (lo + hi) >> 1;
    if (__ldg(k + mid) <= e) lo = mid; else hi = mid;
  }
  return lo;
}

__device__ __forceinline__ double xs_walk(const Table& T, double e, int32_t& bin) {
  const double* __restrict__ k = T.k;
  int32_t i = bin;
  while (i > 0 && __ldg(k + i) > e) --i;
  while (i < T.n - 2 && __ldg(k + i + 1) <= e) ++i;
  bin = i;
  const double k0 = __ldg(k + i), k1 = __ldg(k + i + 1);
  const double v0 = __ldg(T.v + i), v1 = __ldg(T.v + i + 1);
  const double t = (e - k0) / (k1 - k0);
  return v0 + t * (v1 - v0);
}

__device__ __forceinline__ Mat refresh_xs_walk(const Tables& T, const Phys& ph, double e,
                                               uint32_t& nrange, int32_t& bin_s, int32_t& bin_a) {
  const double es = clamp_count(e, T.s, nrange);
  const double ea = clamp_count(e, T.c, nrange);
  const double ss = xs_walk(T.s, es, bin_s);
  const double sa = xs_walk(T.c, ea, bin_a);
  const double t = ss + sa;
  Mat m;
  m.st = t * kBarn;
  m.pa = t > 0.0 ? sa / t : 0.0;
  const double rs = t > 0.0 ? ss / t : 0.0;
  m.H = e - rs * (e * ph.f);
  return m;
}

__device__ __forceinline__ double speed(double e, const Phys& ph) {
  return sqrt(e * ph.kv);
}

}  // namespace nt
