// nt_internal.h -- kernel parameter blocks and launchers shared by the runtime (nt_api.cu)
// and the kernel translation units.  Not part of the public ABI.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "nt_device.cuh"

namespace nt {

struct TrackParams {
  Mesh mesh;
  Tables xs;
  Phys ph;
  Soa p;
  ParticleAoS* aos;           // particle_layout 1: the AoS copy the history kernel works on
  int64_t n;                  // local particles
  int64_t lo, hi;             // local index range processed by this launch
  int64_t first_id;           // global id of local index 0
  uint64_t seed;
  double dt;
  int64_t max_events;
  int32_t refill_min;         // refill a warp's idle lanes once at least this many are idle
  // history kernel regime parking
  int32_t phase;              // 1: track [lo, hi) (resume_q null); 2: resume resume_q
  int32_t park_coll_below;    // park a colliding lane while fewer lanes of its warp collide
  const int32_t* resume_q;
  const unsigned long long* resume_count;
  int32_t* park_q;            // out-queue of parked local indices
  unsigned long long* park_count;
  // resume_prefetch (kQ kernels): parks write queue-ordered records (kParkF64 f64 columns,
  // then kParkU32 u32 columns, park_cap entries each) instead of the particle store + queue
  // index; phase 2 streams them into a per-warp shared-memory ring with cp.async
  double* park_rec;
  int64_t park_cap;
  // fused phases (fused_consumers > 0): one launch; CTAs [0, coll_ctas) start as consumers
  // of park_q (entries published as index + 1 after a fence), the others produce (phase 1)
  // and turn consumer when their range is exhausted
  int32_t coll_ctas;
  uint32_t n_prod;                  // producer warps
  unsigned long long* park_taken;   // park_q entries claimed by consumers
  unsigned int* prod_done;          // producer warps finished producing
  // x-slab decomposition (decomposition 1): particles leaving columns [slab_lo, slab_hi)
  int32_t slab_lo, slab_hi;
  int32_t* out_q;             // emigrant local indices
  unsigned long long* out_count;
  // tally_mode 3: the hot window of cells privatised in shared memory (whole-mesh columns)
  int32_t hot_x0, hot_y0, hot_nx, hot_ny;
  unsigned long long* counter;      // dynamic work counter (particles claimed)
  unsigned long long* stats_u;      // [SU_COUNT]
  double* stats_f;                  // [SF_COUNT]
  double* slot_f;                   // [SF_COUNT][grid * block] per-thread f64 statistic slots
  // deterministic-mode flush records (cell << 40 | (pid - lo) << 24 | seq, value)
  unsigned long long* rec_key;
  double* rec_val;
  unsigned long long* rec_count;
  unsigned long long rec_cap;
};

struct InjectParams {
  Soa p;
  const double* ex;
  const double* ey;
  int32_t nx, ny;
  double W, H;
  int64_t n_local, first_id;
  double sx, sy, sw, sh, e0;
  uint64_t seed;
};

// ---- launchers (nt_kernels.cu) ----------------------------------------------------------
void launch_edges(double* ex, int32_t nx, double W, double* ey, int32_t ny, double H,
                  cudaStream_t s);
void launch_inject(const InjectParams& ip, cudaStream_t s);
// History (Over Particles) tracking: grid = persistent CTAs.
// The density format (tp.mesh.fmt) and the storage layout (tp.mesh.tiled) select the
// instantiation; 128-thread CTAs with <= 80 registers (6 resident per SM), or -- minb = 7,
// production u8 + block map only -- <= 72 registers (7 per SM).
// tally_mode 1/2/3 (production u8 + block map only): warp-aggregated flushes / CAS-emulated
// fp64 add / shared-memory hot window (tp.hot_*).
// xs_search 2 (u8 + block map only): the cached-bin linear walk; 0, 1 and 3 are data
// changes (the caller passes tables with direct rows / without bucket index / index only).
void launch_history(const TrackParams& tp, bool det, int grid, int minb, int tally_mode,
                    int xs_search, bool slab, cudaStream_t s);
// particle_layout 1: copy the particle store SoA -> AoS (to_aos) or back, particles [0, n)
void launch_aos_copy(const Soa& p, ParticleAoS* aos, int64_t n, bool to_aos, cudaStream_t s);
// Slab decomposition: pack the emigrants (out_q[0, n)) into records, those left of slab_lo
// first (counter cnt[0]), the others from the end (cnt[1]); unpack n records into the slots
// free_slots[0, n_free) and then [base, ...), status 2, and queue them in arr_q.
void launch_slab_pack(const TrackParams& tp, const int32_t* out_q, int64_t n, SlabRec* dst,
                      unsigned long long* cnt, cudaStream_t s);
void launch_slab_unpack(const Soa& p, const SlabRec* src, int64_t n, const int32_t* free_slots,
                        int64_t n_free, int64_t base, int32_t* arr_q, cudaStream_t s);
int history_max_ctas_per_sm(bool det, int fmt, bool tiled, bool blk, int minb, int tally);
// cross-section tables on the device: the interleaved pairs kv [n + 1], the bucket index
// idx [nb + 1] (base, shift: the bucket of a bit pattern is (bits - base) >> shift) and the
// direct bucket rows [nb] (xs_search 0, 4; if rows); *wide |= 1 if a bucket spans more than one key
void launch_xs_prepare(const double* k, const double* v, int64_t n, uint64_t base, int shift,
                       int64_t nb, bool rows, uint32_t* idx, double2* kv, double2* row,
                       unsigned int* wide, cudaStream_t s);
// unionised grid (xs_search 0): row[6b .. 6b+5] = the scatter then capture pairs of union
// bucket b (nb buckets over bits base + (b << shift)); *wide |= 1 if unusable
void launch_xs_urows(const double* ks, const double2* kvs, int64_t ns, const double* kc,
                     const double2* kvc, int64_t nc, uint64_t base, int shift, int64_t nb,
                     double2* row, unsigned int* wide, cudaStream_t s);
// resident CTAs per SM of the resume_prefetch kernel with its ring (phase 2)
int history_ring_ctas_per_sm(bool tiled);
void launch_det_apply(const unsigned long long* keys, const double* vals,
                      unsigned long long n, double* tally, cudaStream_t s);
void launch_threefry_debug(const uint64_t* in, int64_t n, uint64_t* out, cudaStream_t s);
void launch_xs_debug(const Tables& T, const double* e, int64_t n, double* os, double* oa,
                     cudaStream_t s);
// CUB radix sort of (key, value) pairs; temp_bytes query when temp == nullptr.
cudaError_t sort_pairs(void* temp, size_t& temp_bytes, const unsigned long long* kin,
                       unsigned long long* kout, const double* vin, double* vout,
                       unsigned long long n, int end_bit, cudaStream_t s);

// Every device allocation of the library goes through device_malloc (nt_api.cu), which
// counts them: nt_debug_alloc_count lets the tests assert that a timestep allocates
// nothing once the context's buffers exist.
cudaError_t device_malloc(void** p, size_t bytes);
// out[k] = (double)su[k] for k < SU_COUNT, out[SU_COUNT + k] = sf[k] for k < SF_COUNT.
void launch_stats_to_f64(const unsigned long long* su, const double* sf, double* out,
                         cudaStream_t s);

constexpr int kHistoryBlock = 128;
// resume ring (history kernel, resume_prefetch): a parked record is 15 f64 (x, y, ox, oy,
// exn, eyn, E, w, n_mfp, census distance, acc, dstep, sigma_t, p_a, H) + 6 u32 (cx, cy, ctr,
// facets, collisions, local index) = 144 B; claims and copies move batches of kRingB
// records, and each warp holds two batches (one being consumed, one in flight).
constexpr int kParkF64 = 15, kParkU32 = 6, kRingB = 12;
constexpr int kRingHalfBytes = kRingB * (kParkF64 * 8 + kParkU32 * 4);     // 1728
constexpr int kRingCtaBytes = 2 * kRingHalfBytes * (kHistoryBlock / 32);   // 13824
constexpr int kHotCells = 2048;     // tally_mode 3: cells of the shared-memory hot window (16 KB)
// history kernel: events a lane may run between two warp votes (refill checks); the A/B
// sweep in profiles/ab/r01_ab4_history_variants.md chose 256
constexpr int kInnerEvents = 256;   // (also best for the parked-particle phase: ab9, ab10)

}  // namespace nt

namespace nt {
// Mesh preparation (nt_kernels.cu).
cudaError_t launch_density_check(const double* rho, int64_t n, unsigned long long* bad,
                                 cudaStream_t s);
// Validation + distinct values in one pass (a chunk of the density): bad[0] += invalid
// values, distinct bit patterns into the open-addressing set (kDistinctSlots u64, all ones =
// empty), bad[1] += patterns inserted, bad[2] = 1 once the set is half full.
constexpr int kDistinctSlots = 4096;
cudaError_t launch_check_distinct(const double* rho, int64_t n, unsigned long long* bad,
                                  unsigned long long* set, cudaStream_t s);
// The set's patterns sorted into uniq[0, count) (count <= kDistinctSlots / 2).
cudaError_t launch_distinct_sort(const unsigned long long* set, unsigned long long* uniq,
                                 cudaStream_t s);
// Sort the density bit patterns (k0 -> k1) and write the distinct ones to k0, their count to
// *d_count.  temp == nullptr: query temp_bytes.
cudaError_t density_distinct(const double* rho, int64_t n, unsigned long long* k0,
                             unsigned long long* k1, void* temp, size_t& temp_bytes,
                             int* d_count, cudaStream_t s);
cudaError_t launch_encode(const double* rho, int64_t n, const Mesh& M,
                          const unsigned long long* uniq, int nu, double cn, int fmt, void* code,
                          double* nd_tab, cudaStream_t s);
// Row-major [ny][nx] <-> the mesh's storage layout (cell_index).
// Block map (Mesh::blk) of the u8 code map: blk[by * nbx + bx] = the block's code if uniform,
// else kBlkMixed.  M.bshift / M.nbx / M.nblk describe the blocks.
cudaError_t launch_block_map(const uint8_t* code, const Mesh& M, uint8_t* blk, cudaStream_t s);
cudaError_t launch_relayout(const double* src, double* dst, int64_t n, const Mesh& M,
                            bool to_storage, cudaStream_t s);
}  // namespace nt
