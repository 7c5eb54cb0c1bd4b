/*
 * neutral_b200.h -- C ABI of the B200-native neutral particle-history tracker.
 *
 * The method is the Monte Carlo neutral-particle transport mini-app "neutral" of
 * Martineau & McIntosh-Smith, "Exploring On-Node Parallelism with Neutral, a Monte Carlo
 * Neutral Particle Transport Mini-App", IEEE CLUSTER 2017.  "P:L1-L2 (§X)" cites lines of
 * that paper's text.  The exact arithmetic is DESIGN.md §3; the readings of
 * the paper it relies on are DESIGN.md §4.
 *
 * Conventions for every call:
 *  - Every call returns nt_status; the library never aborts or exits.  On failure
 *    nt_last_error(ctx) holds a one-line message (storage owned by ctx).
 *  - Pointer arguments may be host or device memory (detected with
 *    cudaPointerGetAttributes, copied with cudaMemcpyDefault).  Inputs are deep-copied
 *    during the call: the caller keeps ownership and may free them on return.
 *  - All device memory belongs to the context and is released by nt_destroy.
 *  - All work is ordered on the context stream (the caller's stream if given).
 *    nt_run_timestep, nt_read_tally and nt_read_particles synchronise that stream
 *    before returning.
 *  - Call order (state machine): nt_create -> nt_init_mesh -> nt_load_cross_sections
 *    -> nt_inject_particles -> nt_run_timestep (repeatable) -> nt_read_*.
 *    Out-of-order calls return NT_ERR_STATE.  Re-running an earlier stage
 *    invalidates the later ones.
 *  - One context per host thread; contexts are independent.
 *  - Units: metres, seconds, kg/m^3, eV, barns.  The tally is eV x weight, raw.
 */
#ifndef NEUTRAL_B200_H
#define NEUTRAL_B200_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define NT_ABI_VERSION 5

typedef struct nt_ctx nt_ctx;

typedef enum {
    NT_OK = 0,
    NT_ERR_ARG = 1,        /* invalid argument (message says which)                   */
    NT_ERR_STATE = 2,      /* call out of order                                       */
    NT_ERR_OOM = 3,        /* device allocation failed                                */
    NT_ERR_CUDA = 4,       /* CUDA runtime error                                      */
    NT_ERR_NCCL = 5,       /* NCCL error (nranks > 1)                                 */
    NT_ERR_XS_RANGE = 6,   /* step completed; some energies were outside a table      */
    NT_ERR_NONFINITE = 7,  /* step completed; some particle ended non-finite          */
    NT_ERR_EVENT_CAP = 8,  /* step completed; some history hit max_events_per_history */
    NT_ERR_UNSUPPORTED = 9 /* feature not available in this build / configuration     */
} nt_status;

enum { NT_MODE_HISTORY = 0, NT_MODE_EVENT = 1 };

/* Context options.  Zero-initialise (or nt_options_default) and set what you need. */
typedef struct {
    int32_t device;            /* CUDA device ordinal                                     */
    void *stream;              /* cudaStream_t to order work on, or NULL = own stream     */
    int32_t mode;              /* NT_MODE_HISTORY: Over Particles (§V-A);
                                  NT_MODE_EVENT: Over Events (§V-B)             */
    int32_t deterministic;     /* 1: fixed-order tally = the oracle's (particle id, flush
                                  sequence) order per cell; 0: fp64 atomics   */
    int32_t rank, nranks;      /* this process's rank and the world size (0, 1 = 1 GPU)   */
    const void *nccl_unique_id;/* 128-byte ncclUniqueId (nt_get_unique_id on rank 0,
                                  broadcast by the caller); required when nranks > 1.  When
                                  given, the context joins that NCCL communicator and every
                                  timestep allreduces the tally and statistics (also for
                                  nranks == 1, which exercises the same path on one GPU)  */
    double A;                  /* target mass / neutron mass       (0 -> 1.0)            */
    double molar_mass;         /* kg/mol                           (0 -> 1e-3)           */
    double e_min;              /* energy cutoff, eV    (0 -> 1.0)            */
    double w_min;              /* weight cutoff        (0 -> 1e-3)           */
    int64_t max_events_per_history; /* guard per history per step  (0 -> 1e9)            */
    int32_t block_size;        /* threads per CTA of the tracking kernel (0 -> default)   */
    int32_t ctas_per_sm;       /* persistent CTAs per SM (0 -> occupancy maximum)         */
    int64_t det_batch;         /* deterministic mode: particles per batch (0 -> 65536)    */
    int32_t refill_min;        /* history mode: a warp refills its idle lanes once at least
                                  this many are idle (0 -> 4)                              */
    int32_t density_format;    /* 0: lossless u8/u16 material codes when the density map
                                  holds <= 256 / 65536 distinct values, else f64; with u8
                                  codes (<= 254 values) also a block map (the code of each
                                  uniform 2^k x 2^k-cell block, <= 16 KB) that the history
                                  kernel keeps in shared memory;
                                  1: always the f64 map;
                                  2: as 0 without the block map (ablation)                 */
    int32_t layout;            /* storage of the tally and density maps: 0: 4x4-cell tiles
                                  (a tile's 16 f64 tally cells = one 128 B line, so a
                                  particle's consecutive facets stay in few L2 lines);
                                  1: row-major.  nt_read_tally always returns row-major.  */
    int32_t tally_mode;        /* production tally flushes: 0: one fp64
                                  atomic add per flush; 1: warp-aggregated -- lanes flushing
                                  into the same cell at the same time are summed with warp
                                  shuffles and one lane issues the atomic; 2: the fp64 add
                                  emulated by a 64-bit compare-and-swap loop;
                                  3: a per-CTA shared-memory copy of the hot window
                                  hot_* (privatisation), merged with one atomic
                                  per cell when the CTA ends.  Ablations: history mode,
                                  production, u8 block-map meshes; others use 0.          */
    int32_t defer_below;       /* history mode, collision deferral: a lane whose next event
                                  is a collision while fewer than this many lanes of its
                                  warp collide is parked (state to the particle store) and
                                  resumed by a second launch of the tracking kernel, where
                                  such particles -- mostly inside dense matter -- collide
                                  together.  Results are unchanged.  0 -> 8; 1 disables;
                                  at most 33 (33: park every collision)                    */
    int32_t xs_search;         /* cross-section bin search: 0 (default)
                                  the unionised grid of 4 where built, else the direct rows
                                  of 4 per table; 4 direct bucket rows -- a bucket index
                                  over the keys' bit patterns (about four buckets per key)
                                  whose every bucket stores the three (key, value) pairs
                                  its energies can need, so a lookup is one dependent 48 B
                                  load (built when every bucket spans at most one key,
                                  else as 3); 1 plain binary
                                  search over the table; 2 the paper's cached-index search
                                  -- a linear walk from the particle's previous bin
                                  (history mode, u8 block-map meshes; others use 3); 3 the
                                  bucket index alone (the index pair, then the pairs: two
                                  dependent loads; a binary search inside buckets holding
                                  more than one key).  The unionised grid (0): one bucket
                                  index over both tables whose rows hold both tables' pairs
                                  (96 B), one bucket computation and one row per refresh
                                  (built when every bucket spans at most one key of each
                                  table).  All five return the same bin.                  */
    /* physics variants (DESIGN.md §4 R30-R32; the defaults are the paper's problem)      */
    int32_t boundary;          /* 0 reflective on all four sides; 1 vacuum: a
                                  facet on the mesh boundary ends the history (escape)     */
    int32_t analog_absorption; /* 0 implicit capture, w <- w (1 - p_a) at every collision
                                  (north star, R8); 1 the paper's two branches
                                  sampled: absorbed with probability p_a, else scattered
                                  with w unchanged (the scatter draws its n_mfp from the
                                  next RNG counter)                                        */
    int32_t roulette;          /* 0 a weight below w_min ends the history;
                                  1 Russian roulette: survive with probability
                                  w / roulette_weight at weight roulette_weight (one RNG
                                  counter)                                                 */
    int32_t decomposition;     /* 0: replicated mesh, particles split by global id, tally
                                  allreduced; 1: x-slabs (SURVEY §8(f) row
                                  1) -- rank r owns the mesh columns [floor(r nx/P),
                                  floor((r+1) nx/P)) and tracks the particles inside them;
                                  a particle crossing a slab edge migrates to the
                                  neighbour (nt_run_timestep exchanges them over NCCL, or
                                  the caller drives nt_slab_*).  Production tally only.   */
    double roulette_weight;    /* survivor weight (0 -> 2 w_min)                           */
    int32_t hot_x0, hot_y0;    /* tally_mode 3: first column and row of the hot window     */
    int32_t hot_nx, hot_ny;    /* its size in cells, hot_nx * hot_ny <= 2048 (16 KB)       */
    int32_t particle_layout;   /* 0: structure of arrays; 1: array of 128 B
                                  records while the history kernel runs (ablation, P:526-551;
                                  production tally, default kernel; others use 0)          */
    int32_t fused_consumers;   /* history mode, production: 0 runs the parked collisions in
                                  a second launch after phase 1 (the default); k > 0 fuses
                                  both phases into one launch: k - 1 CTAs per SM resume
                                  parked particles from the start, and every other warp
                                  turns to them as soon as the particle range is exhausted
                                  (its idle lanes resume parked particles while its last
                                  own histories still run).  Results are unchanged.  u8
                                  block-map meshes, default kernel options                */
    int32_t xs_l2_persist;     /* 1: while the tracking kernels run, an L2 access-policy
                                  window on the context stream marks the cross-section
                                  tables persisting (large lookup tables can
                                  become the bottleneck), with a device-wide persisting
                                  carve-out of up to the tables' size set at
                                  nt_load_cross_sections and released at nt_destroy (the
                                  limit is device-wide, and a window the caller had set on
                                  the same stream is replaced, then cleared);
                                  0: no window (default)                                  */
    int32_t resume_prefetch;   /* history mode, production, default kernel options: 1 a
                                  parked particle's state is written as a queue-ordered
                                  144 B record, and the second launch streams the records
                                  into a per-warp shared-memory ring with cp.async one
                                  batch ahead of use (refills of resumed particles read
                                  shared memory); 0 (default) the state goes to the
                                  particle store and a queue of indices.  Results are
                                  unchanged.  (Measured: 1 is 2% slower on csp and split,
                                  DESIGN.md §8.)                                          */
} nt_options;

/* Statistics of one timestep (sums over the particles this rank -- or, when nranks > 1,
 * all ranks -- tracked).  events = n_facets + n_collisions + n_census. */
typedef struct {
    uint64_t n_alive_start, n_facets, n_collisions, n_census, n_killed;
    double tally_total;        /* sum of all deposits flushed this step                  */
    double census_energy, census_weight;   /* sum of w*E, w over particles at census     */
    double killed_energy, killed_weight;   /* sum of w*E, w over particles killed        */
    double absorbed_weight;    /* weight removed by implicit capture          */
    uint64_t n_xs_range, n_nonfinite, n_event_cap;
    float track_ms;            /* device time of the tracking kernel(s)                   */
    float reduce_ms;           /* device time of the cross-GPU tally reduction            */
    float step_ms;             /* device time of the whole timestep                       */
    uint32_t n_launches;       /* kernels this library launched for the step              */
    uint64_t n_escaped;        /* histories ended at a vacuum boundary                    */
    uint64_t n_absorbed;       /* histories ended by a sampled absorption                 */
    double escaped_energy, escaped_weight;   /* sum of w*E, w over escaped particles       */
    double absorbed_energy;    /* sum of w*E of the absorbed particles (the track-length
                                  deposits already carry it in expectation)                */
    double roulette_gain;      /* weight added by roulette survivors: census + killed +
                                  absorbed + escaped weight = initial weight + gain        */
} nt_step_stats;

/* Structure-of-arrays particle view used by nt_read_particles / nt_write_particles.
 * Each pointer may be NULL (field skipped), a host pointer or a device pointer. */
typedef struct {
    double *x, *y;             /* position, m                                             */
    double *ox, *oy;           /* direction cosines                                       */
    double *e;                 /* energy, eV                                              */
    double *w;                 /* weight                                      */
    double *mfp;               /* mean free paths to the next collision                   */
    int32_t *cx, *cy;          /* containing cell                                         */
    uint32_t *ctr;             /* next RNG counter                            */
    uint8_t *status;           /* 1 alive (at census), 0 dead                             */
    uint32_t *nfac, *ncol, *ncen; /* cumulative facet / collision / census events         */
    double *dep;               /* cumulative energy this particle deposited in the tally  */
    int64_t *gid;              /* global particle id (the RNG key)             */
} nt_particles;

/* Library identity. */
int32_t nt_abi_version(void);
const char *nt_build_info(void);       /* compile flags, arch, det/fmad settings          */
const char *nt_status_string(nt_status s);

/* Fill *opt with the defaults listed above. */
nt_status nt_options_default(nt_options *opt);

/* Write a fresh 128-byte ncclUniqueId into out[128] (rank 0 only; for nranks > 1). */
nt_status nt_get_unique_id(void *out128);

/* Create a context on opt->device.  For nranks > 1 this joins the NCCL communicator
 * (collective over all ranks).  *out is NULL on failure. */
nt_status nt_create(const nt_options *opt, nt_ctx **out);
nt_status nt_destroy(nt_ctx *ctx);     /* NULL is a no-op                                 */
const char *nt_last_error(const nt_ctx *ctx); /* never NULL                               */

/* The structured 2D mesh of cell-centred mass densities:
 * nx x ny uniform cells over [0,width] x [0,height], density[ny][nx] row-major, kg/m^3,
 * finite and >= 0.  Cell edges are edge(i) = (i*width)/nx.  With x-slabs
 * (decomposition 1) every rank passes the whole map but stores -- and validates -- only
 * its columns [floor(r nx/P), floor((r+1) nx/P)) plus one halo column on each side; its
 * tally holds those columns too (nt_read_tally assembles the whole map). */
nt_status nt_init_mesh(nt_ctx *ctx, int32_t nx, int32_t ny, double width, double height,
                       const double *density);

/* The two microscopic cross-section tables of one material, scatter and capture
 * (§IV-D): keys in eV strictly increasing and finite, values in barns finite and
 * >= 0, n >= 2 each.  Lookup = bin search + linear interpolation. */
nt_status nt_load_cross_sections(nt_ctx *ctx,
                                 const double *scatter_keys, const double *scatter_vals,
                                 int64_t n_scatter,
                                 const double *capture_keys, const double *capture_vals,
                                 int64_t n_capture);

/* Create this rank's particles: global ids [first_id, first_id + n_local) of n_total,
 * positions uniform in the source rectangle [src_x, src_x+src_w] x [src_y, src_y+src_h]
 * (inside the mesh), isotropic directions, energy initial_energy, weight 1
 * (§IV-F).  Random numbers: Threefry-2x64-20 keyed by (global id, seed)
 * (P:296-300), so results do not depend on how ids are split across ranks. */
nt_status nt_inject_particles(nt_ctx *ctx, int64_t n_total, int64_t first_id,
                              int64_t n_local, double src_x, double src_y, double src_w,
                              double src_h, double initial_energy, uint64_t seed);

/* Track every alive particle for one timestep of length dt seconds until census or death
 * (Listing 1, or Listing 2 P:362-373 in event mode).  Zeroes the tally first
 * (the tally is per timestep), then accumulates every flushed deposit
 * (P:391-401).  When nranks > 1 the tally and stats are summed over ranks (NCCL
 * allreduce over NVLink) -- a collective call.  Device-side anomalies do not abort the
 * step: it completes, stats are filled, and the return is NT_ERR_XS_RANGE,
 * NT_ERR_NONFINITE or NT_ERR_EVENT_CAP.  stats may be NULL. */
nt_status nt_run_timestep(nt_ctx *ctx, double dt, nt_step_stats *stats);

/* Copy the per-cell tally [ny][nx] (f64) of the last step into dst (host or device).
 * reduced = 1: the cross-rank sum (equal to the local tally without a communicator);
 * reduced = 0: this rank's own partial tally.  With a communicator the step allreduces
 * out of place (local partial -> a second tally buffer), so both stay readable without a
 * copy. */
nt_status nt_read_tally(nt_ctx *ctx, double *dst, int32_t reduced);

/* Copy local particles [first, first+count) (local indices) into dst's arrays. */
nt_status nt_read_particles(nt_ctx *ctx, int64_t first, int64_t count,
                            const nt_particles *dst);
/* Overwrite local particles [first, first+count) from src (checkpoint / resume: the RNG
 * is counter based, so a restored particle continues bit-exactly). */
nt_status nt_write_particles(nt_ctx *ctx, int64_t first, int64_t count,
                             const nt_particles *src);

/* ---- slab decomposition driven by the caller (decomposition = 1) -------------------
 * One timestep = nt_slab_begin, then rounds until no rank has emigrants: nt_slab_round
 * tracks this rank's particles (the first round: its own; later rounds: the arrivals)
 * until census, death or a slab edge; nt_slab_export hands over the emigrants as packed
 * records (those leaving to the left first, n_left + n_right of them), which the caller
 * delivers to the neighbours' nt_slab_import; nt_slab_end returns this rank's statistics
 * (sum them over ranks; the tally is read with nt_read_tally(reduced = 0) and summed).
 * Per-particle results equal the replicated run's (the RNG is keyed by global id).
 * Local slots of emigrated particles keep status 4 (moved); arrivals are appended. */
int64_t   nt_slab_record_bytes(void);
nt_status nt_slab_begin(nt_ctx *ctx, double dt);
nt_status nt_slab_round(nt_ctx *ctx, int64_t *n_emigrants);
nt_status nt_slab_export(nt_ctx *ctx, void *dst, int64_t capacity, int64_t *n_left,
                         int64_t *n_right);
nt_status nt_slab_import(nt_ctx *ctx, const void *src, int64_t n);
nt_status nt_slab_end(nt_ctx *ctx, nt_step_stats *stats);
/* Local particle slots in use (the range nt_read_particles accepts): n_local at
 * injection, growing when slab arrivals find no free slot. */
nt_status nt_particle_slots(nt_ctx *ctx, int64_t *n_slots);

/* Verification entry points (run the device code paths in isolation). */
/* Device allocations the library has made so far, process-wide (every cudaMalloc goes
 * through one counter).  A timestep on a context whose buffers exist allocates nothing. */
int64_t nt_debug_alloc_count(void);
/* Device bytes the context holds for the mesh: density (f64 and codes, block map) and the
 * tally buffers.  With x-slabs (decomposition 1) only the rank's columns plus a one-column
 * halo are stored, so this scales as 1/nranks.  -1 for a NULL context. */
int64_t nt_debug_mesh_bytes(const nt_ctx *ctx);
/* Which loaded tables have direct bucket rows (xs_search 0): bit 0 scatter, bit 1 capture;
 * bit 2: the unionised grid (xs_search 4) was built; -1 for a NULL context. */
int32_t nt_debug_xs_rows(const nt_ctx *ctx);
/* The density storage nt_init_mesh chose: 2 u8 material codes, 1 u16 codes, 0 the f64 map
 * (-1 for a NULL context, or before nt_init_mesh); *n_distinct (if not NULL) = the number
 * of distinct density values found (0 for the f64 format without codes). */
int32_t nt_debug_density_format(const nt_ctx *ctx, int32_t *n_distinct);
/* out[2i], out[2i+1] = threefry2x64_20(ctr = {in[4i], in[4i+1]}, key = {in[4i+2], in[4i+3]}). */
nt_status nt_debug_threefry(nt_ctx *ctx, const uint64_t *in, int64_t n, uint64_t *out);
/* Microscopic XS from the loaded tables: out_s[i], out_a[i] at energies[i] (no clamp
 * counting). */
nt_status nt_debug_xs(nt_ctx *ctx, const double *energies, int64_t n, double *out_s,
                      double *out_a);

#ifdef __cplusplus
}
#endif
#endif /* NEUTRAL_B200_H */
