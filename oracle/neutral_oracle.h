/*
 * neutral_oracle.h -- plain, slow, single-threaded CPU oracle for the neutral
 * particle-history tracking loop (Martineau & McIntosh-Smith, CLUSTER 2017).
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load or call this library.  It shares
 * no code, header, constant table or helper with the CUDA product path
 * (paper_conf_cluster_martineaum17_b200/csrc); the two agree because both follow
 * DESIGN.md §3 (the algorithm as read from PAPER.md), not because they share text.
 *
 * Citations "P:L1-L2 (§X)" point into /root/reference/PAPER.md.
 *
 * Parity pins (tests/test_oracle_*.py): Threefry KATs (P1), u01 lattice (P2),
 * injection geometry (P3), vacuum closed form (P4), population (P5), flight
 * length law (P6), scatter kinematics / slowing-down law (P7), implicit-capture
 * weights and weight ledger (P8), XS lookup vs brute force (P9), energy balance
 * (P10), symmetry (P11), printed workload facts (P12); variants (R30-R32,
 * tests/test_oracle_variants.py): vacuum-escape closed form, escape/absorption/
 * roulette ledgers, the sampled-absorption branch law and counter budget,
 * roulette unbiasedness; census clock (tests/test_oracle_census.py): the flight-time
 * ledger tfl equals k*dt at the k-th census (R21's distance-timer conversion through a
 * collision), the first-flight law across a census (census n_mfp carry-over, R23), and
 * the invariance of a history under splitting its timestep at a census.
 * Parity unpinned: absolute per-cell tally values at paper scale (the paper's
 * Fig. 2 plots are absent) -- only P10-P12 constrain them.
 */
#ifndef NEUTRAL_ORACLE_H
#define NEUTRAL_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* Problem definition: structured 2D mesh of cell-centred mass densities
 * and two cross-section tables. */
typedef struct {
    int32_t nx, ny;
    double width, height;          /* m */
    const double *density;         /* [ny][nx] kg/m^3, row-major */
    const double *scatter_keys;    /* eV, strictly increasing */
    const double *scatter_vals;    /* barns */
    int64_t n_scatter;
    const double *capture_keys;
    const double *capture_vals;
    int64_t n_capture;
    double A;                      /* target mass / neutron mass */
    double molar_mass;             /* kg/mol */
    double e_min;                  /* eV, energy cutoff */
    double w_min;                  /* weight cutoff */
    int64_t max_events;            /* per history per step; guard */
    /* variants (readings R30-R32 in DESIGN.md §4) */
    int32_t boundary;              /* 0 reflective, 1 vacuum: escape     */
    int32_t analog;                /* 0 implicit capture (R8), 1 sampled absorption  */
    int32_t roulette;              /* 0 hard w_min kill (R7), 1 Russian roulette     */
    int32_t pad;
    double roulette_weight;        /* survivor weight of the roulette                */
} or_problem;

/* Particle store, structure of arrays, indexed by LOCAL index 0..n-1;
 * global id = first_id + local index.  All arrays caller-owned. */
typedef struct {
    double *x, *y, *ox, *oy, *e, *w, *mfp;
    int32_t *cx, *cy;
    uint32_t *ctr;
    uint8_t *status;               /* 1 = alive (at census), 0 = dead */
    uint32_t *nfac, *ncol, *ncen;  /* cumulative event counters */
    double *dep;                   /* cumulative energy this particle tallied */
    double *tfl;                   /* cumulative flight time (s): sum over segments of
                                    * length / speed -- an instrument of the oracle only
                                    * (pins the census clock); it
                                    * feeds back into nothing */
} or_particles;

/* Ledger of one step (sums over the particles stepped). */
typedef struct {
    uint64_t n_alive_start, n_facets, n_collisions, n_census, n_killed;
    double tally_total, census_energy, census_weight, killed_energy,
           killed_weight, absorbed_weight;
    uint64_t n_xs_range, n_nonfinite, n_event_cap;
    uint64_t n_escaped, n_absorbed;
    double escaped_energy, escaped_weight, absorbed_energy, roulette_gain;
} or_stats;

void     or_threefry2x64_20(uint64_t c0, uint64_t c1, uint64_t k0, uint64_t k1,
                            uint64_t out[2]);
double   or_u01(uint64_t x);
double   or_edge(int32_t i, double extent, int32_t n);
int32_t  or_cell_of(double q, double extent, int32_t n);
int64_t  or_xs_index(const double *keys, int64_t n, double e);
double   or_xs_lookup(const double *keys, const double *vals, int64_t n, double e);

void or_inject(const or_problem *pb, or_particles *pt, int64_t first_id,
               int64_t n_local, double src_x, double src_y, double src_w,
               double src_h, double initial_energy, uint64_t seed);

/* One timestep for local particles [0, n_local).  Deposits are summed into
 * tally[ny*nx] in (particle id, flush sequence) order; tally is NOT zeroed.
 * stats is zeroed and filled. */
void or_step(const or_problem *pb, or_particles *pt, int64_t first_id,
             int64_t n_local, uint64_t seed, double dt, double *tally,
             or_stats *stats);

#ifdef __cplusplus
}
#endif
#endif
