/*
 * neutral_oracle.c -- the CPU oracle (TEST INFRASTRUCTURE ONLY; see header).
 *
 * A plain transcription of the algorithm in DESIGN.md §3, which is the
 * paper's method (§IV-A..F, §V-A Listing 1, §V-C) with the readings
 * listed in DESIGN.md §4 where the paper is silent.  Single-threaded; particles
 * are tracked in id order, so deposits reach the tally in (particle id, flush
 * sequence) order.  Build: gcc -O2 -ffp-contract=off -fno-fast-math (no FMA
 * contraction, so every expression below rounds exactly as written).
 *
 * Library primitives used as steps: libm log, cos, sin, sqrt.
 */
#include "neutral_oracle.h"
#include <math.h>
#include <string.h>

/* ---- constants (DESIGN.md §4 readings R-const) ------------------------------ */
static const double OR_AVOGADRO = 6.02214076e23;     /* mol^-1, SI exact      */
static const double OR_EV       = 1.602176634e-19;   /* J, SI exact           */
static const double OR_MN       = 1.67492749804e-27; /* kg, CODATA 2018       */
static const double OR_BARN     = 1.0e-28;           /* m^2                   */
static const double OR_TWO_PI   = 6.283185307179586;

/* ---- Threefry-2x64-20 (Random123 Threefry, §IV-F) ----------------- *
 * Salmon et al., "Parallel random numbers: as easy as 1, 2, 3" (SC'11):
 * key schedule ks2 = C240 ^ k0 ^ k1; 20 rounds of (add, rotate, xor) with the
 * 2x64 rotation constants; key injection after every 4 rounds. */
static uint64_t or_rotl64(uint64_t x, unsigned r)
{
    return (x << r) | (x >> (64u - r));
}

void or_threefry2x64_20(uint64_t c0, uint64_t c1, uint64_t k0, uint64_t k1,
                        uint64_t out[2])
{
    static const unsigned R[8] = {16, 42, 12, 31, 16, 32, 24, 21};
    uint64_t ks[3];
    ks[0] = k0;
    ks[1] = k1;
    ks[2] = 0x1BD11BDAA9FC1A22ULL ^ k0 ^ k1;
    uint64_t x0 = c0 + ks[0];
    uint64_t x1 = c1 + ks[1];
    for (int r = 0; r < 20; ++r) {
        x0 += x1;
        x1 = or_rotl64(x1, R[r % 8]);
        x1 ^= x0;
        if (r % 4 == 3) {
            uint64_t s = (uint64_t)(r + 1) / 4;
            x0 += ks[s % 3];
            x1 += ks[(s + 1) % 3] + s;
        }
    }
    out[0] = x0;
    out[1] = x1;
}

/* u(x) = ((x >> 11) | 1) * 2^-53: an odd multiple of 2^-53 in (0, 1), exact. */
double or_u01(uint64_t x)
{
    return (double)((x >> 11) | 1ULL) * 0x1.0p-53;
}

/* ---- mesh (§IV-C) -------------------------------------------------- */
double or_edge(int32_t i, double extent, int32_t n)
{
    return ((double)i * extent) / (double)n;
}

/* The unique i in [0, n-1] with edge(i) <= q < edge(i+1); q >= edge(n) -> n-1. */
int32_t or_cell_of(double q, double extent, int32_t n)
{
    if (!(q >= 0.0)) return 0;
    if (q >= or_edge(n, extent, n)) return n - 1;
    int32_t lo = 0, hi = n;            /* edge(lo) <= q < edge(hi) */
    while (hi - lo > 1) {
        int32_t mid = lo + (hi - lo) / 2;
        if (or_edge(mid, extent, n) <= q) lo = mid; else hi = mid;
    }
    return lo;
}

/* ---- microscopic cross sections (§IV-D) ---------------------------- *
 * Energy-bin search then linear interpolation.  i = max{i in [0,N-2]: k[i] <= e}
 * for e already clamped into [k[0], k[N-1]]. */
int64_t or_xs_index(const double *keys, int64_t n, double e)
{
    if (e >= keys[n - 1]) return n - 2;
    if (e <= keys[0]) return 0;
    int64_t lo = 0, hi = n - 1;        /* keys[lo] <= e < keys[hi] */
    while (hi - lo > 1) {
        int64_t mid = lo + (hi - lo) / 2;
        if (keys[mid] <= e) lo = mid; else hi = mid;
    }
    return lo;
}

double or_xs_lookup(const double *keys, const double *vals, int64_t n, double e)
{
    int64_t i = or_xs_index(keys, n, e);
    double t = (e - keys[i]) / (keys[i + 1] - keys[i]);
    return vals[i] + t * (vals[i + 1] - vals[i]);
}

/* ---- per-history material state ------------------------- */
typedef struct {
    double st;   /* total microscopic XS in m^2: (sigma_s + sigma_a) * barn */
    double pa;   /* absorption probability sigma_a / sigma_t                 */
    double H;    /* expected heating response per collision, eV */
} or_mat;

static double or_clamp_count(const double *keys, int64_t n, double e,
                             uint64_t *n_range)
{
    if (e < keys[0]) { ++*n_range; return keys[0]; }
    if (e > keys[n - 1]) { ++*n_range; return keys[n - 1]; }
    return e;
}

static or_mat or_refresh_xs(const or_problem *pb, double e, uint64_t *n_range)
{
    double es = or_clamp_count(pb->scatter_keys, pb->n_scatter, e, n_range);
    double ea = or_clamp_count(pb->capture_keys, pb->n_capture, e, n_range);
    double ss = or_xs_lookup(pb->scatter_keys, pb->scatter_vals, pb->n_scatter, es);
    double sa = or_xs_lookup(pb->capture_keys, pb->capture_vals, pb->n_capture, ea);
    double t = ss + sa;
    double A = pb->A;
    double f = (A * A + 1.0) / ((A + 1.0) * (A + 1.0)); /* mean E'/E, elastic */
    or_mat m;
    m.st = t * OR_BARN;
    m.pa = t > 0.0 ? sa / t : 0.0;
    double rs = t > 0.0 ? ss / t : 0.0;
    m.H = e - rs * (e * f);
    return m;
}

static double or_speed(double e)   /* m/s of a neutron with kinetic energy e eV */
{
    double kv = (2.0 * OR_EV) / OR_MN;
    return sqrt(e * kv);
}

/* ---- source injection (§IV-F) -------------------------------------- */
void or_inject(const or_problem *pb, or_particles *pt, int64_t first_id,
               int64_t n_local, double src_x, double src_y, double src_w,
               double src_h, double initial_energy, uint64_t seed)
{
    for (int64_t i = 0; i < n_local; ++i) {
        uint64_t p = (uint64_t)(first_id + i);
        uint64_t r[2];
        or_threefry2x64_20(0, 0, p, seed, r);
        double x = src_x + or_u01(r[0]) * src_w;
        double y = src_y + or_u01(r[1]) * src_h;
        or_threefry2x64_20(1, 0, p, seed, r);
        double theta = OR_TWO_PI * or_u01(r[0]);
        pt->x[i] = x;
        pt->y[i] = y;
        pt->cx[i] = or_cell_of(x, pb->width, pb->nx);
        pt->cy[i] = or_cell_of(y, pb->height, pb->ny);
        pt->ox[i] = cos(theta);
        pt->oy[i] = sin(theta);
        pt->mfp[i] = -log(or_u01(r[1]));
        pt->e[i] = initial_energy;
        pt->w[i] = 1.0;
        pt->ctr[i] = 2;
        pt->status[i] = 1;
        pt->nfac[i] = 0;
        pt->ncol[i] = 0;
        pt->ncen[i] = 0;
        pt->dep[i] = 0.0;
        pt->tfl[i] = 0.0;
    }
}

/* ---- one history for one timestep (Listing 1, §V-A) ---------------- */
static void or_flush(double *tally, int32_t nx, int32_t cx, int32_t cy,
                     double *acc, double *dep, or_stats *st)
{
    /* P:397-401 (§V-C): deposit leaves the register at a facet,
     * at census and (reading S15) at a kill. */
    tally[(int64_t)cy * nx + cx] += *acc;
    *dep += *acc;
    st->tally_total += *acc;
    *acc = 0.0;
}

static void or_history(const or_problem *pb, or_particles *pt, int64_t i,
                       uint64_t pid, uint64_t seed, double dt, double cn,
                       double *tally, or_stats *st)
{
    const int32_t nx = pb->nx, ny = pb->ny;
    const double W = pb->width, Hh = pb->height, A = pb->A;
    double x = pt->x[i], y = pt->y[i], ox = pt->ox[i], oy = pt->oy[i];
    double e = pt->e[i], w = pt->w[i], mfp = pt->mfp[i];
    int32_t cx = pt->cx[i], cy = pt->cy[i];
    uint32_t c = pt->ctr[i];
    double dep = pt->dep[i];
    double tfl = pt->tfl[i];           /* flight-time ledger: += segment / speed */
    double acc = 0.0;

    or_mat m = or_refresh_xs(pb, e, &st->n_xs_range);
    double nd = pb->density[(int64_t)cy * nx + cx] * cn;  /* number density */
    double sig = nd * m.st;                                /* Sigma_t, 1/m    */
    double v = or_speed(e);
    double dcen = v * dt;              /* census timer, as a distance */
    double iox = 1.0 / ox, ioy = 1.0 / oy;
    int64_t nev = 0;

    for (;;) {
        if (nev >= pb->max_events) {   /* guard: count, flush, stop the history */
            st->n_event_cap++;
            or_flush(tally, nx, cx, cy, &acc, &dep, st);
            pt->status[i] = 0;
            st->n_killed++;
            st->killed_energy += w * e;
            st->killed_weight += w;
            break;
        }
        ++nev;
        /* calculate_time_to_events(): facet, collision, census */
        double tx = ox > 0.0 ? (or_edge(cx + 1, W, nx) - x) * iox
                  : ox < 0.0 ? (or_edge(cx, W, nx) - x) * iox : INFINITY;
        if (tx < 0.0) tx = 0.0;
        double ty = oy > 0.0 ? (or_edge(cy + 1, Hh, ny) - y) * ioy
                  : oy < 0.0 ? (or_edge(cy, Hh, ny) - y) * ioy : INFINITY;
        if (ty < 0.0) ty = 0.0;
        int axis_x = tx < ty;
        double df = axis_x ? tx : ty;
        double dc = sig > 0.0 ? mfp / sig : INFINITY;
        double ds = dcen;

        if (dc < df && dc < ds) {
            /* ---- collision ---- */
            acc += ((w * dc) * sig) * m.H;
            tfl += dc / v;
            x = x + dc * ox;
            y = y + dc * oy;
            dcen = dcen - dc;
            uint64_t r[2];
            or_threefry2x64_20(c, 0, pid, seed, r);
            c += 1;
            pt->ncol[i]++;
            st->n_collisions++;
            double mfp_u = or_u01(r[1]);           /* the draw for the new n_mfp  */
            if (!pb->analog) {
                double w_old = w;                  /* implicit capture */
                w = w * (1.0 - m.pa);
                st->absorbed_weight += w_old - w;
            } else {
                /* reading R31 (S8 reading A): absorb with probability p_a ("two main
                 * branches"); the scatter branch draws its n_mfp from the next
                 * counter because word b decided the branch. */
                if (or_u01(r[1]) < m.pa) {
                    or_flush(tally, nx, cx, cy, &acc, &dep, st);
                    st->n_absorbed++;
                    st->absorbed_weight += w;
                    st->absorbed_energy += w * e;
                    pt->status[i] = 0;
                    break;
                }
                uint64_t r2[2];
                or_threefry2x64_20(c, 0, pid, seed, r2);
                c += 1;
                mfp_u = or_u01(r2[0]);
            }
            double mu = 1.0 - 2.0 * or_u01(r[0]);  /* CM cosine, isotropic        */
            double e2 = e * (((A * A + (2.0 * A) * mu) + 1.0) / ((A + 1.0) * (A + 1.0)));
            double ct = 0.5 * ((A + 1.0) * sqrt(e2 / e) - (A - 1.0) * sqrt(e / e2));
            double sgn = (r[0] & 1ULL) ? -1.0 : 1.0;
            double q = 1.0 - ct * ct;
            double stt = sgn * sqrt(q > 0.0 ? q : 0.0);
            double nox = ox * ct - oy * stt;
            double noy = ox * stt + oy * ct;
            ox = nox;
            oy = noy;
            double tcen = dcen / v;
            e = e2;
            int kill = e < pb->e_min || w < pb->w_min;   /* termination    */
            if (kill && pb->roulette && !(e < pb->e_min)) {
                /* reading R32: Russian roulette instead of the hard weight cut: survive
                 * with probability w / w_s at weight w_s (one counter) */
                uint64_t r3[2];
                or_threefry2x64_20(c, 0, pid, seed, r3);
                c += 1;
                if (or_u01(r3[0]) < w / pb->roulette_weight) {
                    st->roulette_gain += pb->roulette_weight - w;
                    w = pb->roulette_weight;
                    kill = 0;
                }
            }
            if (kill) {
                or_flush(tally, nx, cx, cy, &acc, &dep, st);
                st->killed_energy += w * e;
                st->killed_weight += w;
                st->n_killed++;
                pt->status[i] = 0;
                break;
            }
            v = or_speed(e);
            dcen = tcen * v;
            m = or_refresh_xs(pb, e, &st->n_xs_range);
            sig = nd * m.st;
            iox = 1.0 / ox;
            ioy = 1.0 / oy;
            mfp = -log(mfp_u);
        } else if (df < ds) {
            /* ---- facet ---------------------------- */
            int escaped = 0;
            acc += ((w * df) * sig) * m.H;
            tfl += df / v;
            double nm = mfp - df * sig;
            mfp = nm > 0.0 ? nm : 0.0;
            dcen = dcen - df;
            if (axis_x) {
                y = y + df * oy;
                x = ox > 0.0 ? or_edge(cx + 1, W, nx) : or_edge(cx, W, nx);
                or_flush(tally, nx, cx, cy, &acc, &dep, st);
                int at_boundary = ox > 0.0 ? cx == nx - 1 : cx == 0;
                if (at_boundary && pb->boundary) { escaped = 1; }
                else if (ox > 0.0) {
                    if (cx == nx - 1) { ox = -ox; iox = -iox; } else { cx += 1; }
                } else {
                    if (cx == 0) { ox = -ox; iox = -iox; } else { cx -= 1; }
                }
            } else {
                x = x + df * ox;
                y = oy > 0.0 ? or_edge(cy + 1, Hh, ny) : or_edge(cy, Hh, ny);
                or_flush(tally, nx, cx, cy, &acc, &dep, st);
                int at_boundary = oy > 0.0 ? cy == ny - 1 : cy == 0;
                if (at_boundary && pb->boundary) { escaped = 1; }
                else if (oy > 0.0) {
                    if (cy == ny - 1) { oy = -oy; ioy = -ioy; } else { cy += 1; }
                } else {
                    if (cy == 0) { oy = -oy; ioy = -ioy; } else { cy -= 1; }
                }
            }
            pt->nfac[i]++;
            st->n_facets++;
            if (escaped) {                 /* reading R30: vacuum boundary, escape */
                st->n_escaped++;
                st->escaped_energy += w * e;
                st->escaped_weight += w;
                pt->status[i] = 0;
                break;
            }
            nd = pb->density[(int64_t)cy * nx + cx] * cn;   /* load new density */
            sig = nd * m.st;
        } else {
            /* ---- census ------------------------------------ */
            acc += ((w * ds) * sig) * m.H;
            tfl += ds / v;
            x = x + ds * ox;
            y = y + ds * oy;
            double nm = mfp - ds * sig;
            mfp = nm > 0.0 ? nm : 0.0;
            or_flush(tally, nx, cx, cy, &acc, &dep, st);
            pt->ncen[i]++;
            st->n_census++;
            st->census_energy += w * e;
            st->census_weight += w;
            break;
        }
    }
    if (!(isfinite(x) && isfinite(y) && isfinite(e) && isfinite(w))) st->n_nonfinite++;
    pt->x[i] = x; pt->y[i] = y; pt->ox[i] = ox; pt->oy[i] = oy;
    pt->e[i] = e; pt->w[i] = w; pt->mfp[i] = mfp;
    pt->cx[i] = cx; pt->cy[i] = cy; pt->ctr[i] = c; pt->dep[i] = dep;
    pt->tfl[i] = tfl;
}

void or_step(const or_problem *pb, or_particles *pt, int64_t first_id,
             int64_t n_local, uint64_t seed, double dt, double *tally,
             or_stats *stats)
{
    memset(stats, 0, sizeof(*stats));
    double cn = OR_AVOGADRO / pb->molar_mass;   /* atoms per kg */
    for (int64_t i = 0; i < n_local; ++i) {
        if (pt->status[i] != 1) continue;
        stats->n_alive_start++;
        or_history(pb, pt, i, (uint64_t)(first_id + i), seed, dt, cn, tally, stats);
    }
}
