// nt_mesh.cu -- mesh preparation on the device: density validation and the lossless
// density encoding (u8 / u16 material codes + number-density table) used by the tracker.
#include <cub/device/device_radix_sort.cuh>
#include <cub/device/device_select.cuh>

#include "nt_internal.h"

namespace nt {

// Count cells whose density is not finite or < 0 (nt_init_mesh validation).
__global__ void density_check_kernel(const double* __restrict__ rho, int64_t n,
                                     unsigned long long* bad) {
  unsigned long long local = 0;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x) {
    const double v = rho[i];
    if (!(v >= 0.0) || !isfinite(v)) ++local;
  }
  for (int o = 16; o > 0; o >>= 1) local += __shfl_xor_sync(kFull, local, o);
  if ((threadIdx.x & 31) == 0 && local) atomicAdd(bad, local);
}

__global__ void bits_kernel(const double* __restrict__ rho, int64_t n,
                            unsigned long long* __restrict__ out) {
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x)
    out[i] = (unsigned long long)__double_as_longlong(rho[i]);
}

// code[cell_index(cx, cy)] = index of rho[cy][cx]'s bit pattern among the sorted distinct
// patterns uniq[0..nu)  (rho row-major as given; codes in the storage layout)
template <class T>
__global__ void encode_kernel(const double* __restrict__ rho, int64_t n, Mesh M,
                              const unsigned long long* __restrict__ uniq, int nu,
                              T* __restrict__ code) {
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x) {
    const unsigned long long b = (unsigned long long)__double_as_longlong(rho[i]);
    int lo = 0, hi = nu;                         // uniq[lo] <= b < uniq[hi]
    while (hi - lo > 1) {
      const int mid = (lo + hi) >> 1;
      if (uniq[mid] <= b) lo = mid; else hi = mid;
    }
    const int32_t cy = (int32_t)(i / M.nx), cx = (int32_t)(i - (int64_t)cy * M.nx);
    code[cell_index(M, cx, cy)] = (T)lo;
  }
}

// Row-major [ny][nx] <-> storage layout (to_storage: gather from rm into st; else back).
__global__ void relayout_kernel(const double* __restrict__ src, double* __restrict__ dst,
                                int64_t n, Mesh M, int to_storage) {
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int32_t cy = (int32_t)(i / M.nx), cx = (int32_t)(i - (int64_t)cy * M.nx);
    const int64_t s = cell_index(M, cx, cy);
    if (to_storage) dst[s] = src[i]; else dst[i] = src[s];
  }
}

// One thread per block: the block's code if all its cells (inside the mesh) share it.
__global__ void block_map_kernel(const uint8_t* __restrict__ code, Mesh M,
                                 uint8_t* __restrict__ blk) {
  const int32_t b = blockIdx.x * blockDim.x + threadIdx.x;
  if (b >= M.nblk) return;
  const int32_t by = b / M.nbx, bx = b - by * M.nbx;
  const int32_t x0 = bx << M.bshift, y0 = by << M.bshift, side = 1 << M.bshift;
  const int32_t x1 = min(x0 + side, M.nx), y1 = min(y0 + side, M.ny);
  const uint32_t c0 = code[cell_index(M, x0, y0)];
  uint32_t out = c0;
  for (int32_t cy = y0; cy < y1 && out != kBlkMixed; ++cy)
    for (int32_t cx = x0; cx < x1; ++cx)
      if (code[cell_index(M, cx, cy)] != c0) { out = kBlkMixed; break; }
  blk[b] = (uint8_t)out;
}

cudaError_t launch_block_map(const uint8_t* code, const Mesh& M, uint8_t* blk, cudaStream_t s) {
  block_map_kernel<<<(M.nblk + 127) / 128, 128, 0, s>>>(code, M, blk);
  return cudaGetLastError();
}

// nd_tab[k] = rho_k * cn: the first product of DESIGN.md §3 MAT, rounded once, as in place.
__global__ void nd_table_kernel(const unsigned long long* __restrict__ uniq, int nu, double cn,
                                double* __restrict__ tab) {
  const int k = blockIdx.x * blockDim.x + threadIdx.x;
  if (k < nu) tab[k] = __longlong_as_double((long long)uniq[k]) * cn;
}

// Validation + distinct density values in one pass over a chunk (nt_init_mesh, while the
// next chunk is still being copied): bad[0] counts values not finite and >= 0; every valid
// value's bit pattern is inserted into an open-addressing set (kDistinctSlots slots, empty =
// all ones, which no valid density has); bad[1] counts the distinct patterns inserted and
// bad[2] != 0 once the set is half full (the caller then falls back to the sorting path).
__global__ void check_distinct_kernel(const double* __restrict__ rho, int64_t n,
                                      unsigned long long* bad, unsigned long long* set) {
  unsigned long long nbad = 0;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
       i += (int64_t)gridDim.x * blockDim.x) {
    const double v = rho[i];
    if (!(v >= 0.0) || !isfinite(v)) { ++nbad; continue; }
    const unsigned long long b = (unsigned long long)__double_as_longlong(v);
    unsigned h = (unsigned)((b * 0x9E3779B97F4A7C15ull) >> 52) & (kDistinctSlots - 1);
    for (int probe = 0; probe < kDistinctSlots; ++probe) {
      const unsigned long long cur = ld_volatile(set + h);
      if (cur == b) break;
      if (cur == ~0ull) {
        if (ld_volatile(bad + 2)) break;            // overflowed: the sort path takes over
        const unsigned long long old = atomicCAS(set + h, ~0ull, b);
        if (old == ~0ull) {
          if (atomicAdd(bad + 1, 1ull) + 1 >= (unsigned long long)(kDistinctSlots / 2)) atomicExch(bad + 2, 1ull);
          break;
        }
        if (old == b) break;
      }
      h = (h + 1) & (kDistinctSlots - 1);
    }
  }
  for (int o = 16; o > 0; o >>= 1) nbad += __shfl_xor_sync(kFull, nbad, o);
  if ((threadIdx.x & 31) == 0 && nbad) atomicAdd(bad, nbad);
}

// The set's patterns in increasing order: uniq[rank] (one block; <= kDistinctSlots / 2 keys).
__global__ void distinct_sort_kernel(const unsigned long long* __restrict__ set,
                                     unsigned long long* __restrict__ uniq) {
  __shared__ unsigned long long s[kDistinctSlots];
  for (int k = threadIdx.x; k < kDistinctSlots; k += blockDim.x) s[k] = set[k];
  __syncthreads();
  for (int k = threadIdx.x; k < kDistinctSlots; k += blockDim.x) {
    const unsigned long long b = s[k];
    if (b == ~0ull) continue;
    int rank = 0;
    for (int j = 0; j < kDistinctSlots; ++j) rank += (s[j] != ~0ull && s[j] < b) ? 1 : 0;
    uniq[rank] = b;
  }
}

static unsigned grid_for(int64_t n) {
  const int64_t b = (n + 255) / 256;
  return (unsigned)(b > 148 * 32 ? 148 * 32 : (b < 1 ? 1 : b));
}

cudaError_t launch_density_check(const double* rho, int64_t n, unsigned long long* bad,
                                 cudaStream_t s) {
  density_check_kernel<<<grid_for(n), 256, 0, s>>>(rho, n, bad);
  return cudaGetLastError();
}

cudaError_t launch_check_distinct(const double* rho, int64_t n, unsigned long long* bad,
                                  unsigned long long* set, cudaStream_t s) {
  if (n > 0) check_distinct_kernel<<<grid_for(n), 256, 0, s>>>(rho, n, bad, set);
  return cudaGetLastError();
}

cudaError_t launch_distinct_sort(const unsigned long long* set, unsigned long long* uniq,
                                 cudaStream_t s) {
  distinct_sort_kernel<<<1, 1024, 0, s>>>(set, uniq);
  return cudaGetLastError();
}

cudaError_t density_distinct(const double* rho, int64_t n, unsigned long long* k0,
                             unsigned long long* k1, void* temp, size_t& temp_bytes,
                             int* d_count, cudaStream_t s) {
  if (temp == nullptr) {
    size_t a = 0, b = 0;
    cudaError_t e = cub::DeviceRadixSort::SortKeys(nullptr, a, k0, k1, n, 0, 64, s);
    if (e != cudaSuccess) return e;
    e = cub::DeviceSelect::Unique(nullptr, b, k1, k0, d_count, n, s);
    temp_bytes = a > b ? a : b;
    return e;
  }
  bits_kernel<<<grid_for(n), 256, 0, s>>>(rho, n, k0);
  cudaError_t e = cub::DeviceRadixSort::SortKeys(temp, temp_bytes, k0, k1, n, 0, 64, s);
  if (e != cudaSuccess) return e;
  return cub::DeviceSelect::Unique(temp, temp_bytes, k1, k0, d_count, n, s);
}

cudaError_t launch_encode(const double* rho, int64_t n, const Mesh& M,
                          const unsigned long long* uniq, int nu, double cn, int fmt, void* code,
                          double* nd_tab, cudaStream_t s) {
  if (fmt == kDensU8)
    encode_kernel<uint8_t><<<grid_for(n), 256, 0, s>>>(rho, n, M, uniq, nu, (uint8_t*)code);
  else
    encode_kernel<uint16_t><<<grid_for(n), 256, 0, s>>>(rho, n, M, uniq, nu, (uint16_t*)code);
  nd_table_kernel<<<(nu + 255) / 256, 256, 0, s>>>(uniq, nu, cn, nd_tab);
  return cudaGetLastError();
}

cudaError_t launch_relayout(const double* src, double* dst, int64_t n, const Mesh& M,
                            bool to_storage, cudaStream_t s) {
  relayout_kernel<<<grid_for(n), 256, 0, s>>>(src, dst, n, M, to_storage ? 1 : 0);
  return cudaGetLastError();
}

}  // namespace nt
