// Microbenchmark for the Parboil-shaped fp32 SpMV (BJ.cfg[2]):
// is the sell-sorted kernel's bound -- one L1->L2 request per random x gather
// (ncu: l1tex__m_l1tex2xbar_req_cycles_active 84.7 % of peak, 14.9 M sectors
// for 11.5 M nonzeros) -- avoidable by a 2-D tiling?
//
// Tile (row block of RB rows, column part q of 2^colbits columns): its
// nonzeros sorted by column, so the 32 gathers of one warp instruction fall in
// a few x sectors (RB*11/n nonzeros per column); y of the row block lives in
// shared memory (fp32 red.shared.add); each tile writes its RB partials to
// part[q][row], and a combine pass sums the CQ parts per row.
// mode 0: column-sorted tiles; mode 1: the same tiles with the nonzero order
// shuffled (uncoalesced gathers: isolates the coalescing effect).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o pbtile pbtile.cu
#include <algorithm>
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <numeric>
#include <random>
#include <vector>

#define CK(x)                                                                   \
  do {                                                                          \
    cudaError_t e_ = (x);                                                       \
    if (e_ != cudaSuccess) {                                                    \
      printf("CUDA %s at %d: %s\n", #x, __LINE__, cudaGetErrorString(e_));      \
      exit(1);                                                                  \
    }                                                                           \
  } while (0)

__device__ __forceinline__ float ldf(const float* p) {
  float r;
  asm volatile("ld.global.nc.L1::no_allocate.f32 %0, [%1];" : "=f"(r) : "l"(p));
  return r;
}
__device__ __forceinline__ unsigned ldu(const unsigned* p) {
  unsigned r;
  asm volatile("ld.global.nc.L1::no_allocate.u32 %0, [%1];" : "=r"(r) : "l"(p));
  return r;
}

template <int U>
__global__ void __launch_bounds__(1024) k_tile(const float* __restrict__ vals, const unsigned* __restrict__ idx,
                                               const long long* __restrict__ toff, const float* __restrict__ x,
                                               float* __restrict__ part, int RB, int colbits, int CQ, int m) {
  extern __shared__ float ys[];
  const int t = blockIdx.x, rb = t / CQ, q = t % CQ;
  for (int i = threadIdx.x; i < RB; i += blockDim.x) ys[i] = 0.f;
  __syncthreads();
  const float* xb = x + (size_t(q) << colbits);
  const unsigned cmask = (1u << colbits) - 1;
  const long long k0 = toff[t], k1 = toff[t + 1];
  const int nt = blockDim.x;
  for (long long kb = k0 + threadIdx.x; kb < k1; kb += (long long)nt * U) {
    float v[U];
    unsigned p[U];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const long long k = kb + (long long)u * nt;
      v[u] = k < k1 ? ldf(vals + k) : 0.f;
      p[u] = k < k1 ? ldu(idx + k) : 0u;
    }
    float xv[U];
#pragma unroll
    for (int u = 0; u < U; ++u) xv[u] = __ldg(xb + (p[u] & cmask));
#pragma unroll
    for (int u = 0; u < U; ++u)
      if (kb + (long long)u * nt < k1) atomicAdd(&ys[p[u] >> colbits], v[u] * xv[u]);
  }
  __syncthreads();
  const int r0 = rb * RB;
  for (int i = threadIdx.x; i < RB && r0 + i < m; i += blockDim.x) part[size_t(q) * m + r0 + i] = ys[i];
}

__global__ void k_combine(const float* __restrict__ part, float* __restrict__ y, int m, int CQ) {
  for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < m; i += gridDim.x * blockDim.x) {
    float s = 0.f;
    for (int q = 0; q < CQ; ++q) s += part[size_t(q) * m + i];
    y[i] = s;
  }
}

int main() {
  const int m = 1 << 20, n = 1 << 20;
  std::mt19937_64 rng(20180324);
  std::vector<int> len(m), perm(m);
  std::iota(perm.begin(), perm.end(), 0);
  std::shuffle(perm.begin(), perm.end(), rng);
  long long nnz = 0;
  for (int r = 0; r < m; ++r) {
    const int L = std::max(1, (int)std::floor(10000.0 * std::pow(double(r + 1), -0.545)));
    len[perm[r]] = L;
    nnz += L;
  }
  std::vector<int> rowptr(m + 1, 0), col(nnz);
  std::vector<float> val(nnz);
  for (int i = 0; i < m; ++i) rowptr[i + 1] = rowptr[i] + len[i];
  std::uniform_int_distribution<int> cd(0, n - 1);
  std::uniform_real_distribution<float> vd(-1.f, 1.f);
  for (long long k = 0; k < nnz; ++k) {
    col[k] = cd(rng);
    val[k] = vd(rng);
  }
  std::vector<float> xh(n);
  for (auto& v : xh) v = vd(rng);
  // reference y (double)
  std::vector<double> yref(m, 0.0);
  for (int i = 0; i < m; ++i)
    for (int k = rowptr[i]; k < rowptr[i + 1]; ++k) yref[i] += double(val[k]) * double(xh[col[k]]);
  printf("m %d nnz %lld\n", m, nnz);

  float *dx, *dy, *dpart;
  CK(cudaMalloc(&dx, 4 * n));
  CK(cudaMalloc(&dy, 4 * m));
  CK(cudaMalloc(&dpart, size_t(4) * m * 64));
  CK(cudaMemcpy(dx, xh.data(), 4 * n, cudaMemcpyHostToDevice));
  CK(cudaFuncSetAttribute(k_tile<4>, cudaFuncAttributeMaxDynamicSharedMemorySize, 220 * 1024));
  CK(cudaFuncSetAttribute(k_tile<8>, cudaFuncAttributeMaxDynamicSharedMemorySize, 220 * 1024));

  struct Cfg { int rowbits, RB, mode, threads, U; };
  const Cfg cfgs[] = {{14, 16384, 0, 1024, 4}, {15, 32768, 0, 1024, 4}, {16, 49152, 0, 1024, 4},
                      {16, 32768, 0, 1024, 4}, {15, 32768, 1, 1024, 4}, {15, 32768, 0, 512, 4},
                      {15, 32768, 0, 1024, 8}, {14, 16384, 0, 512, 8}};
  for (const Cfg& c : cfgs) {
    const int colbits = 32 - c.rowbits;
    const int CQ = std::max(1, n >> colbits);
    const int nrb = (m + c.RB - 1) / c.RB;
    const int ntiles = nrb * CQ;
    std::vector<std::vector<std::pair<unsigned, float>>> tiles(ntiles);
    for (int i = 0; i < m; ++i) {
      const int rb = i / c.RB, rl = i % c.RB;
      for (int k = rowptr[i]; k < rowptr[i + 1]; ++k) {
        const int q = col[k] >> colbits, cl = col[k] & ((1 << colbits) - 1);
        tiles[size_t(rb) * CQ + q].push_back({(unsigned(rl) << colbits) | unsigned(cl), val[k]});
      }
    }
    std::vector<long long> toff(ntiles + 1, 0);
    std::vector<unsigned> idx;
    std::vector<float> vv;
    idx.reserve(nnz);
    vv.reserve(nnz);
    const unsigned cmask = (1u << colbits) - 1;
    for (int t = 0; t < ntiles; ++t) {
      auto& T = tiles[t];
      std::sort(T.begin(), T.end(), [&](const std::pair<unsigned, float>& a, const std::pair<unsigned, float>& b) {
        return (a.first & cmask) != (b.first & cmask) ? (a.first & cmask) < (b.first & cmask) : a.first < b.first;
      });
      if (c.mode == 1) std::shuffle(T.begin(), T.end(), rng);
      for (auto& e : T) {
        idx.push_back(e.first);
        vv.push_back(e.second);
      }
      toff[t + 1] = (long long)idx.size();
    }
    unsigned* didx;
    float* dv;
    long long* dtoff;
    CK(cudaMalloc(&didx, 4 * nnz));
    CK(cudaMalloc(&dv, 4 * nnz));
    CK(cudaMalloc(&dtoff, 8 * (ntiles + 1)));
    CK(cudaMemcpy(didx, idx.data(), 4 * nnz, cudaMemcpyHostToDevice));
    CK(cudaMemcpy(dv, vv.data(), 4 * nnz, cudaMemcpyHostToDevice));
    CK(cudaMemcpy(dtoff, toff.data(), 8 * (ntiles + 1), cudaMemcpyHostToDevice));
    const size_t smem = size_t(4) * c.RB;
    auto run = [&]() {
      if (c.U == 4)
        k_tile<4><<<ntiles, c.threads, smem>>>(dv, didx, dtoff, dx, dpart, c.RB, colbits, CQ, m);
      else
        k_tile<8><<<ntiles, c.threads, smem>>>(dv, didx, dtoff, dx, dpart, c.RB, colbits, CQ, m);
    };
    auto comb = [&]() { k_combine<<<148 * 8, 256>>>(dpart, dy, m, CQ); };
    for (int w = 0; w < 3; ++w) {
      run();
      comb();
    }
    CK(cudaDeviceSynchronize());
    std::vector<float> yh(m);
    CK(cudaMemcpy(yh.data(), dy, 4 * m, cudaMemcpyDeviceToHost));
    double maxrel = 0;
    for (int i = 0; i < m; ++i) {
      double b = 0;
      for (int k = rowptr[i]; k < rowptr[i + 1]; ++k) b += std::fabs(double(val[k]) * double(xh[col[k]]));
      if (b > 0) maxrel = std::max(maxrel, std::fabs(double(yh[i]) - yref[i]) / b);
    }
    cudaEvent_t a, b, e2;
    CK(cudaEventCreate(&a));
    CK(cudaEventCreate(&b));
    CK(cudaEventCreate(&e2));
    const int reps = 20;
    float best_t = 1e9, best_all = 1e9;
    for (int r = 0; r < reps; ++r) {
      CK(cudaEventRecord(a));
      run();
      CK(cudaEventRecord(b));
      comb();
      CK(cudaEventRecord(e2));
      CK(cudaEventSynchronize(e2));
      float t1, t2;
      CK(cudaEventElapsedTime(&t1, a, b));
      CK(cudaEventElapsedTime(&t2, a, e2));
      best_t = std::min(best_t, t1);
      best_all = std::min(best_all, t2);
    }
    long long tmax = 0;
    for (int t = 0; t < ntiles; ++t) tmax = std::max(tmax, toff[t + 1] - toff[t]);
    printf("RB %5d colbits %d CQ %2d tiles %4d (max %lld nnz, mean %lld) mode %d thr %4d U %d: tile %6.1f us, +combine %6.1f us, maxrel %.2e %s\n",
           c.RB, colbits, CQ, ntiles, tmax, nnz / ntiles, c.mode, c.threads, c.U, best_t * 1e3, best_all * 1e3, maxrel,
           cudaGetErrorString(cudaGetLastError()));
    fflush(stdout);
    cudaFree(didx);
    cudaFree(dv);
    cudaFree(dtoff);
  }
  return 0;
}
