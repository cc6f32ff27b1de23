// error.cu -- device reduction of the error metric (Table 1).
//   MRE = mean over {i : e_i != 0} of |e_i - a_i| / |e_i|
//   ME  = sum |e - a| / sum |e|      (Sobel's "mean error")
//   MAE = mean |e - a|
// Per-element terms in fp32 (e - a is exact when e and a are within 2x), sums
// in fp64.  Deterministic: a fixed grid of kErrBlocks blocks, each thread
// walks a fixed index sequence, fixed-order tree reductions, then one block
// reduces the per-block partials in index order.
#include <cuda_runtime.h>

#include <cstdint>

namespace kp {

constexpr int kErrBlocks = 148 * 4;
constexpr int kErrThreads = 256;

__device__ __forceinline__ float to_f(float v) { return v; }
__device__ __forceinline__ float to_f(uint8_t v) { return (float)v; }

template <typename T>
__device__ __forceinline__ void err_term(int metric, T ev, T av, double& s, double& t, long long& c) {
  const float e = to_f(ev), a = to_f(av);
  const float d = fabsf(e - a);
  if (metric == 0) {
    if (e != 0.f) { s += (double)__fdiv_rn(d, fabsf(e)); c += 1; }
  } else {
    s += (double)d;
    t += (double)fabsf(e);
    c += 1;
  }
}

template <typename T>
__global__ void __launch_bounds__(kErrThreads) err_partial(const T* __restrict__ e, const T* __restrict__ a,
                                                           long long n, int metric, int vec,
                                                           double* ps, double* pt, long long* pc) {
  double s = 0, t = 0;
  long long c = 0;
  const long long tid = (long long)blockIdx.x * kErrThreads + threadIdx.x;
  const long long nth = (long long)kErrBlocks * kErrThreads;
  constexpr int V = 16 / sizeof(T);
  long long done = 0;
  if (vec) {  // 16-B vector loads, 2 in flight per thread
    const long long nv = n / V;
    const uint4* e4 = reinterpret_cast<const uint4*>(e);
    const uint4* a4 = reinterpret_cast<const uint4*>(a);
    for (long long i = tid; i < nv; i += nth) {
      const uint4 ue = __ldg(e4 + i), ua = __ldg(a4 + i);
      const T* pe = reinterpret_cast<const T*>(&ue);
      const T* pa = reinterpret_cast<const T*>(&ua);
#pragma unroll
      for (int k = 0; k < V; ++k) err_term<T>(metric, pe[k], pa[k], s, t, c);
    }
    done = nv * V;
  }
  for (long long i = done + tid; i < n; i += nth) err_term<T>(metric, e[i], a[i], s, t, c);

  __shared__ double ss[kErrThreads], st[kErrThreads];
  __shared__ long long sc[kErrThreads];
  ss[threadIdx.x] = s;
  st[threadIdx.x] = t;
  sc[threadIdx.x] = c;
  __syncthreads();
  for (int k = kErrThreads / 2; k > 0; k >>= 1) {
    if (threadIdx.x < k) {
      ss[threadIdx.x] += ss[threadIdx.x + k];
      st[threadIdx.x] += st[threadIdx.x + k];
      sc[threadIdx.x] += sc[threadIdx.x + k];
    }
    __syncthreads();
  }
  if (threadIdx.x == 0) {
    ps[blockIdx.x] = ss[0];
    pt[blockIdx.x] = st[0];
    pc[blockIdx.x] = sc[0];
  }
}

// one block: thread t sums partials t, t + 256, ... in index order, then a
// fixed-order shared-memory tree (deterministic; the former one-thread loop
// over 3 x 592 partials was a 65-us serial tail)
__global__ void __launch_bounds__(kErrThreads) err_final(const double* ps, const double* pt, const long long* pc,
                                                         int nparts, double* out) {
  __shared__ double ss[kErrThreads], st[kErrThreads];
  __shared__ long long sc[kErrThreads];
  double s = 0, t = 0;
  long long c = 0;
  for (int i = threadIdx.x; i < nparts; i += kErrThreads) { s += ps[i]; t += pt[i]; c += pc[i]; }
  ss[threadIdx.x] = s;
  st[threadIdx.x] = t;
  sc[threadIdx.x] = c;
  __syncthreads();
  for (int k = kErrThreads / 2; k > 0; k >>= 1) {
    if (threadIdx.x < k) {
      ss[threadIdx.x] += ss[threadIdx.x + k];
      st[threadIdx.x] += st[threadIdx.x + k];
      sc[threadIdx.x] += sc[threadIdx.x + k];
    }
    __syncthreads();
  }
  if (threadIdx.x == 0) {
    out[0] = ss[0];
    out[1] = st[0];
    out[2] = (double)sc[0];
  }
}

// scratch: 3 * kErrBlocks + 3 doubles
cudaError_t launch_error(int is_u8, const void* exact, const void* approx, long long n, int metric, double* scratch,
                         cudaStream_t s) {
  double* ps = scratch;
  double* pt = ps + kErrBlocks;
  long long* pc = reinterpret_cast<long long*>(pt + kErrBlocks);
  double* out = reinterpret_cast<double*>(pc + kErrBlocks);
  const int vec = ((reinterpret_cast<uintptr_t>(exact) | reinterpret_cast<uintptr_t>(approx)) & 15) == 0;
  if (is_u8)
    err_partial<uint8_t><<<kErrBlocks, kErrThreads, 0, s>>>(static_cast<const uint8_t*>(exact),
                                                            static_cast<const uint8_t*>(approx), n, metric, vec,
                                                            ps, pt, pc);
  else
    err_partial<float><<<kErrBlocks, kErrThreads, 0, s>>>(static_cast<const float*>(exact),
                                                          static_cast<const float*>(approx), n, metric, vec, ps,
                                                          pt, pc);
  err_final<<<1, kErrThreads, 0, s>>>(ps, pt, pc, kErrBlocks, out);
  return cudaGetLastError();
}

size_t error_scratch_doubles() { return 3 * (size_t)kErrBlocks + 3; }

}  // namespace kp
