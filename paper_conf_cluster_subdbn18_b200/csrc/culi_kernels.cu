// culi_kernels.cu — sm_100a kernels of libculi.so: image relocation, batch eval (one thread per form,
// warps take consecutive forms of the binned order), define (sequential), result export.
// The eval/apply machine itself is culi_machine.cuh.
#include <cuda_runtime.h>
#include <stdint.h>

#include "culi_machine.cuh"

namespace culi {

// Relocate an uploaded image in place: image-local indices -> heap indices.
__global__ void culi_relocate_kernel(uint8_t* tag, uint64_t* word, uint64_t base, uint64_t n,
                                     uint32_t str_base, uint32_t* roots, uint32_t nroots) {
  uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
    uint64_t g = base + i;
    uint32_t t = tag[g] & KIND_MASK;
    if (t == K_CONS) {
      uint64_t w = word[g];
      uint32_t a = lo32(w), b = hi32(w);
      a = a < IMG_FIRST ? a : (uint32_t)(base + a - IMG_FIRST);
      b = b < IMG_FIRST ? b : (uint32_t)(base + b - IMG_FIRST);
      word[g] = pack2(a, b);
    } else if (t == K_STR) {
      uint64_t w = word[g];
      word[g] = pack2(lo32(w) + str_base, hi32(w));
    }
  }
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nroots; i += stride) {
    uint32_t r = roots[i];
    roots[i] = r < IMG_FIRST ? r : (uint32_t)(base + r - IMG_FIRST);
  }
}

__device__ __forceinline__ void write_result(const EvalArgs& A, uint32_t f, const FormOut& o) {
  A.rtag[f] = o.err ? (uint8_t)K_ERROR : (uint8_t)o.t;
  A.rerr[f] = o.err;
  A.rsteps[f] = o.steps;
  A.rword[f] = o.w;
  if (o.err == E_OOM) atomicExch(&A.flags[0], 1);
}

__device__ __forceinline__ Ctx make_ctx(const EvalArgs& A, uint32_t slot) {
  Ctx C;
  C.A = &A;
  C.kb = A.kst + slot;
  C.vb = A.vst + slot;
  return C;
}

// Batch mode.  Shared memory per block: the persistent code segment [code_lo, code_lo + code_n) as
// {w.lo, w.hi, tag, 0} and the global frame [0, gst) ("stage").  Each warp takes 32
// consecutive forms of the (binned) order with one atomicAdd and runs them to completion.
__global__ void __launch_bounds__(128) culi_eval_kernel(const __grid_constant__ EvalArgs A) {
  uint4* scode = culi_smem;
  uint64_t* sgword = reinterpret_cast<uint64_t*>(culi_smem + A.code_n);
  uint8_t* sgtag = reinterpret_cast<uint8_t*>(sgword + A.gst);
  for (uint32_t i = threadIdx.x; i < A.code_n; i += blockDim.x) {
    uint64_t w = A.H.word[A.code_lo + i];
    scode[i] = make_uint4(lo32(w), hi32(w), A.H.tag[A.code_lo + i], 0);
  }
  for (uint32_t i = threadIdx.x; i < A.gst; i += blockDim.x) {
    sgword[i] = A.H.gword[i];
    sgtag[i] = A.H.gtag[i];
  }
  __syncthreads();
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  Ctx C = make_ctx(A, slot);
  int lane = threadIdx.x & 31;
  for (;;) {
    uint32_t b = 0;
    if (lane == 0) b = atomicAdd(A.next, 32u);
    b = __shfl_sync(0xffffffffu, b, 0);
    if (b >= A.nforms) break;
    uint32_t i = b + lane;
    if (i < A.nforms) {
      uint32_t f = A.perm ? A.perm[i] : i;
      FormOut o = eval_form(C, A.roots[f]);
      write_result(A, f, o);
    }
  }
}

// Define mode (culi_define): forms evaluated in order by one thread; define/defun/defmacro write the
// global frame; stops at the first error.  No staging: this kernel writes globals.
__global__ void culi_define_kernel(const __grid_constant__ EvalArgs A) {
  if (blockIdx.x != 0 || threadIdx.x != 0) return;
  Ctx C = make_ctx(A, 0);
  for (uint32_t f = 0; f < A.nforms; ++f) {
    FormOut o = eval_form(C, A.roots[f]);
    write_result(A, f, o);
    if (o.err) {
      A.flags[1] = (int)f + 1;
      A.flags[2] = o.err;
      return;
    }
  }
}

// Export: serialize every CONS/STR result into pre-order tokens {word, tag}; the
// record's word becomes offset | count << 32.  The thread's V-stack is the DFS stack.
__global__ void __launch_bounds__(128) culi_export_kernel(ExportArgs X) {
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  uint32_t nthreads = gridDim.x * blockDim.x;
  for (uint32_t f = slot; f < X.nforms; f += nthreads) {
    uint32_t t = X.rtag[f];
    if (t != K_CONS && t != K_STR) continue;
    uint32_t root = (uint32_t)X.rword[f];
    unsigned long long ntok = 0;
    uint32_t sp = 0, n = root;
    bool ovf = false;
    for (;;) {                                     // pass 1: count tokens
      ++ntok;
      if ((X.tag[n] & KIND_MASK) == K_CONS) {
        uint64_t w = X.word[n];
        if (sp >= X.vcap) { ovf = true; break; }
        X.vst[(size_t)sp * X.nslots + slot].x = hi32(w);
        ++sp;
        n = lo32(w);
        continue;
      }
      if (sp == 0) break;
      --sp;
      n = X.vst[(size_t)sp * X.nslots + slot].x;
    }
    if (ovf) { atomicExch(&X.flags[4], 1); continue; }
    unsigned long long off = atomicAdd(X.pcount, ntok);
    if (off + ntok > X.pcap) { atomicExch(&X.flags[3], 1); continue; }
    n = root;
    sp = 0;
    unsigned long long k = off;
    for (;;) {                                     // pass 2: write tokens
      uint32_t nt = X.tag[n] & KIND_MASK;
      uint64_t w = X.word[n];
      X.payload[k++] = make_uint4(lo32(w), hi32(w), nt, 0);
      if (nt == K_CONS) {
        X.vst[(size_t)sp * X.nslots + slot].x = hi32(w);
        ++sp;
        n = lo32(w);
        continue;
      }
      if (sp == 0) break;
      --sp;
      n = X.vst[(size_t)sp * X.nslots + slot].x;
    }
    X.rword[f] = (off & 0xffffffffull) | (ntok << 32);
  }
}

__global__ void culi_reset_kernel(unsigned long long* top, unsigned long long top_value, uint32_t* next,
                                  unsigned long long* pcount, int* flags) {
  *top = top_value;
  *next = 0;
  *pcount = 0;
  for (int k = 0; k < 8; ++k) flags[k] = 0;
}

// ---- host launchers ----------------------------------------------------------------------------------
cudaError_t launch_relocate(cudaStream_t s, uint8_t* tag, uint64_t* word, uint64_t base, uint64_t n,
                            uint32_t str_base, uint32_t* roots, uint32_t nroots, int sms) {
  uint64_t work = n > nroots ? n : nroots;
  uint64_t blocks = (work + 255) / 256;
  if (blocks > (uint64_t)sms * 16) blocks = (uint64_t)sms * 16;
  if (blocks == 0) blocks = 1;
  culi_relocate_kernel<<<(unsigned)blocks, 256, 0, s>>>(tag, word, base, n, str_base, roots, nroots);
  return cudaGetLastError();
}

size_t eval_smem_bytes(const EvalArgs& A) {
  return (size_t)A.code_n * sizeof(uint4) + (size_t)A.gst * 9 + 16;
}

cudaError_t launch_eval(cudaStream_t s, const EvalArgs& A, uint32_t blocks) {
  size_t smem = eval_smem_bytes(A);
  if (smem > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(culi_eval_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                         (int)smem);
    if (e != cudaSuccess) return e;
  }
  culi_eval_kernel<<<blocks, 128, smem, s>>>(A);
  return cudaGetLastError();
}

cudaError_t launch_define(cudaStream_t s, const EvalArgs& A) {
  culi_define_kernel<<<1, 32, 0, s>>>(A);
  return cudaGetLastError();
}

cudaError_t launch_export(cudaStream_t s, const ExportArgs& X, uint32_t blocks) {
  culi_export_kernel<<<blocks, 128, 0, s>>>(X);
  return cudaGetLastError();
}

cudaError_t launch_reset(cudaStream_t s, unsigned long long* top, unsigned long long top_value,
                         uint32_t* next, unsigned long long* pcount, int* flags) {
  culi_reset_kernel<<<1, 1, 0, s>>>(top, top_value, next, pcount, flags);
  return cudaGetLastError();
}

}  // namespace culi
