// sg_aux.cu -- nvcc-compiled (sm_100a) helper kernels of the runtime.
//   sg_flush_l2: evict L2 (126 MB on B200) between timed iterations (benchmark
//                hygiene): overwrite a scratch buffer larger than L2, then read it
//                back so the dirty lines are written back before the timed window
//                opens (the next kernel starts with a cold, clean L2).
#include <cuda_runtime.h>
#include <stdint.h>

#include "../../include/sg.h"

__global__ void __launch_bounds__(256) sg_flush_write(int4* p, size_t n16, int salt) {
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n16; i += (size_t)gridDim.x * blockDim.x)
        p[i] = make_int4((int)i, salt, (int)(i >> 32), salt ^ (int)i);
}

__global__ void __launch_bounds__(256) sg_flush_read(const int4* p, size_t n16, int* sink) {
    int acc = 0;
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n16; i += (size_t)gridDim.x * blockDim.x) {
        int4 v = __ldcg(p + i);
        acc ^= v.x ^ v.y ^ v.z ^ v.w;
    }
    if (acc == 0x7fffffff) *sink = acc;  // practically never taken; keeps the loads alive
}

extern "C" sg_status sg_flush_l2(void* scratch, int64_t bytes, void* stream) {
    static int salt = 0;
    if (!scratch || bytes < 64) return SG_E_ARG;
    size_t n16 = (size_t)bytes / 16 - 1;  // last 16 bytes: sink
    int* sink = (int*)((char*)scratch + n16 * 16);
    sg_flush_write<<<148 * 8, 256, 0, (cudaStream_t)stream>>>((int4*)scratch, n16, ++salt);
    sg_flush_read<<<148 * 8, 256, 0, (cudaStream_t)stream>>>((const int4*)scratch, n16, sink);
    return cudaGetLastError() == cudaSuccess ? SG_OK : SG_E_CUDA;
}
