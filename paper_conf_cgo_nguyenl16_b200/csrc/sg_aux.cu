// sg_aux.cu -- nvcc-compiled (sm_100a) helper kernels of the runtime.
//   sg_flush_l2: overwrite a scratch buffer larger than L2 (126 MB on B200)
//                between timed iterations (benchmark hygiene).
#include <cuda_runtime.h>
#include <stdint.h>

#include "../../include/sg.h"

__global__ void __launch_bounds__(256) sg_flush_kernel(int4* p, size_t n16, int salt) {
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n16; i += (size_t)gridDim.x * blockDim.x)
        p[i] = make_int4((int)i, salt, (int)(i >> 32), salt ^ (int)i);
}

extern "C" sg_status sg_flush_l2(void* scratch, int64_t bytes, void* stream) {
    static int salt = 0;
    if (!scratch || bytes < 16) return SG_E_ARG;
    size_t n16 = (size_t)bytes / 16;
    sg_flush_kernel<<<148 * 8, 256, 0, (cudaStream_t)stream>>>((int4*)scratch, n16, ++salt);
    return cudaGetLastError() == cudaSuccess ? SG_OK : SG_E_CUDA;
}
