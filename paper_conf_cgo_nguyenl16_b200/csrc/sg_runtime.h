// sg_runtime.h -- plan object and runtime of the stream-graph executor.
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <map>
#include <string>
#include <vector>

#include "sg_codegen.h"
#include "sg_internal.h"

namespace sg {

struct CompiledKernel {
    KernelInfo ki;
    std::string cubin;
    std::string log;
    // per physical device (index = device ordinal)
    std::vector<CUmodule> mod;
    std::vector<CUfunction> fn;            // main variant (TMA pipeline when ki.has_tma)
    std::vector<CUfunction> fn_sync;       // register mode: synchronous fallback; staged: stream-start variant
    std::vector<int> max_blocks_per_sm;
    std::vector<int> max_blocks_sync;
    // feedback loop state (per device): live buffer and the stream-start image
    std::vector<void*> state, state0;
    // staged kernels: side stream + fork/join events for the stream-start variant (per device)
    std::vector<cudaStream_t> aux;
    std::vector<cudaEvent_t> ev_fork, ev_join;
};

struct CutRing {          // one boundary stream between partitions (a PDG edge member)
    int edge = -1;                     // representative cut edge (Plan::ring_rep)
    int group = 0;                     // replica group owning this ring
    int src_part = -1, dst_part = -1;  // -1: graph input / output
    std::vector<int> dst_parts;        // every consumer partition (a duplicated stream shipped once)
    int src_gpu = 0, dst_gpu = 0;
    int64_t lo = 0, extra = 0, per_iter = 0;
    int64_t slot_items = 0;
    std::vector<void*> src_slots, dst_slots;  // device buffers (dst == src when same GPU)
    std::vector<void*> host_slots;            // SG_TRANSPORT_HOST: pinned staging buffer per slot
    std::vector<cudaEvent_t> ev_copied, ev_consumed, ev_produced;
};

struct IoBinding {
    std::vector<const void*> in;
    std::vector<int64_t> in_base, in_limit;
    std::vector<void*> out;
    std::vector<int64_t> out_base;
};

struct RankOp {
    int32_t op, part, edge, peer;
    int64_t frag, kb, ke, items;
};

struct GpuCtx {
    int dev = 0;
    cudaStream_t compute = nullptr, copy = nullptr;
    cudaEvent_t ev_start = nullptr, ev_done = nullptr;
};

struct Plan {
    Flat flat;
    int G = 1;
    int R = 1, Gs = 1;                     // replica groups, GPUs per group (G = R * Gs)
    sg_plan_opts opts{};
    std::vector<Partition> parts;
    std::vector<int> part_order;           // topological order of partitions
    std::vector<CompiledKernel> kernels;   // one per partition
    std::vector<int> devices;              // logical gpu -> physical device
    bool virtual_gpus = false;
    double est_tmax = 0;
    bool ilp_optimal = false;
    bool chain_fission = false;            // p.flat is the chain-fissioned graph
    std::vector<PdgEdge> pdg;
    // cut edges: the edge whose ring carries this edge's items (itself, or -- for outputs of one duplicate
    // splitter whose consumers sit on the same other GPU -- the lowest such edge: the stream is shipped
    // once per destination GPU, SURVEY.md 8(c)-4 reading 15); -1 for edges inside a partition
    std::vector<int> ring_rep;
    std::vector<int64_t> ring_lo, ring_extra;  // per representative: union of its members' windows
    void cut_window(int e, int64_t& lo, int64_t& extra) const {
        const int r = ring_rep.empty() || ring_rep[e] < 0 ? e : ring_rep[e];
        if (!ring_lo.empty() && ring_rep[e] >= 0) { lo = ring_lo[r]; extra = ring_extra[r]; return; }
        edge_window(flat, e, lo, extra);
    }
    // info arrays
    std::vector<int64_t> reps, ninit;
    std::vector<int32_t> node_type, node_kind, node_part, part_gpu, part_mode;
    std::vector<double> part_time;
    int input_gpu = 0, output_gpu = 0;
    int64_t iters_per_fragment = 0;
    // runtime state (created lazily)
    bool rt_ready = false;
    std::vector<GpuCtx> gpus;
    std::vector<CutRing> rings;
    int64_t rt_fragment = 0;
    int ring_depth = 2;
    int64_t last_launches = 0;
    cudaEvent_t user_ev = nullptr;

    // sg_run_host staging (device buffers reused across calls)
    void* host_in_dev = nullptr;
    void* host_out_dev = nullptr;
    size_t host_in_cap = 0, host_out_cap = 0;
    cudaStream_t host_stream = nullptr;
    cudaStream_t host_in_stream = nullptr, host_out_stream = nullptr;  // chunked copy pipeline
    std::vector<cudaEvent_t> host_ev;
    // set by run_host for a multi-partition plan: run() copies each fragment's input prefix in and its
    // output range out on the host streams, interleaved with the fragment pipeline
    const void* pipe_hin = nullptr;
    void* pipe_hout = nullptr;
    std::vector<cudaEvent_t> pipe_ev;

    // one process per GPU (sg_dist.cpp)
    void* comm = nullptr;  // ncclComm_t
    int comm_rank = 0, comm_device = 0;
    bool dist_ready = false;
    int64_t dist_F = 0;
    std::map<int, std::vector<void*>> dist_slots;
    std::map<int, std::vector<cudaEvent_t>> dist_ev;
    cudaStream_t dist_compute = nullptr, dist_comm = nullptr;
    cudaEvent_t dist_join = nullptr;

    ~Plan();
    void run(const void* in, int64_t n, void* out, cudaStream_t stream);
    void run_host(const void* hin, int64_t n, void* hout);
    void profile_partitions(int64_t n, int reps, double* ns_per_iter);
    void comm_init(int nranks, int rank, const uint8_t id[128], int device);
    void run_rank(const void* in, int64_t n, void* out, cudaStream_t stream);
    void dist_release();
};

int64_t launch_kernel(CompiledKernel& ck, int dev, const IoBinding& io, int64_t kb, int64_t ke, cudaStream_t stream,
                      bool is_f32);
// feedback-loop partitions: (allocate and) reset the persistent state to its stream-start image on `stream`
void reset_state(CompiledKernel& ck, int dev, cudaStream_t stream);
int64_t fragment_size(const Plan& p, int64_t n);
std::vector<RankOp> rank_schedule(const Plan& p, int rank, int64_t n, int64_t F);
void nccl_unique_id(uint8_t out[128]);

// NVRTC -> sm_100a cubin (cached by content hash in memory and on disk).
void compile_kernel(CompiledKernel& ck, int verbose);
std::string nvrtc_version();

}  // namespace sg
