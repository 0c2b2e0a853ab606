// sg_codegen.h -- per-partition CUDA code generation.
#pragma once
#include <string>
#include <vector>

#include "sg_internal.h"

namespace sg {

struct CodegenOpts {
    int mode = 0;        // 0 auto, 1 register, 2 staged
    int threads = 0;     // 0 auto
    int tile = 0;        // staged: iterations per tile (0 auto)
    int smem_budget = 0; // bytes per CTA (0 = auto)
};

// What the runtime needs to launch a generated kernel.
struct KernelInfo {
    std::string name;
    std::string source;       // full CUDA source (includes sg_device.cuh)
    int mode = 0;             // 1 register (thread per iteration), 2 staged, 4 feedback loop (sequential)
    int threads = 0;          // CTA size
    int tile = 0;             // iterations per CTA tile
    int min_blocks = 1;       // __launch_bounds__ second argument
    size_t smem = 0;          // dynamic shared memory bytes
    std::vector<int> in_edges, out_edges;   // boundary edges (flat edge ids), argument order
    // per boundary edge: window of local positions needed/produced by one range
    // of W iterations: [lo, lo + per_iter*W + extra)
    std::vector<int64_t> in_lo, in_extra, out_lo, out_extra;
    int64_t flops_per_iter = 0;     // algorithmic fp32 flops (FMA = 2), as written
    int64_t intops_per_iter = 0;    // algorithmic integer ops (CE = 2 min/max)
    int64_t dfma_per_iter = 0;
    int n_levels = 0;
    // register mode: the TMA-pipelined variant (name) and the synchronous fallback (name_sync)
    std::string name_sync;
    bool has_tma = false;
    int tma_in = 0, tma_out = 0;     // 1: 2-D tensor map + 128B swizzle, 2: per-row bulk copies
    int64_t pin = 0, pout = 0, off_in = 0, off_out = 0;
    int threads_sync = 0, tile_sync = 0;
    size_t smem_sync = 0;
    bool fused = false;              // staged mode: fused fast path present
    int reg_variant = 0;             // register mode: 0 TMA / synchronous rows, 1 in-place components (bulk
                                     // copies), 2 demand-ordered wide single-component rows
    int64_t flops_exec_per_iter = -1;  // fused: algorithmic flops after dead/zero pruning (no recompute)
    std::string name_start;          // staged fused: stream-start variant (tiles with k0 < ksafe)
    int demand_runs = 1;             // register demand-ordered: warps (output-group runs) per iteration row
    double par_eff = 1.0;            // fused frame-FIR levels: ideal FFMA issue / simulated issue (<= 1)
    int split_level = 0;             // > 0: a frame-FIR level that cannot fill the CTA starts at this level
    std::vector<std::pair<int, int>> node_level;  // fused: (flat node, level) of every node of the partition
    int64_t ksafe = 0;
    // feedback loop (mode 4): persistent state (4-byte words) and its image at the stream start
    int64_t state_words = 0;
    std::vector<uint32_t> state_init;
};

// Boundary input / output edges of a node set (sorted, deterministic).
void partition_boundary(const Flat& f, const std::vector<int>& nodes, std::vector<int>& ins, std::vector<int>& outs);

// Window [lo, lo + per_iter*W + extra) of local positions a range of W iterations
// reads on edge e (its consumer's needs; graph output: the produced positions).
void edge_window(const Flat& f, int e, int64_t& lo, int64_t& extra);

bool register_mode_eligible(const Flat& f, const std::vector<int>& nodes, std::string* why);
// all compute filters are bit kinds (INTO_BITS / BITS_TO_INT / XOR / XOR_CONST / SBOX): bitslice mode
bool bitslice_eligible(const Flat& f, const std::vector<int>& nodes, std::string* why);

KernelInfo generate_kernel(const Flat& f, const std::vector<int>& nodes, int part_id, const CodegenOpts& opt);

// Algorithmic work of one node per steady-state iteration (as written).
void node_work(const Flat& f, int v, int64_t& flops, int64_t& intops, int64_t& dfma);

bool is_view_kind(int kind);

extern const char* kDeviceHeader;  // sg_device.cuh contents (embedded)

}  // namespace sg
