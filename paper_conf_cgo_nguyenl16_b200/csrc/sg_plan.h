// sg_plan.h -- planner: PEE, Algorithm 1, PDG, ILP mapping, plan assembly.
#pragma once
#include <array>
#include <vector>

#include "sg_internal.h"
#include "sg_runtime.h"

namespace sg {

// B200 performance-estimation engine (section 3.3, re-derived
// for sm_100a): estimate of one partition, ns per steady-state iteration.
// Work a partition's kernel executes per steady-state iteration, after the code generator's view
// resolution, dead-firing elimination, zero-tap pruning and CSE (sg_pee.cpp).
struct PartitionWork {
    double flops = 0, intops = 0, dfma = 0;   // executed fp32 flops (FMA = 2), integer ops, fp64 ops
    double reads = 0, writes = 0;             // items read (non-zero peek items) / written by live firings
    double firings = 0;                       // live firings
    double in_bytes = 0, out_bytes = 0;       // boundary streams
    int in_edges = 0, out_edges = 0;          // boundary edges (each a load / store stream of its own)
    double row_items = 0;                     // register mode: items of one iteration held by one thread
    int components = 0;                       // register-eligible: independent dependence components of an
                                              // iteration (outputs sharing no input item); 0 otherwise
    double halo_firings = 0;                  // firings recomputed per tile (peek halos)
    double loop_firings = 0;                  // feedback loops: sequential firings per iteration
    int levels = 0;                           // longest chain of compute nodes
    int cse_nodes = 0;                        // compute nodes found identical to an earlier one
    bool frame = false;                       // contains frame FIRs (BEAM_FIR)
};
PartitionWork partition_work(const Flat& f, const std::vector<int>& nodes, bool components = false);

struct PeeEstimate {
    double t = 0, t_comp = 0, t_dt = 0;
    int mode = 0;
    bool bitslice = false;
    double bitslice_ops = 0;  // bitslice mode: 32-lane ALU ops per iteration
    bool fused = true;        // staged mode: the fused path is expected (every view map affine)
    PartitionWork work;
    bool io_bound() const { return t_dt >= t_comp; }
};
PeeEstimate pee_estimate(const Flat& f, const std::vector<int>& nodes);
// The estimate refined with the generated kernel's own decisions (fused path, tile, register variant):
// ns per iteration, steady state (no launch term).
double pee_refine(const PeeEstimate& est, const KernelInfo& ki);
double launch_ns_per_iter(int64_t iters_per_fragment);  // per-fragment kernel launch, amortised per iteration

// The paper's analytic model Eq. III.8-III.12, kept as a
// reference implementation for tests and reports (calibrated for M2090).
double paper_model(const std::vector<double>& t, const std::vector<double>& fr, int S, int W, int F, double D,
                   double C1, double C2, double* tcomp, double* tdt, double* tdb);

bool is_convex(const Flat& f, const std::vector<char>& in_set);

// Algorithm 1.  cap > 0 limits T(merged) (G-aware).
std::vector<std::vector<int>> algorithm1(const Flat& f, double cap, int64_t iters_per_fragment = 0);

// ILP of Eq. III.1-III.7 solved exactly by branch and bound (or brute force).
struct MapResult {
    std::vector<int> assign;
    double tmax = 0;
    bool optimal = false;
};
MapResult map_partitions(const std::vector<double>& T, const std::vector<PdgEdge>& pdg, const Topology& topo,
                         double lat, double bw, int time_limit_ms, int method, long long node_limit = 0);
double mapping_cost(const std::vector<double>& T, const std::vector<PdgEdge>& pdg, const Topology& topo, double lat,
                    double bw, const std::vector<int>& assign);

void build_plan(Plan& p, const sg_graph& g, int G, const sg_plan_opts& o);

}  // namespace sg
