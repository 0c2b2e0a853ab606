/*
 * sg.h -- C ABI of the B200-native synchronous-dataflow stream-graph executor.
 *
 * Follows the problem statement of Nguyen & Lee:
 *   input  = a stream graph: filters (nodes) with firing rates, edges weighted
 *            by their buffer size, composed by pipeline / split-join
 *            (section 2.1.1; section 3.1),
 *            plus the number of GPUs G and their topology (PAPER.md:494-502,
 *            section 3.2.2);
 *   output = partitions and a partition->GPU mapping minimising Tmax
 *            (Eq. III.1-III.7), then generated kernels and
 *            their pipelined execution.
 *
 * Conventions (all calls):
 *   - Every call returns sg_status (0 = SG_OK, < 0 = error) unless noted.
 *     No C++ exception crosses this boundary.  sg_last_error() returns a
 *     thread-local message describing the last failure on the calling thread.
 *   - Handles are opaque and owned by the caller; destroy them with the
 *     matching *_destroy.  Distinct handles may be used from distinct threads;
 *     one handle is not thread-safe.
 *   - Streams are in NATURAL ORDER at the boundary: item i of the input stream
 *     is input[i]; item i of the output stream is output[i].  Items are 4-byte
 *     words of the graph's dtype.
 *   - There is no CPU fallback: sg_run needs a CUDA device (sm_100a) and fails
 *     with SG_E_CUDA otherwise.  Graph building, sg_plan (rates, partitioning,
 *     ILP mapping, code generation and NVRTC compilation to sm_100a cubins) and
 *     the size queries work without a GPU.
 */
#ifndef SG_H_
#define SG_H_

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
    SG_OK = 0,
    SG_E_ARG = -1,          /* bad argument (NULL handle, negative size, bad kind params) */
    SG_E_STRUCTURE = -2,    /* ill-formed hierarchy (unclosed split-join, empty graph, ...) */
    SG_E_RATE = -3,         /* balance equations inconsistent */
    SG_E_UNSUPPORTED = -4,  /* kind/dtype combination not supported */
    SG_E_NOMEM = -5,        /* host or device allocation failed */
    SG_E_CUDA = -6,         /* CUDA driver/runtime/NVRTC failure, or no device */
    SG_E_COMM = -7,         /* inter-GPU transport failure */
    SG_E_PLAN = -8,         /* partitioning / mapping failed (e.g. ILP infeasible) */
    SG_E_SIZE = -9          /* a partition does not fit the device (shared memory) */
} sg_status;

typedef enum { SG_F32 = 0, SG_I32 = 1 } sg_dtype;

/* Splitters: duplicate or weighted round-robin.  Joiners are always weighted
 * round-robin (StreamIt `roundrobin`; default weight 1). */
typedef enum { SG_SPLIT_DUPLICATE = 0, SG_SPLIT_ROUNDROBIN = 1 } sg_split_kind;

/*
 * Filter kinds.  PAPER.md defines no filter body; the semantics below are the
 * readings of SURVEY.md 8(c)-3, repeated in DESIGN.md ("Readings").  x[i] is
 * peek(i) (oldest first), y[j] the j-th pushed item.  FMA means one IEEE
 * fused multiply-add; all other operations are single IEEE float operations.
 *
 *  kind                  p_i                p_f              peek / pop / push
 *  SG_K_IDENTITY         -                  -                1 / 1 / 1
 *  SG_K_FIR              {L, pop}           c[L]             max(L,pop)/pop/1: acc=0; acc=FMA(x[i],c[i],acc) i<L
 *  SG_K_DELAY            {k}                -                prework pushes k zeros, then 1/1/1
 *  SG_K_DECIMATE         {M}                -                M/M/1: y = x[0]
 *  SG_K_EXPAND           {M}                -                1/1/M: x[0], then M-1 zeros
 *  SG_K_COMPARE_EXCHANGE {up}               -                2/2/2: (min,max) if up else (max,min); signed
 *  SG_K_FFT_REORDER      {n}                -                2n/2n/2n: even complex items, then odd
 *  SG_K_COMBINE_DFT      {j}                -                2j/2j/2j: j/2 radix-2 butterflies, w=e^{-2 pi i k/j}
 *  SG_K_FM_DEMOD         -                  {gain}           2/1/1: (float)(gain * atan((double)(x0*x1)))
 *  SG_K_SUBTRACT         -                  -                2/2/1: x1 - x0
 *  SG_K_AMPLIFY          -                  {k}              1/1/1: x0 * k
 *  SG_K_ADD              {n}                -                n/n/1: s=0; s=s+x[i] in order (i32: wrapping)
 *  SG_K_BEAM_FIR         {L, dec, frame}    wr[L], wi[L]     2F/2F/2F/dec: per-frame complex FIR, zero history
 *  SG_K_BEAMFORM         {nch}              wr[nch], wi[nch] 2nch/2nch/2: complex weighted sum
 *  SG_K_MAGNITUDE        -                  -                2/2/1: sqrt(FMA(a,a,b*b))
 *  SG_K_MULTIPLY         -                  -                2/2/1: x0 * x1 (MatMul's pairwise product)
 *  --- DES on a bit-per-item stream (Fig. 4.2a), SG_I32 only except PERMUTE:
 *  SG_K_PERMUTE          {n, idx[m]}        -                n/n/m: y[k] = x[idx[k]], 0 <= idx < n (any dtype)
 *  SG_K_XOR              {n}                -                2n/2n/n: y[i] = x[i] ^ x[n+i]
 *  SG_K_XOR_CONST        {n, k[n]}          -                n/n/n: y[i] = x[i] ^ k[i]
 *  SG_K_SBOX             {t[64]}            -                6/6/4: b_i = x[i]&1; v = t[16(2b0+b5) + 8b1+4b2+2b3+b4];
 *                                                            y[i] = (v >> (3-i)) & 1 (FIPS 46-3 S-box, t in [0,15])
 *  SG_K_INTO_BITS        -                  -                1/1/32: y[k] = (x >> (31-k)) & 1 (MSB first)
 *  SG_K_BITS_TO_INT      -                  -                32/32/1: y = sum_k (x[k]&1) << (31-k)
 *
 * dtype SG_I32 admits IDENTITY, DELAY, DECIMATE, EXPAND, COMPARE_EXCHANGE, ADD.
 */
typedef enum {
    SG_K_IDENTITY = 0,
    SG_K_FIR = 1,
    SG_K_DELAY = 2,
    SG_K_DECIMATE = 3,
    SG_K_EXPAND = 4,
    SG_K_COMPARE_EXCHANGE = 5,
    SG_K_FFT_REORDER = 6,
    SG_K_COMBINE_DFT = 7,
    SG_K_FM_DEMOD = 8,
    SG_K_SUBTRACT = 9,
    SG_K_AMPLIFY = 10,
    SG_K_ADD = 11,
    SG_K_BEAM_FIR = 12,
    SG_K_BEAMFORM = 13,
    SG_K_MAGNITUDE = 14,
    SG_K_MULTIPLY = 15,
    SG_K_PERMUTE = 16,
    SG_K_XOR = 17,
    SG_K_XOR_CONST = 18,
    SG_K_SBOX = 19,
    SG_K_INTO_BITS = 20,
    SG_K_BITS_TO_INT = 21
} sg_filter_kind;

typedef struct {
    sg_filter_kind kind;
    int32_t n_i;
    const int32_t* p_i; /* copied by sg_add_filter; caller keeps ownership */
    int32_t n_f;
    const float* p_f;   /* copied by sg_add_filter; caller keeps ownership */
} sg_filter_desc;

/* Handle type names carry a _t / _s suffix so that they do not collide with
 * the function sg_plan() in C's ordinary identifier namespace. */
typedef struct sg_graph sg_graph;
typedef struct sg_plan_s sg_plan_t;

/* Partitioner selection for sg_plan_opts.partitioner. */
enum {
    SG_PART_ALGORITHM1 = 0, /* the paper's Algorithm 1 with the B200 PEE */
    SG_PART_SINGLE = 1,     /* one partition (SPSG baseline) */
    SG_PART_PER_FILTER = 2, /* one partition per filter (splitters/joiners ride along) */
    SG_PART_USER = 3,       /* node_partition[] supplied by the caller */
    SG_PART_CHAIN = 4       /* one partition per chain-fission group (needs chain_groups >= 2); nodes before
                               the fissioned split-join join the first group, nodes after it the last */
};

/* Where boundary streams between GPUs travel (P2P) in the one-process runtime
 * (sg_run); the one-process-per-GPU runtime (sg_run_rank) always uses NCCL send/recv and ignores it.
 * sg_plan rejects any other value with SG_E_ARG. */
enum {
    SG_TRANSPORT_AUTO = 0,  /* cudaMemcpyPeerAsync between distinct devices; D2D cudaMemcpyAsync between
                               virtual GPUs on one device */
    SG_TRANSPORT_P2P = 1,   /* cudaMemcpyPeerAsync for every cut edge between GPUs, virtual GPUs included */
    SG_TRANSPORT_HOST = 2   /* host-staged pair, as in [7]: D2H into a pinned host
                               buffer, then H2D, in order on the producer GPU's copy stream */
};

typedef struct sg_plan_opts {
    int32_t partitioner;           /* SG_PART_*; default SG_PART_ALGORITHM1 */
    const int32_t* node_partition; /* SG_PART_USER: partition id per node (flattened order) */
    int32_t n_node_partition;
    int32_t tile_iters;            /* iterations per CTA tile; 0 = chosen by the PEE */
    int32_t threads;               /* threads per CTA; 0 = chosen by the PEE */
    int64_t iters_per_fragment;    /* multi-GPU fragment size; 0 = auto */
    int32_t transport;             /* SG_TRANSPORT_* */
    int32_t virtual_gpus;          /* 1: map the G logical GPUs onto streams of one device */
    const int32_t* devices;        /* physical device per logical GPU (NULL: 0..G-1) */
    int32_t ilp_time_limit_ms;     /* exact branch-and-bound budget; 0 = 10000 */
    int32_t codegen_mode;          /* 0 auto, 1 register (thread per iteration), 2 staged, 3 staged general path only */
    double link_gbps;              /* NVLink bandwidth per direction for the ILP; 0 = 770 */
    double link_latency_us;        /* per-transfer latency Lat (Eq. III.3); 0 = 10 */
    int32_t verbose;
    int32_t plan_only;             /* 1: stop after partitioning and mapping (no code generation,
                                      no NVRTC); sg_run on such a plan returns SG_E_ARG */
    int32_t replicas;              /* hybrid replica x pipeline plans: 0 or 1 = the paper's
                                      pipeline mapping of all partitions onto the G GPUs (Eq. III.5: each
                                      partition on exactly one GPU); R > 1 (R | G) = R replica groups of G/R
                                      GPUs, each holding the whole graph mapped by the ILP onto its G/R GPUs,
                                      fragments dealt round-robin to the groups; -1 = R chosen by the cost
                                      model max(Tmax(G/R)/R, input / output distribution over NVLink).
                                      With sg_comm_init / sg_run_rank, rank g * (G/R) + l is GPU l of group
                                      g and runs fragments f with f % R == g; output fragments land on the
                                      output rank of their group (gathering them is the caller's). */
    int32_t chain_groups;          /* order-preserving chain fission of the largest eligible
                                      split-join (a duplicate splitter and/or a roundrobin(1) joiner feeding
                                      ADD(n_branches)): its branches are cut into contiguous groups; the
                                      splitter becomes a forward chain (each group's splitter relays the
                                      stream to the next), the joiner + ADD an accumulate chain
                                      acc_g = ADD(acc_{g-1}, group g's outputs), bit-identical to the
                                      sequential ADD.  0 = the planner compares the graph as written with its
                                      fission into G/R groups (Algorithm 1 on more than one GPU only) and
                                      keeps the smaller Tmax; -1 = never; k >= 2 = always, k groups (any
                                      partitioner; node ids then refer to the fissioned graph, see
                                      sg_plan_info).  SG_E_PLAN if k >= 2 and nothing is eligible. */
} sg_plan_opts;

typedef struct sg_plan_info_s {
    int32_t n_nodes;                 /* flattened nodes: filters, splitters, joiners */
    int32_t n_edges;
    int32_t n_partitions;
    int32_t n_gpus;
    int64_t in_per_iter;             /* input items consumed per steady-state iteration */
    int64_t out_per_iter;            /* output items produced per steady-state iteration */
    const int64_t* reps;             /* [n_nodes] repetition vector (gcd 1) */
    const int64_t* init_firings;     /* [n_nodes] firings of the init schedule (may be < 0: lag) */
    const int32_t* node_type;        /* [n_nodes] 0 filter, 1 dup splitter, 2 rr splitter, 3 joiner */
    const int32_t* node_kind;        /* [n_nodes] sg_filter_kind or -1 */
    const int32_t* node_partition;   /* [n_nodes] */
    const int32_t* partition_gpu;    /* [n_partitions] */
    const double* partition_time;    /* [n_partitions] PEE estimate T(p), ns per iteration */
    const int32_t* partition_mode;   /* [n_partitions] 1 register, 2 staged */
    double est_tmax;                 /* ILP objective, ns per iteration */
    int32_t input_device;            /* device holding the caller's input */
    int32_t output_device;           /* device holding the caller's output */
    int64_t iters_per_fragment;
    int32_t ilp_optimal;             /* 1 if the branch-and-bound proved optimality */
    double flops_per_iter_written;   /* algorithmic fp32 flops per iteration as written (FMA = 2) */
    double flops_per_iter_pruned;    /* same after dead-firing / zero-tap elimination (<= written) */
    int64_t intops_per_iter;         /* algorithmic integer ops per iteration (min/max, adds) */
    int32_t replicas;                /* replica groups R; partition_gpu[] is the mapping inside group 0,
                                        group r runs partition p on logical GPU r * (n_gpus / R) + partition_gpu[p] */
    int32_t chain_fission;           /* 1: the plan runs the chain-fissioned graph (sg_plan_opts.chain_groups);
                                        n_nodes and every per-node array describe that graph */
} sg_plan_info_t;

/* ---- graph construction (the top-level stream is an implicit pipeline) ---- */
sg_status sg_graph_create(sg_dtype dtype, sg_graph** out);
void sg_graph_destroy(sg_graph* g);

/* Append a filter to the currently open pipeline.  Rates are derived from kind
 * and parameters; parameters are validated and copied.  *elem_id (optional)
 * receives the element's index in construction order. */
sg_status sg_add_filter(sg_graph* g, const sg_filter_desc* desc, int32_t* elem_id);

/* Append a split-join with n_branches branches to the currently open pipeline.
 * split_w (ROUNDROBIN only) and join_w may be NULL (all weights 1); they are
 * copied.  Each branch is then filled between sg_branch_begin / sg_branch_end,
 * in any order; every branch must be filled (possibly empty = identity). */
sg_status sg_add_splitjoin(sg_graph* g, sg_split_kind kind, const int32_t* split_w,
                           const int32_t* join_w, int32_t n_branches, int32_t* sj_id);
sg_status sg_branch_begin(sg_graph* g, int32_t sj_id, int32_t branch);
sg_status sg_branch_end(sg_graph* g);

/* Append a feedback loop (streams compose by "pipeline ..., split-join ..., and
 * feedback loop"; StreamIt form) to the currently open pipeline.  A joiner
 * RR(join_w[0], join_w[1]) merges the outer input (port 0) with the loop stream's output (port 1);
 * branch 0 is the body, branch 1 the loop stream (fill both with sg_branch_begin / sg_branch_end);
 * a splitter (DUPLICATE, or ROUNDROBIN(split_w[0], split_w[1])) sends port 0 onwards and port 1 into
 * the loop stream.  `enqueue` holds n_enqueue items of the graph dtype (4-byte words), the initial
 * contents of the edge returning to the joiner (the loop delay); it is copied.  Constraints
 * (SG_E_ARG / SG_E_UNSUPPORTED at sg_plan): join_w[1] >= 1, split_w[1] >= 1, no filter with
 * peek > pop inside the loop, no nested feedback loops; the loop must not deadlock (SG_E_RATE).
 * Execution: the loop runs sequentially (it carries state across iterations) as its own partition;
 * everything around it stays data-parallel.  replicas > 1 is rejected for graphs with loops. */
sg_status sg_add_feedbackloop(sg_graph* g, const int32_t join_w[2], sg_split_kind split, const int32_t* split_w,
                              int32_t n_enqueue, const void* enqueue, int32_t* loop_id);

/* ---- planning ---- */
void sg_plan_opts_default(sg_plan_opts* o);

/* Validate, flatten, solve the balance equations (SG_E_RATE), compute the init
 * schedule, partition (Algorithm 1), build the PDG and solve the mapping ILP for
 * n_gpus GPUs, generate one kernel per partition and compile it to sm_100a with
 * NVRTC.  Does not need a GPU; device resources are created on first sg_run.
 * The graph may be destroyed afterwards. */
sg_status sg_plan(const sg_graph* g, int32_t n_gpus, const sg_plan_opts* opts, sg_plan_t** out);

/* Minimal input prefix (items) needed for n_iters iterations; < 0 on error. */
int64_t sg_input_items(const sg_plan_t* p, int64_t n_iters);
/* Output items of n_iters iterations: n_iters * out_per_iter, i.e. the first
 * that many items of the graph's output stream (prework items of the output
 * node included); < 0 on error. */
int64_t sg_output_items(const sg_plan_t* p, int64_t n_iters);

/* Fills *out; pointers inside stay valid until sg_plan_destroy. */
sg_status sg_plan_info(const sg_plan_t* p, sg_plan_info_t* out);

/* Generated CUDA source of partition `part` (NUL-terminated, owned by the plan). */
const char* sg_plan_source(const sg_plan_t* p, int32_t part);

/* ---- execution ---- */
/* Run n_iters steady-state iterations.
 *   input  : device pointer on info.input_device holding >= sg_input_items(n_iters) items
 *   output : device pointer on info.output_device with room for sg_output_items(n_iters) items
 *   stream : cudaStream_t on input_device (NULL = legacy default stream); the call enqueues
 *            work and returns; completion is ordered on `stream`.
 * Inputs are not modified.  n_iters == 0 is a no-op.  Output is bit-identical
 * for every plan of the same graph (Kahn determinism). */
sg_status sg_run(sg_plan_t* p, const void* input, int64_t n_iters, void* output, void* stream);

/* Same, with HOST buffers (host_input: >= sg_input_items items; host_output: >= sg_output_items items;
 * caller-owned; pinned memory makes the copies asynchronous): copies in, runs, copies out, synchronises
 * before returning.  A single-partition plan without feedback loops pipelines 8 chunks of iterations
 * over three streams (host->device copy of chunk c+1, kernel on chunk c, device->host copy of chunk
 * c-1; SG_HOST_CHUNKS overrides the count); other plans copy in, run, copy out.  Same output as sg_run. */
sg_status sg_run_host(sg_plan_t* p, const void* host_input, int64_t n_iters, void* host_output);

/* Measured side of the PEE validation (Fig. 4.1: estimated vs
 * measured partition time).  Runs every partition's kernel ALONE over iterations
 * [0, n_iters), `reps` times after one warm-up launch, on zero-filled scratch
 * boundary windows (the size sg_run's rings hold for one fragment of n_iters), and
 * writes ns per iteration to ns_per_iter[0 .. n_partitions).  Synchronous;
 * allocates and frees its scratch.  SG_E_ARG for n_iters <= 0, reps <= 0 or NULL;
 * SG_E_CUDA without a device (no CPU fallback).  Compare with
 * sg_plan_info_t.partition_time (the PEE estimate, ns per iteration). */
sg_status sg_profile_partitions(sg_plan_t* p, int64_t n_iters, int32_t reps, double* ns_per_iter);

/* Number of kernel launches the last sg_run enqueued (all devices). */
int64_t sg_last_launch_count(const sg_plan_t* p);

void sg_plan_destroy(sg_plan_t* p);

/* Thread-local description of the last error on this thread ("" if none). */
const char* sg_last_error(void);

/* Library version string. */
const char* sg_version(void);

/* ---- one process per GPU (PAPER.md:552-567 with NCCL point-to-point over NVLink) ----
 * Every rank builds the same plan (same graph, n_gpus = world size), rank 0 creates a
 * unique id with sg_comm_unique_id and broadcasts it (e.g. torch.distributed), every
 * rank calls sg_comm_init, then sg_run_rank.  A rank runs only the partitions mapped
 * to it, fragment by fragment; boundary streams travel with ncclSend/ncclRecv on a
 * library-owned stream.  `input` must be given (device pointer on `device`) on the
 * rank whose partition consumes the graph input (sg_plan_info.input_device is that
 * rank), `output` on the rank producing the output; other ranks may pass NULL.  The
 * call enqueues and returns; completion is ordered on `stream`. */
sg_status sg_comm_unique_id(uint8_t id[128]);
sg_status sg_comm_init(sg_plan_t* p, int32_t nranks, int32_t rank, const uint8_t id[128], int32_t device);
sg_status sg_run_rank(sg_plan_t* p, const void* input, int64_t n_iters, void* output, void* stream);

/* The host-side schedule sg_run_rank issues on `rank` (for tests and tracing):
 * op = SG_OP_LAUNCH (partition `part` over iterations [k_begin, k_end)),
 * SG_OP_SEND / SG_OP_RECV (cut edge `edge`, `items` 4-byte items, to/from `peer`).
 * Fills up to `cap` ops; returns the total count (< 0 on error). */
enum { SG_OP_LAUNCH = 0, SG_OP_SEND = 1, SG_OP_RECV = 2 };
typedef struct {
    int32_t op, part, edge, peer;
    int64_t fragment, k_begin, k_end, items;
} sg_rank_op;
int64_t sg_rank_schedule(const sg_plan_t* p, int32_t rank, int64_t n_iters, sg_rank_op* ops, int64_t cap);

/* ---- planner building blocks (PAPER.md sections 3.2-3.3), for tests and tools ----
 * Topology kinds: 0 = NVSwitch star of n_gpus GPUs (uplink k and downlink k per GPU,
 * L = 2G), 1 = the 4-GPU PCIe tree of Fig. 3.3 (n_gpus must be 4). */
int32_t sg_topology_links(int32_t kind, int32_t n_gpus); /* L, or < 0 on error */
/* dtlist as a dense [L][G][G] 0/1 array:
 * dtlist[l*G*G + i*G + j] = 1 iff traffic GPU i -> GPU j loads link l.  Caller-owned. */
sg_status sg_topology_dtlist(int32_t kind, int32_t n_gpus, uint8_t* dtlist);
/* The mapping ILP of Eq. III.1-III.7 on P partitions with
 * times T[P] and PDG edges (e_src, e_dst, e_bytes)[n_e]: minimise Tmax =
 * max(max_j sum_i n_ij T_i, max_l Lat + D_l / bw).  method 0 = exact branch and
 * bound (time limit in ms; *optimal = 0 if it hit the limit), 1 = brute force
 * over G^P.  assign[P] receives the GPU of each partition. */
sg_status sg_map_ilp(int32_t P, const double* T, int32_t n_e, const int32_t* e_src, const int32_t* e_dst,
                     const double* e_bytes, int32_t topo_kind, int32_t n_gpus, double lat, double bw,
                     int32_t time_limit_ms, int32_t method, int32_t* assign, double* tmax, int32_t* optimal);
/* The paper's kernel model, Eq. III.8-III.12: returns T = Texec / W with
 * Tcomp = sum_i t_i / min(f_i, S), Tdt = C1 D / F, Tdb = C2 D / (F + W S),
 * Texec = max(Tcomp, Tdt) + Tdb.  Outputs may be NULL. */
double sg_paper_model(int32_t n, const double* t, const double* f, int32_t S, int32_t W, int32_t F, double D,
                      double C1, double C2, double* tcomp, double* tdt, double* tdb);
/* PDG of a plan: fills up to `cap` edges (partition src, dst,
 * bytes per iteration); returns the number of edges. */
int32_t sg_plan_pdg(const sg_plan_t* p, int32_t cap, int32_t* src, int32_t* dst, double* bytes);

/* PEE inputs of partition `part` (the estimate sees the code generator's own
 * optimisations), per steady-state iteration, written to out[0 .. min(cap, 16)):
 *   0 kernel mode (1 register, 2 staged, 4 feedback loop; bitslice counts as 1), 1 executed fp32 flops
 *   (after view resolution, dead-firing elimination, zero-tap pruning and CSE), 2 integer ops, 3 fp64 ops,
 *   4 items read by live firings, 5 items written, 6 live firings, 7 boundary input bytes, 8 boundary
 *   output bytes, 9 compute levels, 10 halo firings per tile, 11 loop firings, 12 CSE duplicate nodes,
 *   13 frame FIRs present (0/1), 14 bitslice mode (0/1), 15 the plan's estimate T(p) (ns; sg_plan_info's
 *   partition_time), 16 boundary input edges, 17 boundary output edges, 18 items of one iteration at the
 *   boundary (register mode: one thread's row); from the generated kernel (-1 for plan_only plans):
 *   19 staged fused path taken (0/1), 20 iterations per tile, 21 threads per CTA, 22 dynamic shared memory
 *   bytes, 23 CUDA source bytes, 24 register-mode variant (0 TMA / synchronous rows, 1 in-place components,
 *   2 demand-ordered wide rows); 25 dependence components of one iteration (register-eligible partitions);
 *   26 the plan-time expectation of 19 (staged: views only (gather) or at most 8 boundary input streams),
 *   27 the generated kernel's mode (1 register/bitslice, 2 staged, 4 feedback loop, 5 gather), 28 the
 *   fused kernel's frame-FIR parallel efficiency (ideal FFMA issue / the code generator's simulated issue
 *   of its sliding-window levels; 1 without frame FIRs).
 * Returns the number of values written, or -1 (NULL plan / bad partition). */
int32_t sg_pee_features(const sg_plan_t* p, int32_t part, double* out, int32_t cap);

/* Benchmark hygiene: evict L2 by overwriting `bytes` of device scratch memory
 * (> L2 size) and reading it back (dirty lines written back before the next
 * kernel), with nvcc-compiled sm_100a kernels enqueued on `stream`. */
sg_status sg_flush_l2(void* scratch, int64_t bytes, void* stream);

#ifdef __cplusplus
}
#endif
#endif /* SG_H_ */
