// sg_codegen.cpp -- one CUDA kernel per partition ("one partition corresponds
// to one kernel"; code generator PAPER.md:274-277).
//
// Two emitters share one static view resolver:
//
//  * View resolution.  Splitters, joiners and the pure data-movement filters
//    (IDENTITY, DELAY, DECIMATE, EXPAND, FFT_REORDER) never execute: a read of
//    position p on their output is rewritten into a read of their input at a
//    compile-time-resolved position (or a constant zero).  This is the paper's
//    future-work "elimination of splitters and joiners ... re-adjust the index
//    of input data of the follow-up filter" (Figs. 5.1/5.2),
//    generalised to every filter that only rearranges data.  Positions are kept
//    as affine forms of the runtime loop variables; a map whose divisor does
//    not divide every coefficient falls back to a generated runtime reader.
//
//  * Register mode (thread per iteration).  When no node of the partition
//    needs items of a neighbouring iteration (halo 0, peek == pop, aligned init
//    offsets), each thread runs one whole steady-state iteration with every
//    FIFO item an SSA register: the static schedule is flattened by symbolic
//    execution; inputs are loaded lazily from a padded shared-memory row,
//    outputs stored eagerly.  (BitonicSort, FFT.)
//
//  * Staged mode (tile of W iterations per CTA, the paper's one-kernel-per-
//    partition model with FIFOs in shared memory).  Compute
//    filters are grouped into dependence levels; all firings of one level run
//    in parallel across the CTA, one barrier per level; buffers are placed by
//    liveness (the shared-memory footprint of Fig. 3.2).
//    Peek windows that reach into the previous tile are recomputed (halo), so
//    tiles, fragments and GPUs never share state.  FIRs are register-blocked.
//    (FMRadio, FilterBank, BeamFormer, any graph.)
#include "sg_codegen.h"

#include <algorithm>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <cctype>
#include <functional>
#include <map>
#include <numeric>
#include <set>
#include <tuple>
#include <sstream>

namespace sg {

const char* kDeviceHeader =
#include "sg_device_embed.inc"
    ;

static int64_t fdiv(int64_t a, int64_t b) {
    int64_t q = a / b, r = a % b;
    return (r != 0 && ((r < 0) != (b < 0))) ? q - 1 : q;
}
static int64_t fmodp(int64_t a, int64_t b) { return a - fdiv(a, b) * b; }

bool is_view_kind(int k) {
    return k == SG_K_IDENTITY || k == SG_K_DELAY || k == SG_K_DECIMATE || k == SG_K_EXPAND || k == SG_K_FFT_REORDER ||
           k == SG_K_PERMUTE;
}
static bool is_view_node(const Node& n) {
    return n.type == N_FILTER ? is_view_kind(n.kind) : n.type != N_LOOP;
}

void node_work(const Flat& f, int v, int64_t& flops, int64_t& intops, int64_t& dfma) {
    const Node& n = f.nodes[v];
    flops = intops = dfma = 0;
    if (n.type == N_LOOP) {  // the loop graph's work per loop firing, times the loop's firings
        const Flat& sf = *n.loop->sub;
        for (int u = 0; u < (int)sf.nodes.size(); u++) {
            int64_t a, b, c;
            node_work(sf, u, a, b, c);
            flops += a * n.rep;
            intops += b * n.rep;
            dfma += c * n.rep;
        }
        return;
    }
    if (n.type != N_FILTER) return;
    int64_t per = 0;
    switch (n.kind) {
    case SG_K_FIR: per = 2LL * n.iv[0]; break;
    case SG_K_COMBINE_DFT: per = 10LL * (n.iv[0] / 2); break;
    case SG_K_FM_DEMOD: per = 1; dfma = n.rep; break;
    case SG_K_SUBTRACT: case SG_K_AMPLIFY: per = 1; break;
    case SG_K_ADD: if (f.dtype == SG_F32) per = n.iv[0]; else intops = n.rep * n.iv[0]; break;
    case SG_K_BEAM_FIR: per = 8LL * n.iv[0] * (n.iv[2] / n.iv[1]); break;
    case SG_K_BEAMFORM: per = 8LL * n.iv[0]; break;
    case SG_K_MAGNITUDE: per = 3; break;
    case SG_K_MULTIPLY: per = 1; break;
    case SG_K_COMPARE_EXCHANGE: intops = 2 * n.rep; break;
    // DES bit kinds, counted as written: one op per XORed bit, one per table lookup, one per bit moved
    case SG_K_XOR: case SG_K_XOR_CONST: intops = (int64_t)n.iv[0] * n.rep; break;
    case SG_K_SBOX: intops = n.rep; break;
    case SG_K_INTO_BITS: case SG_K_BITS_TO_INT: intops = 32 * n.rep; break;
    default: break;
    }
    flops = per * n.rep;
}

// ------------------------------------------------------------ affine forms
struct Lin {
    std::vector<std::pair<std::string, int64_t>> t;
    int64_t c = 0;
    static Lin k(int64_t c) { Lin l; l.c = c; return l; }
    static Lin v(const std::string& name, int64_t a, int64_t c = 0) { Lin l; l.t.push_back({name, a}); l.c = c; return l; }
    bool divisible(int64_t m) const {
        for (auto& p : t) if (p.second % m) return false;
        return true;
    }
    Lin divf(int64_t m) const {
        Lin r;
        for (auto& p : t) if (p.second / m) r.t.push_back({p.first, p.second / m});
        r.c = fdiv(c, m);
        return r;
    }
    int64_t modc(int64_t m) const { return fmodp(c, m); }
    Lin scaled(int64_t s) const {
        Lin r;
        for (auto& p : t) if (p.second * s != 0) r.t.push_back({p.first, p.second * s});
        r.c = c * s;
        return r;
    }
    Lin plus(int64_t d) const { Lin r = *this; r.c += d; return r; }
    bool is_const() const { return t.empty(); }
    int64_t coef(const std::string& name) const {
        for (auto& p : t) if (p.first == name) return p.second;
        return 0;
    }
    std::string vars() const {  // "a*x + b*y" without constant, or ""
        std::string s;
        for (auto& p : t) {
            if (!s.empty()) s += " + ";
            if (p.second == 1) s += p.first;
            else s += "(" + std::to_string(p.second) + ")*" + p.first;
        }
        return s;
    }
    std::string str() const {
        std::string s = vars();
        if (s.empty()) return std::to_string(c);
        if (c) s += " + (" + std::to_string(c) + ")";
        return "(" + s + ")";
    }
};

struct Ref {
    enum K { PHYS, ZERO, RUNTIME } k = PHYS;
    int edge = -1;
    Lin pos;
};

static std::string hexf(float x) {
    if (!std::isfinite(x)) throw Error(SG_E_ARG, "non-finite filter parameter");
    char b[64];
    if (x == 0.0f) return std::signbit(x) ? "(-0.0f)" : "0.0f";
    std::snprintf(b, sizeof b, "%af", (double)x);
    return std::string("(") + b + ")";
}

void partition_boundary(const Flat& f, const std::vector<int>& nodes, std::vector<int>& ins, std::vector<int>& outs) {
    std::vector<char> in(f.nodes.size(), 0);
    for (int v : nodes) in[v] = 1;
    ins.clear();
    outs.clear();
    for (int e = 0; e < (int)f.edges.size(); e++) {
        const Edge& ed = f.edges[e];
        bool s_in = ed.src >= 0 && in[ed.src], d_in = ed.dst >= 0 && in[ed.dst];
        if (d_in && !s_in) ins.push_back(e);
        if (s_in && !d_in) outs.push_back(e);
    }
}

void edge_window(const Flat& f, int e, int64_t& lo, int64_t& extra) {
    const Edge& ed = f.edges[e];
    if (ed.dst < 0) {  // graph output: iteration k owns positions [k*P, (k+1)*P)
        lo = ed.pre + f.nodes[ed.src].ninit * ed.push;
        extra = 0;
        return;
    }
    const Node& v = f.nodes[ed.dst];
    lo = (v.ninit - v.halo) * ed.pop;
    extra = v.halo * ed.pop + ed.peek - ed.pop;
}

// ---------------------------------------------------------------- resolver
class Resolver {
public:
    Resolver(const Flat& f, const std::vector<int>& nodes) : f_(f), inpart_(f.nodes.size(), 0) {
        for (int v : nodes) inpart_[v] = 1;
    }
    bool phys(int e) const {
        const Edge& ed = f_.edges[e];
        if (ed.src < 0 || !inpart_[ed.src]) return true;  // boundary input
        return !is_view_node(f_.nodes[ed.src]);
    }
    Ref resolve(int e, Lin pos) const {
        for (int guard = 0; guard < 100000; guard++) {
            if (phys(e)) return {Ref::PHYS, e, pos};
            const Edge& ed = f_.edges[e];
            const Node& u = f_.nodes[ed.src];
            switch (u.type) {
            case N_SPLIT_DUP: e = u.in[0]; continue;
            case N_SPLIT_RR: {
                int b = ed.sport;
                int64_t w = u.w[b], P = 0;
                for (int i = 0; i < b; i++) P += u.w[i];
                if (!pos.divisible(w)) return {Ref::RUNTIME, e, pos};
                Lin q = pos.divf(w);
                int64_t r = pos.modc(w);
                pos = q.scaled(u.wsum).plus(P + r);
                e = u.in[0];
                continue;
            }
            case N_JOIN: {
                int64_t S = u.wsum;
                if (!pos.divisible(S)) return {Ref::RUNTIME, e, pos};
                Lin q = pos.divf(S);
                int64_t o = pos.modc(S), P = 0;
                int b = 0;
                while (o >= P + u.w[b]) { P += u.w[b]; b++; }
                pos = q.scaled(u.w[b]).plus(o - P);
                e = u.in[b];
                continue;
            }
            case N_FILTER:
                switch (u.kind) {
                case SG_K_IDENTITY: e = u.in[0]; continue;
                case SG_K_DELAY: pos = pos.plus(-(int64_t)u.iv[0]); e = u.in[0]; continue;
                case SG_K_DECIMATE: pos = pos.scaled(u.iv[0]); e = u.in[0]; continue;
                case SG_K_EXPAND: {
                    int64_t M = u.iv[0];
                    if (!pos.divisible(M)) return {Ref::RUNTIME, e, pos};
                    if (pos.modc(M) != 0) return {Ref::ZERO, -1, Lin()};
                    pos = pos.divf(M);
                    e = u.in[0];
                    continue;
                }
                case SG_K_PERMUTE: {
                    const int64_t n = u.iv[0], m = (int64_t)u.iv.size() - 1;
                    if (!pos.divisible(m)) return {Ref::RUNTIME, e, pos};
                    Lin q = pos.divf(m);
                    pos = q.scaled(n).plus(u.iv[1 + pos.modc(m)]);
                    e = u.in[0];
                    continue;
                }
                case SG_K_FFT_REORDER: {
                    int64_t n = u.iv[0], F = 2 * n;
                    if (!pos.divisible(F)) return {Ref::RUNTIME, e, pos};
                    Lin q = pos.divf(F);
                    int64_t o = pos.modc(F), m = o / 2, r = o % 2;
                    int64_t sc = m < n / 2 ? 2 * m : 2 * (m - n / 2) + 1;
                    pos = q.scaled(F).plus(2 * sc + r);
                    e = u.in[0];
                    continue;
                }
                default: break;
                }
                break;
            }
            throw Error(SG_E_UNSUPPORTED, "internal: unresolvable view");
        }
        throw Error(SG_E_UNSUPPORTED, "internal: view chain too long");
    }
    // Physical edges reachable backwards from e through in-partition views.
    void sources(int e, std::set<int>& out) const {
        if (phys(e)) { out.insert(e); return; }
        const Node& u = f_.nodes[f_.edges[e].src];
        for (int i : u.in) sources(i, out);
    }

private:
    const Flat& f_;
    std::vector<char> inpart_;
};

bool register_mode_eligible(const Flat& f, const std::vector<int>& nodes, std::string* why) {
    auto fail = [&](const std::string& s) { if (why) *why = s; return false; };
    std::vector<int> ins, outs;
    partition_boundary(f, nodes, ins, outs);
    if (ins.size() != 1 || outs.size() != 1) return fail("needs exactly one boundary input and output");
    std::vector<char> in(f.nodes.size(), 0);
    for (int v : nodes) in[v] = 1;
    int64_t live = 0;
    for (int v : nodes) {
        const Node& n = f.nodes[v];
        if (n.type == N_LOOP) return fail("feedback loop");
        if (n.halo != 0) return fail("node " + std::to_string(v) + " has a halo");
        if (n.type == N_FILTER && n.kind == SG_K_BEAM_FIR) return fail("frame FIR");
        if (n.type == N_FILTER && n.prework) return fail("prework");
        if (n.type == N_FILTER && !is_view_kind(n.kind)) live = std::max(live, n.peek + n.push);
        for (int e : n.in) {
            const Edge& ed = f.edges[e];
            if (ed.peek != ed.pop) return fail("peeking edge");
            if (ed.src >= 0 && in[ed.src]) {
                const Node& u = f.nodes[ed.src];
                if (n.ninit * ed.pop != ed.pre + u.ninit * ed.push) return fail("misaligned init offsets");
            }
        }
    }
    const Edge& eo = f.edges[outs[0]];
    if (eo.pre) return fail("output prework");
    if (eo.dst >= 0) {
        int64_t lo, ex;
        edge_window(f, outs[0], lo, ex);
        if (ex != 0 || lo != eo.pre + f.nodes[eo.src].ninit * eo.push) return fail("output window misaligned");
    }
    const Edge& ei = f.edges[ins[0]];
    if (ei.per_iter > 512 || eo.per_iter > 256 || ei.per_iter + eo.per_iter > 768 || live > 512)
        return fail("iteration too large for registers");
    return true;
}

// ---------------------------------------------------------------- common
class GenBase {
public:
    GenBase(const Flat& f, const std::vector<int>& nodes, int part)
        : f_(f), nodes_(nodes), part_(part), R_(f, nodes) {
        T_ = f.dtype == SG_F32 ? "float" : "int";
        partition_boundary(f, nodes, ins_, outs_);
    }

protected:
    const Flat& f_;
    std::vector<int> nodes_;
    int part_;
    Resolver R_;
    std::string T_;
    std::vector<int> ins_, outs_;
    std::ostringstream consts_;
    std::map<std::vector<float>, std::string> pool_;
    int ctab_n_ = 0;
    int ipool_n_ = 0;

    std::string const_array(const std::vector<float>& v) {
        auto it = pool_.find(v);
        if (it != pool_.end()) return it->second;
        std::string name = "SG_C" + std::to_string(pool_.size());
        consts_ << "__constant__ float " << name << "[" << std::max<size_t>(1, v.size()) << "] = {";
        for (size_t i = 0; i < v.size(); i++) consts_ << (i ? "," : "") << (i % 8 == 0 ? "\n  " : "") << hexf(v[i]);
        if (v.empty()) consts_ << "0.0f";
        consts_ << "};\n";
        pool_[v] = name;
        return name;
    }
    int64_t pool_len(const std::string& name) const {
        for (auto& kv : pool_) if (kv.second == name) return (int64_t)std::max<size_t>(1, kv.first.size());
        return -1;
    }
    // every pool array of length L as row n of one table (row n = SG_C<n>; rows of other lengths zero)
    std::map<int64_t, std::pair<size_t, std::string>> ctabs_;  // length -> (pool size when emitted, name)
    std::string coef_table(int64_t L) {
        auto it = ctabs_.find(L);
        if (it != ctabs_.end() && it->second.first == pool_.size()) return it->second.second;
        std::vector<const std::vector<float>*> rows(pool_.size(), nullptr);
        for (auto& kv : pool_) rows[std::atoi(kv.second.c_str() + 4)] = &kv.first;
        const std::string name = "SG_CT" + std::to_string(L) + "_" + std::to_string(ctab_n_++);
        consts_ << "__constant__ float " << name << "[" << rows.size() << "][" << L << "] = {";
        for (size_t r = 0; r < rows.size(); r++) {
            consts_ << (r ? ",\n  {" : "\n  {");
            for (int64_t i = 0; i < L; i++)
                consts_ << (i ? "," : "") << ((rows[r] && (int64_t)rows[r]->size() == L) ? hexf((*rows[r])[i]) : std::string("0.0f"));
            consts_ << "}";
        }
        consts_ << "};\n";
        ctabs_[L] = {pool_.size(), name};
        return name;
    }
    // Twiddles of CombineDFT(j): w_k = (cos(2 pi k / j), -sin(2 pi k / j)), double -> float.
    std::pair<std::string, std::string> twiddles(int j) {
        std::vector<float> wr(j / 2), wi(j / 2);
        for (int k = 0; k < j / 2; k++) {
            double a = 2.0 * M_PI * (double)k / (double)j;
            wr[k] = (float)std::cos(a);
            wi[k] = (float)(-std::sin(a));
        }
        return {const_array(wr), const_array(wi)};
    }
    // Work-function call for one firing of compute filter v: x_ -> y_.
    std::string work_call(int v) {
        const Node& n = f_.nodes[v];
        const std::string& T = T_;
        switch (n.kind) {
        case SG_K_FIR: return "sg_work_fir<" + std::to_string(n.peek) + "," + std::to_string(n.iv[0]) + ">(x_, y_, " +
                              const_array(n.fv) + ");";
        case SG_K_COMPARE_EXCHANGE:
            return "sg_work_compare_exchange<" + T + "," + (n.iv[0] ? "true" : "false") + ">(x_, y_);";
        case SG_K_COMBINE_DFT: {
            auto tw = twiddles(n.iv[0]);
            return "sg_work_combine_dft<" + std::to_string(n.iv[0]) + ">(x_, y_, " + tw.first + ", " + tw.second + ");";
        }
        case SG_K_FM_DEMOD:
            return std::string(std::getenv("SG_FM_F32") ? "sg_work_fm_demod_f32" : "sg_work_fm_demod") + "(x_, y_, " +
                   hexf(n.fv[0]) + ");";
        case SG_K_SUBTRACT: return "sg_work_subtract(x_, y_);";
        case SG_K_AMPLIFY: return "sg_work_amplify(x_, y_, " + hexf(n.fv[0]) + ");";
        case SG_K_ADD: return "sg_work_add<" + std::to_string(n.iv[0]) + ">(x_, y_);";
        case SG_K_BEAMFORM: {
            std::vector<float> wr(n.fv.begin(), n.fv.begin() + n.iv[0]), wi(n.fv.begin() + n.iv[0], n.fv.end());
            return "sg_work_beamform<" + std::to_string(n.iv[0]) + ">(x_, y_, " + const_array(wr) + ", " +
                   const_array(wi) + ");";
        }
        case SG_K_MAGNITUDE: return "sg_work_magnitude(x_, y_);";
        case SG_K_MULTIPLY: return "sg_work_multiply(x_, y_);";
        case SG_K_XOR: return "sg_work_xor<" + std::to_string(n.iv[0]) + ">(x_, y_);";
        case SG_K_XOR_CONST: {  // key bits folded into the code (x ^ 0 = x)
            std::string c;
            for (int i = 0; i < n.iv[0]; i++)
                c += "y_[" + std::to_string(i) + "] = x_[" + std::to_string(i) + "]" +
                     (n.iv[1 + i] ? " ^ " + std::to_string(n.iv[1 + i]) : std::string()) + "; ";
            return c;
        }
        case SG_K_SBOX: {  // one 64-bit truth-table mask per output bit: bit i of t[idx] = (M_i >> idx) & 1
            unsigned long long M[4] = {0, 0, 0, 0};
            for (int k = 0; k < 64; k++)
                for (int i = 0; i < 4; i++)
                    if ((n.iv[k] >> (3 - i)) & 1) M[i] |= 1ull << k;
            char b[160];
            std::snprintf(b, sizeof b, "sg_work_sbox(x_, y_, 0x%016llxull, 0x%016llxull, 0x%016llxull, 0x%016llxull);",
                          M[0], M[1], M[2], M[3]);
            return b;
        }
        case SG_K_INTO_BITS: return "sg_work_into_bits(x_, y_);";
        case SG_K_BITS_TO_INT: return "sg_work_bits_to_int(x_, y_);";
        default: break;
        }
        throw Error(SG_E_UNSUPPORTED, std::string("no work function for ") + kind_name(n.kind));
    }
    std::string header(const char* mode) {
        std::ostringstream h;
        h << "// generated by sg_codegen.cpp: partition " << part_ << " (" << mode << " mode), " << nodes_.size()
          << " nodes\n#include \"sg_device.cuh\"\n";
        return h.str();
    }
    void fill_io(KernelInfo& ki) {
        ki.in_edges = ins_;
        ki.out_edges = outs_;
        for (int e : ins_) {
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            ki.in_lo.push_back(lo);
            ki.in_extra.push_back(ex);
        }
        for (int e : outs_) {
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            ki.out_lo.push_back(lo);
            ki.out_extra.push_back(ex);
        }
        for (int v : nodes_) {
            int64_t a, b, c;
            node_work(f_, v, a, b, c);
            ki.flops_per_iter += a;
            ki.intops_per_iter += b;
            ki.dfma_per_iter += c;
        }
    }
    // kernel argument block: all 8-byte words
    //   in ptr[NI], in_base[NI], in_limit[NI], out ptr[NO], out_base[NO], k_begin, k_end
    // extra = 1 (staged kernels): one more word, the runtime tile size SG_WR (<= the compiled tile)
    // The word is always passed; the kernel reads it only when generated with SG_RT_TILE=1, otherwise
    // SG_WR is the compile-time tile `wt` (constant strides measured ~2.5% faster on FMRadio).
    std::string args_struct(int extra = 0, int wt = 0) {
        size_t ni = ins_.size(), no = outs_.size();
        std::ostringstream s;
        s << "struct SgArgs { long long v[" << (3 * ni + 2 * no + 2 + extra) << "]; };\n";
        if (extra && std::getenv("SG_RT_TILE")) s << "#define SG_WR ((int)a.v[" << 3 * ni + 2 * no + 2 << "])\n";
        else if (extra) s << "#define SG_WR " << wt << "\n";
        s << "#define SG_IN(i) (reinterpret_cast<const " << T_ << "*>(a.v[(i)]))\n";
        s << "#define SG_IN_BASE(i) (a.v[" << ni << " + (i)])\n";
        s << "#define SG_IN_LIMIT(i) (a.v[" << 2 * ni << " + (i)])\n";
        s << "#define SG_OUT(i) (reinterpret_cast<" << T_ << "*>(a.v[" << 3 * ni << " + (i)]))\n";
        s << "#define SG_OUT_BASE(i) (a.v[" << 3 * ni + no << " + (i)])\n";
        s << "#define SG_K_BEGIN (a.v[" << 3 * ni + 2 * no << "])\n";
        s << "#define SG_K_END (a.v[" << 3 * ni + 2 * no + 1 << "])\n";
        return s.str();
    }
};

// ------------------------------------------------------------ register mode
class RegGen : public GenBase {
public:
    using GenBase::GenBase;

    KernelInfo run(const CodegenOpts& opt) {
        KernelInfo ki;
        ki.mode = 1;
        ki.name = "sg_part" + std::to_string(part_);
        ki.name_sync = ki.name + "_sync";
        fill_io(ki);
        ein_ = ins_[0];
        eout_ = outs_[0];
        const Edge& ei = f_.edges[ein_];
        const Edge& eo = f_.edges[eout_];
        PIN_ = ei.per_iter;
        POUT_ = eo.per_iter;
        off_in_ = ki.in_lo[0];
        off_out_ = ki.out_lo[0];
        vin_ = PIN_ % 4 == 0;
        vout_ = POUT_ % 4 == 0;
        RIN_S_ = row_stride(PIN_);
        ROUT_S_ = row_stride(POUT_);
        body_.str("");
        // wide rows with one dependence component (2-D DCT): node-order emission keeps every
        // intermediate of the iteration live at once (spills); emit output groups on demand instead
        static const int64_t dmin = std::getenv("SG_DEMAND_MIN") ? std::atoll(std::getenv("SG_DEMAND_MIN")) : 384;
        demand_ = !std::getenv("SG_NO_DEMAND") && PIN_ + POUT_ >= dmin && n_components() == 1;
        if (demand_) emit_body_demand();
        else emit_body();
        const std::string VT4 = T_ == "float" ? "float4" : "int4";
        std::ostringstream src;
        src << header(demand_ ? "register, demand-ordered" : "register") << consts_.str() << args_struct();
        // input re-reads: plain loads (the compiler may keep a run's inputs in registers; with rolled output
        // groups the live ranges stay short) -- measured with rolled groups: DCT 16x16 0.311 -> 0.233 ms, MatMul
        // 16 0.628 -> 0.396 ms per 2^18 iterations against volatile re-reads; SG_DEMAND_VOL=1 forces volatile
        const bool dvol = std::getenv("SG_DEMAND_VOL") ? std::atoi(std::getenv("SG_DEMAND_VOL")) != 0 : false;
        if (demand_)
            src << (!dvol ? "#define SG_LDV(r) (SG_LD1(r))\n"
                          : "#define SG_LDV(r) (*(volatile const " + T_ + "*)&SG_LD1(r))\n");
        if (demand_) {
            ki.reg_variant = 2;
            return run_demand(ki, src, VT4, opt);
        }
        // ---------------- variant 1: synchronous tiles (any alignment / row size)
        int bytes_per_thread = (int)((RIN_S_ + ROUT_S_) * 4);
        int NT = opt.threads;
        if (NT <= 0) {
            NT = 256;
            while (NT > 32 && (size_t)NT * bytes_per_thread > 72 * 1024) NT /= 2;
        }
        ki.threads_sync = NT;
        ki.tile_sync = NT;
        ki.smem_sync = (size_t)NT * bytes_per_thread;
        int minb = std::max(1, std::min(8, (int)((200 * 1024) / std::max<size_t>(1, ki.smem_sync))));
        if (bytes_per_thread * NT > 200 * 1024) minb = 1;
        src << "#define SG_LD4(g) (reinterpret_cast<const " << VT4 << "*>(xr)[g])\n"
            << "#define SG_LD1(r) (xr[r])\n"
            << "#define SG_ST4(g, v) (reinterpret_cast<" << VT4 << "*>(yr)[g] = (v))\n"
            << "#define SG_ST1(g, v) (yr[g] = (v))\n";
        src << "extern \"C\" __global__ void __launch_bounds__(" << NT << ", " << minb << ") " << ki.name_sync
            << "(const SgArgs a) {\n"
            << "  constexpr int NT = " << NT << ";\n"
            << "  extern __shared__ __align__(16) unsigned char sg_smem[];\n"
            << "  " << T_ << "* s_in = reinterpret_cast<" << T_ << "*>(sg_smem);\n"
            << "  " << T_ << "* s_out = s_in + NT * " << RIN_S_ << ";\n"
            << "  const " << T_ << "* gin = SG_IN(0);\n"
            << "  " << T_ << "* gout = SG_OUT(0);\n"
            << "  for (long long t0 = SG_K_BEGIN + (long long)blockIdx.x * NT; t0 < SG_K_END; t0 += (long long)gridDim.x * NT) {\n"
            << "    const int nt = (int)min((long long)NT, SG_K_END - t0);\n"
            << "    const " << T_ << "* gsrc = gin + (t0 * " << PIN_ << "LL + (" << off_in_ << "LL) - SG_IN_BASE(0));\n"
            << (vin_ ? std::string("    if ((reinterpret_cast<unsigned long long>(gsrc) & 15ull) == 0)\n      sg_rows_g2s_v4<") +
                           T_ + ", " + std::to_string(PIN_) + ", " + std::to_string(RIN_S_) + ", NT>(gsrc, s_in, nt);\n    else\n"
                     : std::string())
            << "      sg_rows_g2s_v1<" << T_ << ", " << PIN_ << ", " << RIN_S_ << ", NT>(gsrc, s_in, nt);\n"
            << "    __syncthreads();\n"
            << "    if (threadIdx.x < nt) {\n"
            << "      const " << T_ << "* xr = s_in + threadIdx.x * " << RIN_S_ << ";\n"
            << "      " << T_ << "* yr = s_out + threadIdx.x * " << ROUT_S_ << ";\n"
            << body_.str()
            << "    }\n"
            << "    __syncthreads();\n"
            << "    " << T_ << "* gdst = gout + (t0 * " << POUT_ << "LL + (" << off_out_ << "LL) - SG_OUT_BASE(0));\n"
            << (vout_ ? std::string("    if ((reinterpret_cast<unsigned long long>(gdst) & 15ull) == 0)\n      sg_rows_s2g_v4<") +
                            T_ + ", " + std::to_string(POUT_) + ", " + std::to_string(ROUT_S_) + ", NT>(s_out, gdst, nt);\n    else\n"
                      : std::string())
            << "      sg_rows_s2g_v1<" << T_ << ", " << POUT_ << ", " << ROUT_S_ << ", NT>(s_out, gdst, nt);\n"
            << "  }\n}\n"
            << "#undef SG_LD4\n#undef SG_LD1\n#undef SG_ST4\n#undef SG_ST1\n";
        // ---------------- variant 2: warp-specialised TMA pipeline (PAPER.md:220-228's
        // data-transfer threads become one producer warp driving the TMA engine)
        // layout 1: 128-byte rows, 2-D tensor map with 128B swizzle (one TMA per tile / slab)
        // layout 2: 16-byte-multiple rows, one bulk copy per row into padded shared rows
        ki.tma_in = PIN_ * 4 == 128 ? 1 : (PIN_ % 4 == 0 ? 2 : 0);
        ki.tma_out = POUT_ * 4 == 128 ? 1 : (POUT_ % 4 == 0 ? 2 : 0);
        ki.pin = PIN_;
        ki.pout = POUT_;
        ki.off_in = off_in_;
        ki.off_out = off_out_;
        if (opt.mode != -1 && try_inplace(ki, src, VT4)) {
            ki.reg_variant = 1;
            // in-place component kernel generated
        } else if (ki.tma_in && ki.tma_out && opt.mode != -1) {
            auto stage_bytes = [&](int lay, int64_t P, int64_t RS, int rows) -> int64_t {
                int64_t b = lay == 1 ? rows * 128 : rows * RS * 4;
                return (b + 1023) / 1024 * 1024;
            };
            int nt = 0, nsi = 0, nso = 0;
            for (int budget : {110 * 1024, 220 * 1024}) {
                for (int cand : {128, 64, 32}) {
                    if (opt.threads > 0 && cand != opt.threads) continue;
                    for (int si : {4, 3, 2}) {
                        for (int so : {2, 1}) {
                            int64_t tot = si * stage_bytes(ki.tma_in, PIN_, RIN_S_, cand) +
                                          so * stage_bytes(ki.tma_out, POUT_, ROUT_S_, cand) + 1024;
                            if (tot <= budget && !nt) { nt = cand; nsi = si; nso = so; }
                        }
                    }
                }
                if (nt) break;
            }
            if (nt) {
                const int64_t inb = stage_bytes(ki.tma_in, PIN_, RIN_S_, nt);
                const int64_t outb = stage_bytes(ki.tma_out, POUT_, ROUT_S_, nt);
                ki.threads = nt + 32;
                ki.tile = nt;
                ki.smem = (size_t)(nsi * inb + nso * outb + 1024 + 1024);  // + barriers + alignment slack
                ki.has_tma = true;
                const int nwc = nt / 32;
                src << "// ---- TMA pipeline: " << nt << " rows per tile, " << nsi << " input stages, " << nso
                    << " output stages\n";
                if (ki.tma_in == 1)
                    src << "#define SG_LD4(g) (*reinterpret_cast<const " << VT4 << "*>(xb + ((((g) ^ swz)) << 4)))\n"
                        << "#define SG_LD1(r) (reinterpret_cast<const " << T_ << "*>(xb + ((((r) >> 2) ^ swz) << 4))[(r) & 3])\n";
                else
                    src << "#define SG_LD4(g) (*reinterpret_cast<const " << VT4 << "*>(xb + ((g) << 4)))\n"
                        << "#define SG_LD1(r) (reinterpret_cast<const " << T_ << "*>(xb)[r])\n";
                if (ki.tma_out == 1)
                    src << "#define SG_ST4(g, v) (*reinterpret_cast<" << VT4 << "*>(yb + ((((g) ^ swz)) << 4)) = (v))\n"
                        << "#define SG_ST1(g, v) (reinterpret_cast<" << T_ << "*>(yb + ((((g) >> 2) ^ swz) << 4))[(g) & 3] = (v))\n";
                else
                    src << "#define SG_ST4(g, v) (*reinterpret_cast<" << VT4 << "*>(yb + ((g) << 4)) = (v))\n"
                        << "#define SG_ST1(g, v) (reinterpret_cast<" << T_ << "*>(yb)[g] = (v))\n";
                src << "extern \"C\" __global__ void __launch_bounds__(" << nt + 32 << ", 1) " << ki.name
                    << "(const SgArgs a, const __grid_constant__ SgTmap tin, const __grid_constant__ SgTmap tout) {\n"
                    << "  constexpr int NT = " << nt << ", NWC = " << nwc << ", NSI = " << nsi << ", NSO = " << nso << ";\n"
                    << "  constexpr int INB = " << inb << ", OUTB = " << outb << ";\n"
                    << "  extern __shared__ __align__(1024) unsigned char sg_smem_raw[];\n"
                    << "  unsigned char* sg_smem = reinterpret_cast<unsigned char*>((reinterpret_cast<unsigned long long>(sg_smem_raw) + 1023ull) & ~1023ull);\n"
                    << "  unsigned char* in_st = sg_smem;\n"
                    << "  unsigned char* out_st = sg_smem + NSI * INB;\n"
                    << "  unsigned long long* full = reinterpret_cast<unsigned long long*>(out_st + NSO * OUTB);\n"
                    << "  unsigned long long* empty = full + NSI;\n"
                    << "  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;\n"
                    << "  const long long nrows = SG_K_END - SG_K_BEGIN;\n"
                    << "  const long long ntiles = (nrows + NT - 1) / NT;\n"
                    << "  if (threadIdx.x == 0) {\n"
                    << "    for (int s = 0; s < NSI; s++) { sg_mbar_init(&full[s], 1); sg_mbar_init(&empty[s], NWC); }\n"
                    << "    sg_fence_barrier_init();\n"
                    << "  }\n"
                    << "  __syncthreads();\n"
                    << "  if (warp == NWC) {  // ---- producer warp\n";
                if (ki.tma_in == 1) {
                    src << "    if (lane == 0) {\n"
                        << "      sg_prefetch_tmap(&tin);\n"
                        << "      int i = 0;\n"
                        << "      for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, i++) {\n"
                        << "        const int s = i % NSI;\n"
                        << "        sg_mbar_wait(&empty[s], ((i / NSI) & 1) ^ 1);\n"
                        << "        sg_mbar_arrive_expect_tx(&full[s], NT * 128);\n"
                        << "        sg_tma_load_2d(in_st + s * INB, &tin, 0, (int)(t * NT), &full[s]);\n"
                        << "      }\n"
                        << "    }\n";
                } else {
                    src << "    const " << T_ << "* gin = SG_IN(0) + (SG_K_BEGIN * " << PIN_ << "LL + (" << off_in_
                        << "LL) - SG_IN_BASE(0));\n"
                        << "    int i = 0;\n"
                        << "    for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, i++) {\n"
                        << "      const int s = i % NSI;\n"
                        << "      const int nt = (int)min((long long)NT, nrows - t * NT);\n"
                        << "      sg_mbar_wait(&empty[s], ((i / NSI) & 1) ^ 1);\n"
                        << "      if (lane == 0) sg_mbar_arrive_expect_tx(&full[s], (unsigned)(nt * " << PIN_ * 4 << "));\n"
                        << "      __syncwarp();\n"
                        << "      for (int r = lane; r < nt; r += 32)\n"
                        << "        sg_bulk_g2s(in_st + s * INB + r * " << RIN_S_ * 4 << ", gin + (t * NT + r) * " << PIN_
                        << "LL, " << PIN_ * 4 << ", &full[s]);\n"
                        << "    }\n";
                }
                src << "    return;\n"
                    << "  }\n"
                    << "  // ---- consumer warps: one iteration per thread, registers only\n"
                    << "  " << T_ << "* gout = SG_OUT(0) + (SG_K_BEGIN * " << POUT_ << "LL + (" << off_out_
                    << "LL) - SG_OUT_BASE(0));\n"
                    << "  int i = 0;\n"
                    << "  for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, i++) {\n"
                    << "    const int s = i % NSI, so = i % NSO;\n"
                    << "    const int nt = (int)min((long long)NT, nrows - t * NT);\n"
                    << "    sg_mbar_wait(&full[s], (i / NSI) & 1);\n";
                if (ki.tma_out == 1) src << "    if (lane == 0) sg_bulk_wait_read<NSO - 1>();\n";
                else src << "    sg_bulk_wait_read<NSO - 1>();\n";
                src << "    __syncwarp();\n"
                    << "    const int row = threadIdx.x;\n"
                    << "    const int swz = row & 7;\n"
                    << "    const unsigned char* xb = in_st + s * INB + row * "
                    << (ki.tma_in == 1 ? 128 : RIN_S_ * 4) << ";\n"
                    << "    unsigned char* yb = out_st + so * OUTB + row * " << (ki.tma_out == 1 ? 128 : ROUT_S_ * 4) << ";\n"
                    << "    (void)swz;\n"
                    << "    if (row < nt) {\n"
                    << body_.str()
                    << "    }\n"
                    << "    __syncwarp();\n"
                    << "    if (lane == 0) sg_mbar_arrive(&empty[s]);\n"
                    << "    sg_fence_proxy_async();\n"
                    << "    __syncwarp();\n";
                if (ki.tma_out == 1) {
                    src << "    if (lane == 0 && warp * 32 < nt) {\n"
                        << "      sg_tma_store_2d(&tout, 0, (int)(t * NT + warp * 32), out_st + so * OUTB + warp * 32 * 128);\n"
                        << "      sg_bulk_commit();\n"
                        << "    }\n";
                } else {
                    src << "    if (row < nt) {\n"
                        << "      sg_bulk_s2g(gout + (t * NT + row) * " << POUT_ << "LL, yb, " << POUT_ * 4 << ");\n"
                        << "      sg_bulk_commit();\n"
                        << "    }\n";
                }
                src << "  }\n"
                    << "  sg_bulk_wait<0>();\n"
                    << "}\n";
            }
        }
        if (!ki.has_tma) {
            ki.name = ki.name_sync;
            ki.threads = ki.threads_sync;
            ki.tile = ki.tile_sync;
            ki.smem = ki.smem_sync;
        }
        ki.min_blocks = 1;
        ki.source = src.str();
        return ki;
    }

private:
    // ---------------------------------------------------------------------
    // In-place component variant.  Outputs whose dependence cones share no
    // input item form independent components (FFT: its two branches); each
    // component runs on its own warps (warp-uniform), loads its inputs
    // eagerly, computes, writes its outputs back into the same shared-memory
    // row slots (they are read by no other component) and bulk-stores its
    // contiguous output chunk.  One stage buffer serves as input and output.
    typedef std::vector<uint64_t> Bits;
    std::map<std::pair<int, int64_t>, Bits> cone_memo_;
    Bits cone_of(int e, int64_t pos) {
        Bits b((PIN_ + 63) / 64, 0);
        Ref r = R_.resolve(e, Lin::k(pos));
        if (r.k == Ref::ZERO) return b;
        if (r.edge == ein_) {
            int64_t q = r.pos.c - off_in_;
            if (q < 0 || q >= PIN_) throw Error(SG_E_UNSUPPORTED, "internal: cone out of row");
            b[q / 64] |= 1ull << (q % 64);
            return b;
        }
        const Edge& ed = f_.edges[r.edge];
        const Node& u = f_.nodes[ed.src];
        int64_t g = (r.pos.c - ed.pre) / u.push;
        auto key = std::make_pair(ed.src, g);
        auto it = cone_memo_.find(key);
        if (it != cone_memo_.end()) return it->second;
        for (int64_t i = 0; i < u.peek; i++) {
            Bits c = cone_of(u.in[0], g * u.pop + i);
            for (size_t w = 0; w < b.size(); w++) b[w] |= c[w];
        }
        cone_memo_[key] = b;
        return b;
    }
    std::map<std::pair<int, int64_t>, std::vector<std::string>> dmemo_;
    std::string dval(std::ostringstream& o, int e, int64_t pos) {
        Ref r = R_.resolve(e, Lin::k(pos));
        if (r.k == Ref::ZERO) return "(" + T_ + ")0";
        if (r.edge == ein_) {
            int64_t q = r.pos.c - off_in_ - rel_ilo_;
            static const char* comp[4] = {"x", "y", "z", "w"};
            return "iq" + std::to_string(q / 4) + "." + comp[q % 4];
        }
        const Edge& ed = f_.edges[r.edge];
        int u = ed.src;
        const Node& n = f_.nodes[u];
        int64_t q = r.pos.c - ed.pre, g = q / n.push, j = q % n.push;
        auto key = std::make_pair(u, g);
        auto it = dmemo_.find(key);
        if (it != dmemo_.end()) return it->second[j];
        std::vector<std::string> xs(n.peek);
        for (int64_t i = 0; i < n.peek; i++) xs[i] = dval(o, n.in[0], g * n.pop + i);
        std::vector<std::string> ys(n.push);
        o << "      " << T_ << " ";
        for (int64_t jj = 0; jj < n.push; jj++) {
            ys[jj] = "v" + std::to_string(nv_++);
            o << (jj ? ", " : "") << ys[jj];
        }
        o << ";\n      { const " << T_ << " x_[" << n.peek << "] = {";
        for (int64_t i = 0; i < n.peek; i++) o << (i ? ", " : "") << xs[i];
        o << "}; " << T_ << " y_[" << n.push << "]; " << work_call(u);
        for (int64_t jj = 0; jj < n.push; jj++) o << " " << ys[jj] << " = y_[" << jj << "];";
        o << " }\n";
        dmemo_[key] = ys;
        return ys[j];
    }
    // dval with input names relative to a component's input chunk (group index - ilo/4)
    std::string dval_rel(std::ostringstream& o, int e, int64_t pos, int64_t ilo) {
        rel_ilo_ = ilo;
        return dval(o, e, pos);
    }
    int64_t rel_ilo_ = 0;
    // Demand-ordered kernels keep only the input rows in shared memory (re-read many times) and store
    // each output group straight to global memory from registers: half the shared memory per row, so
    // twice the warps per SM of the staged-row variants; no TMA (the rows are consumed out of order).
    KernelInfo run_demand(KernelInfo& ki, std::ostringstream& src, const std::string& VT4, const CodegenOpts& opt) {
        const int bytes_per_row = (int)(RIN_S_ * 4);
        const int K = demand_K_;
        int NT = opt.threads;
        if (NT <= 0) {
            NT = 256;
            while (NT > 32 * K && (size_t)(NT / K) * bytes_per_row > 100 * 1024) NT /= 2;
        }
        if (NT % (32 * K) != 0) throw Error(SG_E_ARG, "threads must be a multiple of 32 x the demand runs");
        const int TR = NT / K;  // iterations (rows) per tile
        // rows stored transposed (item q of row r at q * (TR + 1) + r): the lanes of a warp -- consecutive
        // rows -- read item q from consecutive banks (row-major rows 4 items apart were a 4-way conflict
        // on every one of DCT 16x16's 4 096 input re-reads per block)
        const int ST = TR + 1;
        // double-buffered tiles (cp.async, 4 bytes each into the transposed slots, conflict-free: ST = 1 mod 32):
        // the next tile streams in while this one computes.  Opt-in (SG_DEMAND_DB=1): measured DCT 16x16
        // 0.229 -> 0.292 ms (half the CTAs per SM), MatMul 16 0.393 -> 0.386 ms
        const bool db = std::getenv("SG_DEMAND_DB") && std::atoi(std::getenv("SG_DEMAND_DB")) != 0;
        const size_t smem = (size_t)PIN_ * ST * 4 * (db ? 2 : 1);
        // CTAs per SM the shared memory allows, but never below 128 registers per thread (the demand
        // bodies' live sets: DCT 16x16 at 42 registers spilled 9 KB per thread)
        const int minb = std::max(1, std::min({8, (int)((220 * 1024) / std::max<size_t>(1, smem)), 65536 / (NT * 128)}));
        src << "#define SG_LD1(r) (xr[(r) * " << ST << "])\n"
            << "#define SG_ST4(g, v) do { const " << VT4 << " t_ = (v); if (ga) reinterpret_cast<" << VT4
            << "*>(yg)[g] = t_; else { yg[4 * (g)] = t_.x; yg[4 * (g) + 1] = t_.y; yg[4 * (g) + 2] = t_.z; yg[4 * (g) + 3] = t_.w; } } while (0)\n"
            << "#define SG_ST1(g, v) (yg[g] = (v))\n";
        src << "extern \"C\" __global__ void __launch_bounds__(" << NT << ", " << minb << ") " << ki.name_sync
            << "(const SgArgs a) {\n"
            << "  constexpr int NT = " << NT << ";\n"
            << "  extern __shared__ __align__(16) unsigned char sg_smem[];\n"
            << "  " << T_ << "* s_in = reinterpret_cast<" << T_ << "*>(sg_smem);\n"
            << "  const " << T_ << "* gin = SG_IN(0);\n"
            << "  " << T_ << "* gout = SG_OUT(0);\n"
            << "  constexpr int TR = " << TR << ";  // rows per tile: " << K << " warp(s) per 32 rows, one demand run each\n"
            << "  const int q_ = (threadIdx.x >> 5) % " << K << ";\n"
            << "  const int r_ = (threadIdx.x >> 5) / " << K << " * 32 + (threadIdx.x & 31);\n"
            << "  (void)q_;\n"
            ;
        if (db) {
            const std::string issue = std::string("{ const int ntn = (int)min((long long)TR, SG_K_END - (T)); const ") + T_ +
                                      "* gs = gin + ((T) * " + std::to_string(PIN_) + "LL + (" + std::to_string(off_in_) +
                                      "LL) - SG_IN_BASE(0)); for (int i = threadIdx.x; i < ntn * " + std::to_string(PIN_) +
                                      "; i += NT) { const int row = i / " + std::to_string(PIN_) + ", q = i - row * " +
                                      std::to_string(PIN_) + "; sg_cp_async4((B) + q * " + std::to_string(ST) +
                                      " + row, gs + i, 4u); } }";
            auto at = [&](const std::string& t, const std::string& buf) {
                std::string r = issue;
                for (size_t p = r.find("(T)"); p != std::string::npos; p = r.find("(T)")) r.replace(p, 3, "(" + t + ")");
                for (size_t p = r.find("(B)"); p != std::string::npos; p = r.find("(B)")) r.replace(p, 3, "(" + buf + ")");
                return r;
            };
            src << "  const long long tstep = (long long)gridDim.x * TR;\n"
                << "  int bsel = 0;\n"
                << "  { const long long tf = SG_K_BEGIN + (long long)blockIdx.x * TR; if (tf < SG_K_END) "
                << at("tf", "s_in") << " }\n"
                << "  sg_cp_async_commit();\n"
                << "  for (long long t0 = SG_K_BEGIN + (long long)blockIdx.x * TR; t0 < SG_K_END; t0 += tstep, bsel ^= 1) {\n"
                << "    const int nt = (int)min((long long)TR, SG_K_END - t0);\n"
                << "    { const long long tn = t0 + tstep; if (tn < SG_K_END) "
                << at("tn", "s_in + (bsel ^ 1) * " + std::to_string(PIN_ * ST)) << " }\n"
                << "    sg_cp_async_commit();\n"
                << "    asm volatile(\"cp.async.wait_group 1;\" ::: \"memory\");  // this tile's group has landed\n"
                << "    __syncthreads();\n"
                << "    const " << T_ << "* s_cur = s_in + bsel * " << PIN_ * ST << ";\n";
        } else {
            static const bool cpa = std::getenv("SG_DEMAND_CPASYNC") && std::atoi(std::getenv("SG_DEMAND_CPASYNC")) != 0;
            src << "  for (long long t0 = SG_K_BEGIN + (long long)blockIdx.x * TR; t0 < SG_K_END; t0 += (long long)gridDim.x * TR) {\n"
            << "    const int nt = (int)min((long long)TR, SG_K_END - t0);\n"
            << "    const " << T_ << "* gsrc = gin + (t0 * " << PIN_ << "LL + (" << off_in_ << "LL) - SG_IN_BASE(0));\n";
            if (cpa)  // (opt-in) the tile through cp.async: no register round trip, every load in flight at once
                src << "    for (int i = threadIdx.x; i < nt * " << PIN_ << "; i += NT) {\n"
                    << "      const int row = i / " << PIN_ << ", q = i - row * " << PIN_ << ";\n"
                    << "      sg_cp_async4(s_in + q * " << ST << " + row, gsrc + i, 4u);\n"
                    << "    }\n"
                    << "    sg_cp_async_commit();\n    sg_cp_async_wait_all();\n    if (false)\n";
            src
            << (PIN_ % 4 == 0 ? std::string("    if ((reinterpret_cast<unsigned long long>(gsrc) & 15ull) == 0) {\n") +
                   // eight 16-byte loads in flight per thread before any shared-memory store (the tile load
                   // is the kernel's only global read; one at a time it was latency-bound)
                   "      const int n4 = nt * " + std::to_string(PIN_ / 4) + ";\n" +
                   "      for (int i0 = threadIdx.x; i0 < n4; i0 += 8 * NT) {\n" +
                   "        " + VT4 + " v[8];\n" +
                   "#pragma unroll\n" +
                   "        for (int u = 0; u < 8; u++) if (i0 + u * NT < n4) v[u] = __ldg(reinterpret_cast<const " + VT4 +
                   "*>(gsrc) + i0 + u * NT);\n" +
                   "#pragma unroll\n" +
                   "        for (int u = 0; u < 8; u++) {\n" +
                   "          const int i = i0 + u * NT;\n" +
                   "          if (i >= n4) break;\n" +
                   "          const int row = i / " + std::to_string(PIN_ / 4) + ", c = i - row * " + std::to_string(PIN_ / 4) + ";\n" +
                   "          " + T_ + "* d = s_in + 4 * c * " + std::to_string(ST) + " + row;\n" +
                   "          d[0] = v[u].x; d[" + std::to_string(ST) + "] = v[u].y; d[" + std::to_string(2 * ST) + "] = v[u].z; d[" +
                   std::to_string(3 * ST) + "] = v[u].w;\n" +
                   "        }\n" +
                   "      }\n    } else\n"
                                : std::string())
            << "    for (int i = threadIdx.x; i < nt * " << PIN_ << "; i += NT) {\n"
            << "      const int row = i / " << PIN_ << ", q = i - row * " << PIN_ << ";\n"
            << "      s_in[q * " << ST << " + row] = gsrc[i];\n"
            << "    }\n"
            << "    __syncthreads();\n"
            << "    const " << T_ << "* s_cur = s_in;\n";
        }
        src << "    " << T_ << "* gdst = gout + (t0 * " << POUT_ << "LL + (" << off_out_ << "LL) - SG_OUT_BASE(0));\n"
            << "    const bool ga = " << (vout_ ? "(reinterpret_cast<unsigned long long>(gdst) & 15ull) == 0" : "false") << ";\n"
            << "    (void)ga;\n"
            ;
        // Output staging (SG_DEMAND_STAGE=1, single-buffered tiles, float4 outputs, every run's input reads
        // before its first rolled loop): once the K warps of a row group have passed their last input read
        // (named barrier), the rows' outputs go into the input tile region, transposed like the inputs, and
        // the CTA copies the tile out with coalesced stores -- instead of per-lane 16-byte stores 1 KB apart.
        const bool stage_env = std::getenv("SG_DEMAND_STAGE") && std::atoi(std::getenv("SG_DEMAND_STAGE")) != 0;
        std::vector<std::string> pre(K), post(K);
        bool stage = stage_env && !db && vout_ && POUT_ <= PIN_ && NT / (32 * K) <= 15;
        for (int k = 0; k < K && stage; k++) {
            const std::string& t = dbodies_[k];
            const size_t last = t.rfind("SG_LDV(");
            const size_t loop = t.find("for (int rr");
            if (last == std::string::npos || (loop != std::string::npos && loop < last)) { stage = false; break; }
            const size_t cut = t.find('\n', last) + 1;
            std::string p1 = t.substr(0, cut), moved;
            // stores before the cut move after the barrier (their values are in registers)
            std::string keep;
            for (size_t i = 0; i < p1.size();) {
                size_t e = p1.find('\n', i);
                if (e == std::string::npos) e = p1.size() - 1;
                const std::string line = p1.substr(i, e + 1 - i);
                (line.find("SG_ST4(") != std::string::npos ? moved : keep) += line;
                i = e + 1;
            }
            pre[k] = keep;
            post[k] = moved + t.substr(cut);
        }
        if (stage) {
            src << "    {\n"
                << "      const int rv = min(r_, nt - 1);  // every lane runs (named barrier); lanes past the tile recompute a row\n"
                << "      const " << T_ << "* xr = s_cur + rv;\n"
                << "      " << T_ << "* ys = s_in + r_;\n"
                << "#define SG_ST4S(g, v) do { const " << VT4 << " t_ = (v); ys[(4 * (g)) * " << ST << "] = t_.x; ys[(4 * (g) + 1) * "
                << ST << "] = t_.y; ys[(4 * (g) + 2) * " << ST << "] = t_.z; ys[(4 * (g) + 3) * " << ST << "] = t_.w; } while (0)\n";
            auto sub = [](std::string x) {
                for (size_t p2 = x.find("SG_ST4("); p2 != std::string::npos; p2 = x.find("SG_ST4(", p2)) x.replace(p2, 7, "SG_ST4S(");
                return x;
            };
            for (int k = 0; k < K; k++)
                src << (K > 1 ? std::string(k ? "      } else if (q_ == " : "      if (q_ == ") + std::to_string(k) + ") {\n" : std::string())
                    << pre[k]
                    << "      asm volatile(\"bar.sync %0, %1;\" :: \"r\"(1 + (int)(threadIdx.x >> 5) / " << K << "), \"r\"("
                    << 32 * K << ") : \"memory\");  // the row group's inputs are dead\n"
                    << sub(post[k]);
            if (K > 1) src << "      }\n";
            src << "#undef SG_ST4S\n"
                << "    }\n"
                << "    __syncthreads();\n"
                << "    for (int i = threadIdx.x; i < nt * " << POUT_ << "; i += NT) {  // coalesced copy-out\n"
                << "      const int row = i / " << POUT_ << ", p = i - row * " << POUT_ << ";\n"
                << "      gdst[i] = s_in[p * " << ST << " + row];\n"
                << "    }\n";
        } else {
            src << "    if (r_ < nt) {\n"
                << "      const " << T_ << "* xr = s_cur + r_;\n"
                << "      " << T_ << "* yg = gdst + (long long)r_ * " << POUT_ << ";\n";
            for (int k = 0; k < K; k++)
                src << (K > 1 ? std::string(k ? "      } else if (q_ == " : "      if (q_ == ") + std::to_string(k) + ") {\n" : std::string())
                    << dbodies_[k];
            if (K > 1) src << "      }\n";
            src << "    }\n";
        }
        src << "    __syncthreads();  // the next tile's loads reuse the rows\n"
            << "  }\n}\n"
            << "#undef SG_LD1\n#undef SG_ST4\n#undef SG_ST1\n";
        ki.has_tma = false;
        ki.tma_in = ki.tma_out = 0;
        ki.name = ki.name_sync;
        ki.threads = ki.threads_sync = NT;
        ki.tile = ki.tile_sync = TR;
        ki.smem = ki.smem_sync = smem;
        ki.min_blocks = 1;
        ki.demand_runs = K;
        ki.source = src.str();
        return ki;
    }
    // number of output components (outputs sharing no input item are in different components)
    int n_components() {
        std::vector<Bits> oc(POUT_);
        for (int64_t p = 0; p < POUT_; p++) oc[p] = cone_of(eout_, off_out_ + p);
        std::vector<int> par(POUT_);
        std::iota(par.begin(), par.end(), 0);
        std::function<int(int)> find = [&](int x) { return par[x] == x ? x : par[x] = find(par[x]); };
        for (int64_t q = 0; q < PIN_; q++) {
            int first = -1;
            for (int64_t p = 0; p < POUT_; p++)
                if (oc[p][q / 64] >> (q % 64) & 1) {
                    if (first < 0) first = (int)p;
                    else par[find((int)p)] = find(first);
                }
        }
        std::set<int> roots;
        for (int64_t p = 0; p < POUT_; p++) roots.insert(find((int)p));
        return (int)roots.size();
    }
    // ---- demand-ordered body: output groups in an order that reuses intermediates (greedy over the
    // sets of firings they need), each group's values computed on demand (memoized firings), inputs
    // re-read from the shared-memory row at every use (volatile: no long input live ranges)
    bool demand_ = false;
    std::map<std::pair<int, int64_t>, std::vector<std::string>> dm_;
    std::string dv(int e, int64_t pos) {
        Ref r = R_.resolve(e, Lin::k(pos));
        if (r.k == Ref::ZERO) return "(" + T_ + ")0";
        if (r.k != Ref::PHYS || !r.pos.is_const()) throw Error(SG_E_UNSUPPORTED, "internal: dynamic ref in register mode");
        if (r.edge == ein_) {
            const int64_t q = r.pos.c - off_in_;
            if (q < 0 || q >= PIN_) throw Error(SG_E_UNSUPPORTED, "internal: register-mode input out of row");
            return "SG_LDV(" + std::to_string(q) + ")";
        }
        const Edge& ed = f_.edges[r.edge];
        const int u = ed.src;
        const Node& n = f_.nodes[u];
        const int64_t q = r.pos.c - ed.pre, g = q / n.push, j = q % n.push;
        auto key = std::make_pair(u, g);
        auto it = dm_.find(key);
        if (it != dm_.end()) return it->second[j];
        std::vector<std::string> xs(n.peek);
        for (int64_t i = 0; i < n.peek; i++) xs[i] = dv(n.in[0], g * n.pop + i);
        std::vector<std::string> ys(n.push);
        body_ << "      " << T_ << " ";
        for (int64_t jj = 0; jj < n.push; jj++) {
            ys[jj] = "v" + std::to_string(nv_++);
            body_ << (jj ? ", " : "") << ys[jj];
        }
        body_ << ";\n      { const " << T_ << " x_[" << n.peek << "] = {";
        for (int64_t i = 0; i < n.peek; i++) body_ << (i ? ", " : "") << xs[i];
        body_ << "}; " << T_ << " y_[" << n.push << "]; " << work_call(u);
        for (int64_t jj = 0; jj < n.push; jj++) body_ << " " << ys[jj] << " = y_[" << jj << "];";
        body_ << " }\n";
        dm_[key] = ys;
        return ys[j];
    }
    void deps_of(int e, int64_t pos, std::set<std::pair<int, int64_t>>& out) {
        Ref r = R_.resolve(e, Lin::k(pos));
        if (r.k == Ref::ZERO || r.edge == ein_) return;
        const Edge& ed = f_.edges[r.edge];
        const Node& n = f_.nodes[ed.src];
        const int64_t g = (r.pos.c - ed.pre) / n.push;
        if (!out.insert({ed.src, g}).second) return;
        for (int64_t i = 0; i < n.peek; i++) deps_of(n.in[0], g * n.pop + i, out);
    }
    // The output groups are split into K contiguous runs of the demand order (about equal new-firing work
    // each; a run recomputes what an earlier run had memoized) -- one body per run, run by its own warps:
    // K warps share one iteration's input row, so a CTA holds NT / K rows instead of NT and the SM K times
    // more warps (DCT 16x16: one row of 1 KB per thread held it to 6 warps per SM).
    std::vector<std::string> dbodies_;
    int demand_K_ = 1;
    void emit_body_demand() {
        const int gs = vout_ ? 4 : 1;
        const int ng = (int)((POUT_ + gs - 1) / gs);
        std::vector<std::set<std::pair<int, int64_t>>> dep(ng);
        for (int g = 0; g < ng; g++)
            for (int64_t p = g * gs; p < std::min<int64_t>(POUT_, (int64_t)(g + 1) * gs); p++) deps_of(eout_, off_out_ + p, dep[g]);
        std::vector<char> done(ng, 0);
        std::vector<int> order;
        int cur = 0;
        for (int step = 0; step < ng; step++) {
            done[cur] = 1;
            order.push_back(cur);
            int best = -1;
            size_t bscore = 0;
            for (int g = 0; g < ng; g++) {
                if (done[g]) continue;
                size_t sc = 0;
                for (auto& k : dep[g]) sc += dep[cur].count(k);
                if (best < 0 || sc > bscore) { best = g; bscore = sc; }
            }
            if (best < 0) break;
            cur = best;
        }
        // K: four runs (64 rows per 256-thread CTA), more when the transposed rows would not fit ~200 KB of
        // shared memory (SG_DEMAND_K overrides); measured: DCT 16x16 K = 1/2/4/8 -> 0.82/0.66/0.40/1.03 ms,
        // MatMul 16 1.40/0.89/0.70/0.91 ms per 2^18 iterations
        int K = 4;
        while (K < 32 && (int64_t)PIN_ * (256 / K + 1) * 4 > 200 * 1024) K *= 2;
        if (const char* e = std::getenv("SG_DEMAND_K")) K = std::max(1, std::atoi(e));
        K = std::max(1, std::min(K, (int)order.size()));
        while (K > 1 && 256 % (32 * K) != 0) K--;
        // new firings per group along the order (one run's memo), then K runs of about equal work
        std::set<std::pair<int, int64_t>> seen;
        std::vector<double> w(order.size());
        double tot = 0;
        for (size_t i = 0; i < order.size(); i++) {
            size_t nw = 0;
            for (auto& k : dep[order[i]]) nw += seen.insert(k).second;
            w[i] = (double)nw + 1.0;
            tot += w[i];
        }
        std::vector<size_t> start{0};
        double acc = 0;
        for (size_t i = 0; i < order.size() && (int)start.size() < K; i++) {
            acc += w[i];
            if (acc >= tot * (double)start.size() / K && i + 1 < order.size()) start.push_back(i + 1);
        }
        K = (int)start.size();
        start.push_back(order.size());
        demand_K_ = K;
        dbodies_.clear();
        for (int k = 0; k < K; k++) {
            dm_.clear();
            std::vector<std::string> gtext;
            std::vector<int> gbase;
            for (size_t i = start[k]; i < start[k + 1]; i++) {
                const int g = order[i];
                body_.str("");
                gbase.push_back(nv_);
                std::string v[4];
                for (int j = 0; j < gs; j++) v[j] = dv(eout_, off_out_ + (int64_t)g * gs + j);
                if (vout_)
                    body_ << "      SG_ST4(" << g << ", make_" << (T_ == "float" ? "float4" : "int4") << "(" << v[0] << ", " << v[1]
                          << ", " << v[2] << ", " << v[3] << "));\n";
                else
                    body_ << "      SG_ST1(" << g << ", " << v[0] << ");\n";
                gtext.push_back(body_.str());
            }
            dbodies_.push_back(roll_groups(gtext, gbase));
        }
        body_.str("");
    }
    // Rolled output groups (SG_DEMAND_ROLL=0 keeps them unrolled): consecutive groups whose code is the same
    // up to (a) the SG_LDV / SG_ST row offsets, which step by the same amount from one group to the next, and
    // (b) their own SSA names -- values memoized by earlier groups are used identically -- become one
    // `#pragma unroll 1` loop over the group's code with the offsets computed from the loop index.  The
    // arithmetic of every output is unchanged; the kernel's straight-line code (DCT / MatMul: 4 runs x
    // 16 groups, tens of KB per run, the instruction-fetch bound) shrinks by the run lengths.
    struct GroupForm { std::string tmpl; std::vector<int64_t> nums; std::vector<char> kind; };
    static GroupForm group_form(const std::string& t, int base) {
        GroupForm f;
        std::string& o = f.tmpl;
        for (size_t i = 0; i < t.size();) {
            auto num_after = [&](const char* kw) -> bool {
                const size_t L = std::strlen(kw);
                if (t.compare(i, L, kw) != 0) return false;
                size_t j = i + L;
                size_t e = j;
                while (e < t.size() && std::isdigit((unsigned char)t[e])) e++;
                if (e == j) return false;
                f.nums.push_back(std::atoll(t.substr(j, e - j).c_str()));
                f.kind.push_back(kw[3] == 'C' ? 1 : 0);  // 1: a coefficient array SG_C<n>
                o += kw;
                o += "@";
                i = e;
                return true;
            };
            if (num_after("SG_LDV(") || num_after("SG_ST4(") || num_after("SG_ST1(")) continue;
            if ((i == 0 || !(std::isalnum((unsigned char)t[i - 1]) || t[i - 1] == '_')) && num_after("SG_C")) continue;
            // SSA names v<n>: the group's own (n >= base) relative, earlier ones (memoized) as they are
            if (t[i] == 'v' && (i == 0 || !(std::isalnum((unsigned char)t[i - 1]) || t[i - 1] == '_')) && i + 1 < t.size() &&
                std::isdigit((unsigned char)t[i + 1])) {
                size_t e = i + 1;
                while (e < t.size() && std::isdigit((unsigned char)t[e])) e++;
                if (e < t.size() && (std::isalnum((unsigned char)t[e]) || t[e] == '_')) { o += t.substr(i, e - i); i = e; continue; }
                const int64_t n = std::atoll(t.substr(i + 1, e - i - 1).c_str());
                o += n >= base ? "w" + std::to_string(n - base) : "v" + std::to_string(n);
                i = e;
                continue;
            }
            o += t[i++];
        }
        return f;
    }
    std::string roll_groups(const std::vector<std::string>& gt, const std::vector<int>& gb) {
        static const bool roll = !std::getenv("SG_DEMAND_ROLL") || std::atoi(std::getenv("SG_DEMAND_ROLL")) != 0;
        std::string out;
        const size_t G = gt.size();
        std::vector<GroupForm> fm(G);
        for (size_t g = 0; g < G; g++) fm[g] = group_form(gt[g], gb[g]);
        size_t g = 0;
        while (g < G) {
            size_t e = g + 1;
            std::vector<int64_t> d;
            if (roll && g + 1 < G && fm[g + 1].tmpl == fm[g].tmpl && fm[g].nums.size() == fm[g + 1].nums.size()) {
                d.resize(fm[g].nums.size());
                for (size_t q = 0; q < d.size(); q++) d[q] = fm[g + 1].nums[q] - fm[g].nums[q];
                e = g + 2;
                while (e < G && fm[e].tmpl == fm[g].tmpl) {
                    bool ok = true;
                    for (size_t q = 0; q < d.size() && ok; q++) ok = fm[e].nums[q] - fm[e - 1].nums[q] == d[q];
                    if (!ok) break;
                    e++;
                }
            }
            // values a rolled group defines must not be read after the loop (they become loop-local)
            if (e - g >= 3) {
                const int lo = gb[g], hi = e < G ? gb[e] : nv_;
                for (size_t h = e; h < G && e - g >= 3; h++) {
                    const std::string& t2 = gt[h];
                    for (size_t i = 0; i + 1 < t2.size(); i++) {
                        if (t2[i] != 'v' || (i && (std::isalnum((unsigned char)t2[i - 1]) || t2[i - 1] == '_')) ||
                            !std::isdigit((unsigned char)t2[i + 1]))
                            continue;
                        const int n = std::atoi(t2.c_str() + i + 1);
                        if (n >= lo && n < hi) { e = g; break; }
                    }
                }
            }
            if (e - g < 3) {  // too short to roll
                out += gt[g];
                g++;
                continue;
            }
            // coefficient arrays that change from group to group: rows of one combined table (same length)
            std::map<size_t, std::string> ctab;
            for (size_t q = 0; q < d.size() && e - g >= 3; q++) {
                if (!fm[g].kind[q] || d[q] == 0) continue;
                int64_t len = -1;
                for (size_t h = g; h < e; h++) {
                    const int64_t l = pool_len("SG_C" + std::to_string(fm[h].nums[q]));
                    if (l <= 0 || (len >= 0 && l != len)) { len = -2; break; }
                    len = l;
                }
                if (len <= 0) { e = g; break; }
                ctab[q] = coef_table(len);
            }
            if (e - g < 3) {
                out += gt[g];
                g++;
                continue;
            }
            // the loop: the group's code with n_q -> (n_q(g) + d_q * rr), own names w<k> local to the body
            std::string body;
            const std::string& t = fm[g].tmpl;
            size_t q = 0;
            for (size_t i = 0; i < t.size(); i++) {
                if (t[i] == '@') {
                    const std::string ix = "(" + std::to_string(fm[g].nums[q]) +
                                           (d[q] ? " + " + std::to_string(d[q]) + " * rr" : std::string()) + ")";
                    if (ctab.count(q)) {  // "SG_C@" -> a row of the combined table
                        body.resize(body.size() - 4);
                        body += ctab[q] + "[" + ix + "]";
                    } else {
                        body += fm[g].kind[q] ? std::to_string(fm[g].nums[q]) : ix;
                    }
                    q++;
                } else {
                    body += t[i];
                }
            }
            out += "      #pragma unroll 1\n      for (int rr = 0; rr < " + std::to_string(e - g) + "; rr++) {  // " +
                   std::to_string(e - g) + " output groups, rolled\n" + body + "      }\n";
            g = e;
        }
        return out;
    }
    bool try_inplace(KernelInfo& ki, std::ostringstream& src, const std::string& VT4) {
        if (PIN_ != POUT_ || PIN_ % 4 != 0 || PIN_ * 4 == 128 || RIN_S_ != ROUT_S_) return false;
        // components: union-find over output positions sharing an input item
        std::vector<Bits> oc(POUT_);
        for (int64_t p = 0; p < POUT_; p++) oc[p] = cone_of(eout_, off_out_ + p);
        std::vector<int> par(POUT_);
        std::iota(par.begin(), par.end(), 0);
        std::function<int(int)> find = [&](int x) { return par[x] == x ? x : par[x] = find(par[x]); };
        for (int64_t q = 0; q < PIN_; q++) {
            int first = -1;
            for (int64_t p = 0; p < POUT_; p++)
                if (oc[p][q / 64] >> (q % 64) & 1) {
                    if (first < 0) first = (int)p;
                    else par[find((int)p)] = find(first);
                }
        }
        std::map<int, std::vector<int64_t>> comps;
        for (int64_t p = 0; p < POUT_; p++) comps[find((int)p)].push_back(p);
        const int C = (int)comps.size();
        if (C < 2 || C > 8) return false;
        struct Comp { int64_t lo, hi; Bits in; };
        std::vector<Comp> cs;
        for (auto& kv : comps) {
            Comp c;
            c.lo = kv.second.front();
            c.hi = kv.second.back() + 1;
            if ((int64_t)kv.second.size() != c.hi - c.lo || c.lo % 4 || c.hi % 4) return false;
            c.in = Bits((PIN_ + 63) / 64, 0);
            for (int64_t p : kv.second) for (size_t w = 0; w < c.in.size(); w++) c.in[w] |= oc[p][w];
            cs.push_back(c);
        }
        // in place: output slot p must not be an input of another component
        for (size_t a = 0; a < cs.size(); a++)
            for (size_t b2 = 0; b2 < cs.size(); b2++) {
                if (a == b2) continue;
                for (int64_t p = cs[a].lo; p < cs[a].hi; p++)
                    if (cs[b2].in[p / 64] >> (p % 64) & 1) return false;
            }
        // tile rows R and stages NS
        const int64_t rowb = RIN_S_ * 4;
        int R = 0, NS = 0;
        for (int r : {128, 96, 64, 32})
            for (int ns : {4, 3, 2})
                if ((int64_t)ns * ((r * rowb + 1023) / 1024 * 1024) + 2048 <= 220 * 1024 && r * (ns - 1) > R * (NS - 1)) {
                    R = r;  // score: rows in flight beyond the tile being computed
                    NS = ns;
                }
        if (!R) return false;
        const int64_t STB = (R * rowb + 1023) / 1024 * 1024;
        const int NWC = (R / 32) * C;
        // bodies (component-relative: loads from its input chunk base, stores to its output base)
        std::vector<std::string> btext(C);
        std::vector<int64_t> ilo(C, 0);
        for (int c = 0; c < C; c++) {
            int64_t first = -1;
            for (int64_t q = 0; q < PIN_ && first < 0; q++) if (cs[c].in[q / 64] >> (q % 64) & 1) first = q;
            ilo[c] = first < 0 ? 0 : first / 4 * 4;
            dmemo_.clear();
            nv_ = 0;
            std::ostringstream o;
            for (int64_t g = 0; g < PIN_ / 4; g++) {
                bool need = false;
                for (int i = 0; i < 4; i++) { int64_t q = 4 * g + i; need |= (cs[c].in[q / 64] >> (q % 64)) & 1; }
                if (need) o << "      const " << VT4 << " iq" << g - ilo[c] / 4 << " = SG_LD4I(" << g - ilo[c] / 4 << ");\n";
            }
            std::ostringstream st;
            for (int64_t g = cs[c].lo / 4; g < cs[c].hi / 4; g++) {
                std::string v[4];
                for (int i = 0; i < 4; i++) v[i] = dval_rel(o, eout_, off_out_ + 4 * g + i, ilo[c]);
                st << "      SG_ST4O(" << g - cs[c].lo / 4 << ", make_" << VT4 << "(" << v[0] << ", " << v[1] << ", " << v[2]
                   << ", " << v[3] << "));\n";
            }
            btext[c] = o.str() + st.str();
        }
        bool shared = true;
        for (int c = 1; c < C; c++) shared = shared && btext[c] == btext[0] && cs[c].hi - cs[c].lo == cs[0].hi - cs[0].lo;
        std::ostringstream bodies;
        std::string ibx = "0", obx = "0";
        for (int c = C - 1; c >= 0; c--) {
            ibx = c == C - 1 ? std::to_string(ilo[c] / 4) : "(comp == " + std::to_string(c) + " ? " + std::to_string(ilo[c] / 4) + " : " + ibx + ")";
            obx = c == C - 1 ? std::to_string(cs[c].lo / 4) : "(comp == " + std::to_string(c) + " ? " + std::to_string(cs[c].lo / 4) + " : " + obx + ")";
        }
        bodies << "    const int ib = " << ibx << ", ob = " << obx << ";\n"
               << "    const unsigned char* xi = xb + ib * 16;\n"
               << "    unsigned char* xo = xb + ob * 16;\n";
        if (shared) {
            bodies << "    {  // one body shared by all " << C << " structurally identical components\n" << btext[0]
                   << "      lo = ob * 4; len = " << cs[0].hi - cs[0].lo << ";\n    }\n";
        } else {
            for (int c = 0; c < C; c++)
                bodies << "    " << (c ? "} else if" : "if") << " (comp == " << c << ") {\n" << btext[c]
                       << "      lo = " << cs[c].lo << "; len = " << cs[c].hi - cs[c].lo << ";\n";
            bodies << "    }\n";
        }
        ki.has_tma = true;
        ki.tma_in = ki.tma_out = 2;
        ki.threads = NWC * 32 + 32;
        ki.tile = R;
        ki.smem = (size_t)(NS * STB + 2048);
        src << "// ---- in-place component pipeline: " << C << " components, " << R << " rows per tile, " << NS
            << " stages\n"
            << "#define SG_LD4I(g) (*reinterpret_cast<const " << VT4 << "*>(xi + ((g) << 4)))\n"
            << "#define SG_ST4O(g, v) (*reinterpret_cast<" << VT4 << "*>(xo + ((g) << 4)) = (v))\n"
            << "extern \"C\" __global__ void __launch_bounds__(" << NWC * 32 + 32 << ", 1) " << ki.name
            << "(const SgArgs a, const __grid_constant__ SgTmap tin, const __grid_constant__ SgTmap tout) {\n"
            << "  constexpr int R = " << R << ", NWC = " << NWC << ", NS = " << NS << ", C = " << C << ";\n"
            << "  constexpr int STB = " << STB << ";\n"
            << "  extern __shared__ __align__(1024) unsigned char sg_smem_raw[];\n"
            << "  unsigned char* st = reinterpret_cast<unsigned char*>((reinterpret_cast<unsigned long long>(sg_smem_raw) + 1023ull) & ~1023ull);\n"
            << "  unsigned long long* full = reinterpret_cast<unsigned long long*>(st + NS * STB);\n"
            << "  unsigned long long* empty = full + NS;\n"
            << "  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;\n"
            << "  const long long nrows = SG_K_END - SG_K_BEGIN;\n"
            << "  const long long ntiles = (nrows + R - 1) / R;\n"
            << "  if (threadIdx.x == 0) {\n"
            << "    for (int s = 0; s < NS; s++) { sg_mbar_init(&full[s], 1); sg_mbar_init(&empty[s], NWC); }\n"
            << "    sg_fence_barrier_init();\n"
            << "  }\n"
            << "  __syncthreads();\n"
            << "  if (warp == NWC) {  // ---- producer warp: one bulk copy per row\n"
            << "    const " << T_ << "* gin = SG_IN(0) + (SG_K_BEGIN * " << PIN_ << "LL + (" << off_in_ << "LL) - SG_IN_BASE(0));\n"
            << "    int i = 0;\n"
            << "    for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, i++) {\n"
            << "      const int s = i % NS;\n"
            << "      const int nt = (int)min((long long)R, nrows - t * R);\n"
            << "      sg_mbar_wait(&empty[s], ((i / NS) & 1) ^ 1);\n"
            << "      if (lane == 0) sg_mbar_arrive_expect_tx(&full[s], (unsigned)(nt * " << PIN_ * 4 << "));\n"
            << "      __syncwarp();\n"
            << "      for (int r = lane; r < nt; r += 32)\n"
            << "        sg_bulk_g2s(st + s * STB + r * " << rowb << ", gin + (t * R + r) * " << PIN_ << "LL, " << PIN_ * 4
            << ", &full[s]);\n"
            << "    }\n"
            << "    return;\n"
            << "  }\n"
            << "  // ---- consumer warps: warp w runs component w % C on rows (w / C) * 32 + lane\n"
            << "  " << T_ << "* gout = SG_OUT(0) + (SG_K_BEGIN * " << POUT_ << "LL + (" << off_out_ << "LL) - SG_OUT_BASE(0));\n"
            << "  const int comp = warp % C;\n"
            << "  const int row = (warp / C) * 32 + lane;\n"
            << "  int i = 0;\n"
            << "  for (long long t = blockIdx.x; t < ntiles; t += gridDim.x, i++) {\n"
            << "    const int s = i % NS;\n"
            << "    const int nt = (int)min((long long)R, nrows - t * R);\n"
            << "    sg_mbar_wait(&full[s], (i / NS) & 1);\n"
            << "    unsigned char* xb = st + s * STB + row * " << rowb << ";\n"
            << "    int lo = 0, len = 0;\n"
            << "    if (row < nt) {\n"
            << bodies.str()
            << "      sg_fence_proxy_async();\n"
            << "      sg_bulk_s2g(gout + (t * R + row) * " << POUT_ << "LL + lo, xb + lo * 4, (unsigned)(len * 4));\n"
            << "      sg_bulk_commit();\n"
            << "      sg_bulk_wait_read<0>();\n"
            << "    }\n"
            << "    __syncwarp();\n"
            << "    if (lane == 0) sg_mbar_arrive(&empty[s]);\n"
            << "  }\n"
            << "  sg_bulk_wait<0>();\n"
            << "}\n"
            << "#undef SG_LD4I\n#undef SG_ST4O\n";
        return true;
    }

    int ein_ = -1, eout_ = -1;
    int64_t PIN_ = 0, POUT_ = 0, off_in_ = 0, off_out_ = 0, RIN_S_ = 0, ROUT_S_ = 0;
    bool vin_ = false, vout_ = false;
    std::ostringstream body_;
    std::map<std::pair<int, int64_t>, std::string> val_;  // (phys edge, local pos) -> SSA name
    std::set<int64_t> loaded_;                            // input groups / items loaded
    int nv_ = 0;

    // Row stride (items) in shared memory: 128-bit row reads by 8 consecutive
    // threads hit 8 distinct 16-byte bank groups iff stride/4 is odd; scalar
    // rows use an odd stride.
    static int64_t row_stride(int64_t P) {
        if (P % 4 == 0) return (P / 4) % 2 == 1 ? P : P + 4;
        return P % 2 == 1 ? P : P + 1;
    }
    std::string input_name(int64_t pos) {
        int64_t r = pos - off_in_;
        if (r < 0 || r >= PIN_) throw Error(SG_E_UNSUPPORTED, "internal: register-mode input out of row");
        if (vin_) {
            int64_t g = r / 4;
            if (!loaded_.count(g)) {
                loaded_.insert(g);
                body_ << "      const " << (T_ == "float" ? "float4" : "int4") << " iq" << g << " = SG_LD4(" << g << ");\n";
            }
            static const char* comp[4] = {"x", "y", "z", "w"};
            return "iq" + std::to_string(g) + "." + comp[r % 4];
        }
        if (!loaded_.count(r)) {
            loaded_.insert(r);
            body_ << "      const " << T_ << " xi" << r << " = SG_LD1(" << r << ");\n";
        }
        return "xi" + std::to_string(r);
    }
    std::string value_of(const Ref& rf) {
        if (rf.k == Ref::ZERO) return "(" + T_ + ")0";
        if (rf.k != Ref::PHYS || !rf.pos.is_const()) throw Error(SG_E_UNSUPPORTED, "internal: dynamic ref in register mode");
        if (rf.edge == ein_) return input_name(rf.pos.c);
        auto it = val_.find({rf.edge, rf.pos.c});
        if (it == val_.end()) throw Error(SG_E_UNSUPPORTED, "internal: value used before definition");
        return it->second;
    }
    void emit_body() {
        // output sources and readiness bookkeeping
        std::vector<Ref> osrc(POUT_);
        std::map<std::pair<int, int64_t>, std::vector<int64_t>> waiters;
        int gs = vout_ ? 4 : 1;
        std::vector<int> pending((POUT_ + gs - 1) / gs, 0);
        for (int64_t p = 0; p < POUT_; p++) {
            osrc[p] = R_.resolve(eout_, Lin::k(off_out_ + p));
            if (osrc[p].k == Ref::PHYS && osrc[p].edge != ein_) {
                waiters[{osrc[p].edge, osrc[p].pos.c}].push_back(p / gs);
                pending[p / gs]++;
            }
        }
        std::vector<char> stored(pending.size(), 0);
        auto store_group = [&](int64_t g) {
            if (stored[g]) return;
            stored[g] = 1;
            if (vout_) {
                std::string v[4];
                for (int i = 0; i < 4; i++) v[i] = value_of(osrc[4 * g + i]);
                body_ << "      SG_ST4(" << g << ", make_" << (T_ == "float" ? "float4" : "int4") << "(" << v[0] << ", "
                      << v[1] << ", " << v[2] << ", " << v[3] << "));\n";
            } else {
                std::string v0 = value_of(osrc[g]);
                body_ << "      SG_ST1(" << g << ", " << v0 << ");\n";
            }
        };
        for (size_t g = 0; g < pending.size(); g++)
            if (pending[g] == 0) store_group((int64_t)g);
        for (int v : nodes_) {
            const Node& n = f_.nodes[v];
            if (is_view_node(n)) continue;
            int ein = n.in[0], eo = n.out[0];
            for (int64_t j = 0; j < n.rep; j++) {
                int64_t lf = n.ninit + j;
                std::vector<std::string> xs(n.peek);
                for (int64_t i = 0; i < n.peek; i++) xs[i] = value_of(R_.resolve(ein, Lin::k(lf * n.pop + i)));
                std::vector<std::string> ys(n.push);
                body_ << "      " << T_ << " ";
                for (int64_t jj = 0; jj < n.push; jj++) {
                    ys[jj] = "v" + std::to_string(nv_++);
                    body_ << (jj ? ", " : "") << ys[jj];
                }
                body_ << ";\n      { const " << T_ << " x_[" << n.peek << "] = {";
                for (int64_t i = 0; i < n.peek; i++) body_ << (i ? ", " : "") << xs[i];
                body_ << "}; " << T_ << " y_[" << n.push << "]; " << work_call(v);
                for (int64_t jj = 0; jj < n.push; jj++) body_ << " " << ys[jj] << " = y_[" << jj << "];";
                body_ << " }\n";
                const Edge& oe = f_.edges[eo];
                for (int64_t jj = 0; jj < n.push; jj++) {
                    int64_t pos = oe.pre + lf * n.push + jj;
                    val_[{eo, pos}] = ys[jj];
                    auto w = waiters.find({eo, pos});
                    if (w != waiters.end())
                        for (int64_t g : w->second)
                            if (--pending[g] == 0) store_group(g);
                }
            }
        }
        for (size_t g = 0; g < pending.size(); g++)
            if (!stored[g]) throw Error(SG_E_UNSUPPORTED, "internal: output group never produced");
    }
};

// ------------------------------------------------------------ bitslice mode
// A partition whose compute filters are all bit kinds -- INTO_BITS reading the boundary input,
// BITS_TO_INT writing the boundary output, XOR / XOR_CONST / SBOX in between -- depends only on
// bit 0 of every inner item (XOR is bitwise, SBOX and BITS_TO_INT read x & 1).  One thread then
// runs 32 iterations at once: an inner item is a 32-bit word whose bit j belongs to the thread's
// j-th iteration (bitslicing across iterations), so one LOP3 does the work of 32 firings.
// INTO_BITS / BITS_TO_INT become 32x32 bit transposes in registers; an S-box becomes a LOP3
// circuit derived from its table at compile time (3-input cofactor functions + a mux tree);
// XOR_CONST key bits become complement flags folded into the LUT immediates (free).
static bool is_bit_kind(int k) {
    return k == SG_K_INTO_BITS || k == SG_K_BITS_TO_INT || k == SG_K_XOR || k == SG_K_XOR_CONST || k == SG_K_SBOX;
}

bool bitslice_eligible(const Flat& f, const std::vector<int>& nodes, std::string* why) {
    auto fail = [&](const std::string& s) { if (why) *why = s; return false; };
    if (f.dtype != SG_I32) return fail("not an int32 graph");
    if (!register_mode_eligible(f, nodes, why)) return false;
    for (int v : nodes) {
        const Node& n = f.nodes[v];
        if (n.type == N_FILTER && !is_view_kind(n.kind) && !is_bit_kind(n.kind))
            return fail(std::string("non-bit filter ") + kind_name(n.kind));
    }
    std::vector<int> ins, outs;
    partition_boundary(f, nodes, ins, outs);
    if (f.edges[ins[0]].per_iter > 8 || f.edges[outs[0]].per_iter > 8) return fail("row too wide for bitslicing");
    return true;  // domain checks (words only at INTO_BITS / BITS_TO_INT) happen during generation
}

class BitGen : public GenBase {
public:
    using GenBase::GenBase;

    KernelInfo run(const CodegenOpts& opt) {
        KernelInfo ki;
        ki.mode = 1;
        ki.name = "sg_part" + std::to_string(part_);
        ki.name_sync = ki.name;
        fill_io(ki);
        ein_ = ins_[0];
        eout_ = outs_[0];
        PIN_ = f_.edges[ein_].per_iter;
        POUT_ = f_.edges[eout_].per_iter;
        off_in_ = ki.in_lo[0];
        off_out_ = ki.out_lo[0];
        // a run of identical periods (cipher rounds) becomes a rolled loop over a state array
        const bool rolled = !std::getenv("SG_BS_NOROLL") && try_roll();
        // output words: each must be produced by a BITS_TO_INT firing
        std::vector<std::vector<BV>> obits(POUT_);
        for (int64_t p = 0; p < POUT_; p++) {
            Ref r = cur_R_->resolve(eout_, Lin::k(off_out_ + p));
            if (r.k != Ref::PHYS || r.edge == ein_) throw Error(SG_E_UNSUPPORTED, "bitslice: output item is not a BITS_TO_INT word");
            const Edge& ed = f_.edges[r.edge];
            const Node& n = f_.nodes[ed.src];
            if (n.kind != SG_K_BITS_TO_INT) throw Error(SG_E_UNSUPPORTED, "bitslice: output not from BITS_TO_INT");
            int64_t g = (r.pos.c - ed.pre) / n.push;
            std::vector<BV> b(32);
            for (int i = 0; i < 32; i++) b[i] = bit(n.in[0], g * n.pop + i);
            obits[p] = b;
        }
        const int NT = opt.threads > 0 ? opt.threads : 128;
        ki.threads = ki.threads_sync = NT;
        ki.tile = ki.tile_sync = NT * 32;
        ki.smem = ki.smem_sync = 0;
        std::ostringstream s;
        s << header(rolled ? "bitslice, rolled rounds" : "bitslice") << consts_.str() << args_struct();
        s << "extern \"C\" __global__ void __launch_bounds__(" << NT << ", " << (NT <= 128 ? 2 : 1) << ") " << ki.name << "(const SgArgs a) {\n"
          << "  const int lane = threadIdx.x & 31;\n"
          << "  const long long wstep = (long long)gridDim.x * " << NT / 32 << " * 1024;\n"
          << "  const " << T_ << "* gin = SG_IN(0) + ((" << off_in_ << "LL) - SG_IN_BASE(0));\n"
          << "  " << T_ << "* gout = SG_OUT(0) + ((" << off_out_ << "LL) - SG_OUT_BASE(0));\n"
          << "  const bool vin = " << (PIN_ == 2 || PIN_ == 4 ? "(reinterpret_cast<unsigned long long>(gin) & " + std::to_string(PIN_ * 4 - 1) + "ull) == 0" : std::string("false")) << ";\n"
          << "  const bool vout = " << (POUT_ == 2 || POUT_ == 4 ? "(reinterpret_cast<unsigned long long>(gout) & " + std::to_string(POUT_ * 4 - 1) + "ull) == 0" : std::string("false")) << ";\n"
          << "  // CTA-uniform tile loop (every warp of the CTA iterates equally often: barriers are safe);\n"
          << "  // warps past the end compute on zeros and store nothing\n"
          << "  for (long long cb = SG_K_BEGIN + (long long)blockIdx.x * " << NT * 32 << "LL; cb < SG_K_END; cb += wstep) {\n"
          << "    const long long wb = cb + (long long)(threadIdx.x >> 5) * 1024;\n";
        // loads: word q of iteration wb + 32 j + lane -> w<q>[j]
        for (int64_t q = 0; q < PIN_; q++) s << "    unsigned w" << q << "[32];\n";
        s << "#pragma unroll\n"
          << "    for (int j = 0; j < 32; j++) {\n"
          << "      const long long k = wb + 32 * j + lane;\n"
          << "      if (k < SG_K_END) {\n";
        if (PIN_ == 2 || PIN_ == 4) {
            s << "        if (vin) {\n"
              << "          const int" << PIN_ << " t = __ldg(reinterpret_cast<const int" << PIN_ << "*>(gin + k * " << PIN_ << "LL));\n";
            static const char* comp[4] = {"x", "y", "z", "w"};
            for (int64_t q = 0; q < PIN_; q++) s << "          w" << q << "[j] = (unsigned)t." << comp[q] << ";\n";
            s << "        } else {\n";
            for (int64_t q = 0; q < PIN_; q++) s << "          w" << q << "[j] = (unsigned)__ldg(gin + k * " << PIN_ << "LL + " << q << ");\n";
            s << "        }\n";
        } else {
            for (int64_t q = 0; q < PIN_; q++) s << "        w" << q << "[j] = (unsigned)__ldg(gin + k * " << PIN_ << "LL + " << q << ");\n";
        }
        s << "      } else {\n";
        for (int64_t q = 0; q < PIN_; q++) s << "        w" << q << "[j] = 0u;\n";
        s << "      }\n    }\n";
        for (int64_t q : used_cols_) s << "    sg_transpose32(w" << q << ");\n";
        s << body_.str();
        for (int64_t p = 0; p < POUT_; p++) {
            s << "    unsigned o" << p << "[32];\n";
            for (int i = 0; i < 32; i++) s << "    o" << p << "[" << 31 - i << "] = " << obits[p][i].expr() << ";\n";
            s << "    sg_transpose32(o" << p << ");\n";
        }
        s << "#pragma unroll\n"
          << "    for (int j = 0; j < 32; j++) {\n"
          << "      const long long k = wb + 32 * j + lane;\n"
          << "      if (k < SG_K_END) {\n";
        if (POUT_ == 2 || POUT_ == 4) {
            s << "        if (vout) {\n"
              << "          reinterpret_cast<int" << POUT_ << "*>(gout + k * " << POUT_ << "LL)[0] = make_int" << POUT_ << "(";
            for (int64_t p = 0; p < POUT_; p++) s << (p ? ", " : "") << "(int)o" << p << "[j]";
            s << ");\n        } else {\n";
            for (int64_t p = 0; p < POUT_; p++) s << "          gout[k * " << POUT_ << "LL + " << p << "] = (int)o" << p << "[j];\n";
            s << "        }\n";
        } else {
            for (int64_t p = 0; p < POUT_; p++) s << "        gout[k * " << POUT_ << "LL + " << p << "] = (int)o" << p << "[j];\n";
        }
        s << "      }\n    }\n  }\n}\n";
        ki.source = s.str();
        return ki;
    }

private:
    struct BV {  // a packed bit value: register name (or literal) and a complement flag
        std::string s;
        bool neg = false;
        std::string expr() const { return neg ? "(~" + s + ")" : s; }
        bool operator==(const BV& o) const { return s == o.s && neg == o.neg; }
        bool operator<(const BV& o) const { return s != o.s ? s < o.s : neg < o.neg; }
    };
    int ein_ = -1, eout_ = -1;
    int64_t PIN_ = 0, POUT_ = 0, off_in_ = 0, off_out_ = 0;
    std::ostringstream body_;
    // evaluation context: resolver, and (rolled loop) the edge whose items live in the state array S
    const Resolver* cur_R_ = &R_;
    std::unique_ptr<Resolver> rpro_, rbody_, repi_;
    int bedge_ = -2;
    int64_t blo_ = 0, bm_ = 0;
    std::map<int, int64_t> keyslot_;  // XOR_CONST node of period 0 -> first slot in the per-round key table

    // Edges every input -> output path crosses (pipeline boundaries), in topological order.
    std::vector<int> cut_edges() const {
        std::vector<char> in(f_.nodes.size(), 0);
        for (int v : nodes_) in[v] = 1;
        const int s0 = f_.edges[ein_].dst, t0 = f_.edges[eout_].src;
        std::vector<int> cuts;
        for (int e = 0; e < (int)f_.edges.size(); e++) {
            const Edge& ed = f_.edges[e];
            if (ed.src < 0 || ed.dst < 0 || !in[ed.src] || !in[ed.dst]) continue;
            std::vector<char> seen(f_.nodes.size(), 0);
            std::vector<int> st{s0};
            seen[s0] = 1;
            while (!st.empty()) {
                int u = st.back();
                st.pop_back();
                for (int oe : f_.nodes[u].out) {
                    if (oe == e) continue;
                    int w = f_.edges[oe].dst;
                    if (w >= 0 && in[w] && !seen[w]) { seen[w] = 1; st.push_back(w); }
                }
            }
            if (!seen[t0]) cuts.push_back(e);
        }
        std::sort(cuts.begin(), cuts.end(), [&](int a, int b) { return f_.edges[a].src < f_.edges[b].src; });
        return cuts;
    }
    // structural signature of the node id range [a, b] (XOR_CONST constants excluded)
    std::vector<int64_t> signature(int a, int b) const {
        std::vector<int64_t> sig;
        for (int v = a; v <= b; v++) {
            const Node& n = f_.nodes[v];
            sig.push_back(n.type);
            sig.push_back(n.kind);
            sig.push_back(n.rep);
            const size_t niv = n.type == N_FILTER && n.kind == SG_K_XOR_CONST ? 1 : n.iv.size();
            sig.push_back((int64_t)niv);
            for (size_t i = 0; i < niv; i++) sig.push_back(n.iv[i]);
            for (float x : n.fv) { uint32_t w; std::memcpy(&w, &x, 4); sig.push_back(w); }
            for (int32_t w : n.w) sig.push_back(w);
            for (int e : n.in) {
                const Edge& ed = f_.edges[e];
                sig.push_back(ed.src >= a && ed.src <= b ? ed.src - a : -1);
                sig.insert(sig.end(), {ed.sport, ed.pop, ed.peek, ed.push, ed.pre, ed.per_iter});
            }
            for (int e : n.out) {
                const Edge& ed = f_.edges[e];
                sig.push_back(ed.dst >= a && ed.dst <= b ? ed.dst - a : -1);
                sig.push_back(ed.dport);
            }
        }
        return sig;
    }
    static int64_t iter_lo(const Flat& f, int e) {  // first position of iteration 0 on edge e
        const Edge& ed = f.edges[e];
        return ed.pre + f.nodes[ed.src].ninit * ed.push;
    }
    // Find the longest run of >= 3 identical periods between cut edges; set up prologue / body /
    // epilogue resolvers and emit the prologue, the state array and the rolled loop.
    bool try_roll() {
        std::vector<int> cuts = cut_edges();
        const int nseg = (int)cuts.size() - 1;
        if (nseg < 3) return false;
        std::vector<std::vector<int64_t>> sig(nseg);
        for (int i = 0; i < nseg; i++) {
            const int a = f_.edges[cuts[i]].dst, b = f_.edges[cuts[i + 1]].src;
            if (b < a) return false;
            sig[i] = signature(a, b);
        }
        int bs = -1, bp = 0, bk = 0;
        int64_t bcov = 0;
        for (int p = 1; p <= nseg / 3; p++)
            for (int st = 0; st + 3 * p <= nseg; st++) {
                int k = 1;
                while (st + (k + 1) * p <= nseg) {
                    bool same = true;
                    for (int t = 0; t < p && same; t++) same = sig[st + k * p + t] == sig[st + t];
                    if (!same) break;
                    k++;
                }
                const int64_t cov = (int64_t)k * (f_.edges[cuts[st + p]].src - f_.edges[cuts[st]].dst + 1);
                if (k >= 3 && cov > bcov) { bcov = cov; bs = st; bp = p; bk = k; }
            }
        if (bs < 0) return false;
        const int e0 = cuts[bs], e1 = cuts[bs + bp], eend = cuts[bs + bk * bp];
        const int64_t m = f_.edges[e0].per_iter;
        if (f_.edges[e1].per_iter != m || f_.edges[eend].per_iter != m || m > 256) return false;
        const int64_t lo0 = iter_lo(f_, e0), lo1 = iter_lo(f_, e1), loend = iter_lo(f_, eend);
        if (lo0 != lo1 || lo0 != loend) return false;
        const int a0 = f_.edges[e0].dst, b0 = f_.edges[e1].src;   // period 0 = node ids [a0, b0]
        const int np = b0 - a0 + 1;
        const int aend = f_.edges[eend].dst;                       // epilogue starts here
        std::vector<int> pro, body, epi;  // periods 1..K-1 are never evaluated (the loop replays period 0)
        for (int v : nodes_) {
            if (v < a0) pro.push_back(v);
            else if (v <= b0) body.push_back(v);
            else if (v >= aend) epi.push_back(v);
        }
        if (pro.empty()) return false;
        // per-round key table (only if the XOR_CONST constants differ between rounds)
        int64_t kw = 0;
        std::map<int, int64_t> slots;
        bool differ = false;
        for (int v = a0; v <= b0; v++) {
            const Node& n = f_.nodes[v];
            if (n.type != N_FILTER || n.kind != SG_K_XOR_CONST) continue;
            slots[v] = kw;
            kw += n.iv[0];
            for (int k = 1; k < bk; k++) differ = differ || f_.nodes[v + k * np].iv != n.iv;
        }
        std::vector<uint32_t> table;
        if (differ) {
            for (int k = 0; k < bk; k++)
                for (auto& kv : slots) {
                    const Node& n = f_.nodes[kv.first + k * np];
                    for (int i = 0; i < n.iv[0]; i++) table.push_back((n.iv[1 + i] & 1) ? 0xFFFFFFFFu : 0u);
                }
            keyslot_ = slots;
            consts_ << "__constant__ unsigned SG_BSKEY[" << table.size() << "] = {";
            for (size_t i = 0; i < table.size(); i++) consts_ << (i ? "," : "") << (i % 8 == 0 ? "\n  " : "") << "0x" << std::hex << table[i] << std::dec << "u";
            consts_ << "};\n";
        }
        rpro_.reset(new Resolver(f_, pro));
        rbody_.reset(new Resolver(f_, body));
        repi_.reset(new Resolver(f_, epi));
        // prologue: the state at the run's start
        cur_R_ = rpro_.get();
        std::vector<BV> s0(m);
        for (int64_t j = 0; j < m; j++) s0[j] = bit(e0, lo0 + j);
        body_ << "    unsigned S[" << m << "];\n";
        for (int64_t j = 0; j < m; j++) body_ << "    S[" << j << "] = " << s0[j].expr() << ";\n";
        // body: one period from S to the next S
        lop_memo_.clear();
        const std::string pre = body_.str();
        body_.str("");
        cur_R_ = rbody_.get();
        bedge_ = e0;
        blo_ = lo0;
        bm_ = m;
        std::vector<BV> s1(m);
        for (int64_t j = 0; j < m; j++) s1[j] = bit(e1, lo1 + j);
        std::string loop = body_.str();
        body_.str("");
        body_ << pre << "    // " << bk << " identical rounds of " << np << " nodes, rolled\n"
              << "#pragma unroll 1\n"
              << "    for (int r = 0; r < " << bk << "; r++) {\n";
        if (differ) body_ << "      const unsigned* kt = SG_BSKEY + r * " << kw << ";\n";
        body_ << loop;
        for (int64_t j = 0; j < m; j++) body_ << "    const unsigned n" << j << " = " << s1[j].expr() << ";\n";
        for (int64_t j = 0; j < m; j++) body_ << "    S[" << j << "] = n" << j << ";\n";
        body_ << "    }\n";
        // epilogue: everything after the run reads the final S
        lop_memo_.clear();
        keyslot_.clear();
        cur_R_ = repi_.get();
        bedge_ = eend;
        return true;
    }
    int nv_ = 0;
    std::set<int64_t> used_cols_;
    std::map<std::pair<int, int64_t>, std::vector<BV>> memo_;
    std::map<std::tuple<int, BV, BV, BV>, BV> lop_memo_;

    BV fresh(const std::string& rhs) {
        std::string v = "b" + std::to_string(nv_++);
        body_ << "    const unsigned " << v << " = " << rhs << ";\n";
        // optional lockstep barriers: the warps of a CTA stay within one instruction-cache window
        static const int bar = std::getenv("SG_BS_BAR") ? std::atoi(std::getenv("SG_BS_BAR")) : 0;
        if (bar > 0 && nv_ % bar == 0) body_ << "    __syncthreads();\n";
        return {v, false};
    }
    static BV zero() { return {"0u", false}; }
    static BV ones() { return {"0u", true}; }
    // lop3 of true values A, B, C with truth table F (index A<<2 | B<<1 | C); complements folded in
    BV lop3(int F, BV A, BV B, BV C) {
        const int flip = (A.neg ? 4 : 0) | (B.neg ? 2 : 0) | (C.neg ? 1 : 0);
        int L = 0;
        for (int p = 0; p < 8; p++)
            if ((F >> (p ^ flip)) & 1) L |= 1 << p;
        if (L == 0x00) return zero();
        if (L == 0xFF) return ones();
        A.neg = B.neg = C.neg = false;
        if (L == 0xF0) return A;
        if (L == 0x0F) return {A.s, true};
        if (L == 0xCC) return B;
        if (L == 0x33) return {B.s, true};
        if (L == 0xAA) return C;
        if (L == 0x55) return {C.s, true};
        // a function and its complement share one LOP3 (the complement becomes a flag)
        const bool cneg = L > 255 - L;
        if (cneg) L = 255 - L;
        auto key = std::make_tuple(L, A, B, C);
        auto it = lop_memo_.find(key);
        BV r;
        if (it != lop_memo_.end()) {
            r = it->second;
        } else {
            char b[32];
            std::snprintf(b, sizeof b, "0x%02x", L);
            r = fresh("sg_lop3<" + std::string(b) + ">(" + A.s + ", " + B.s + ", " + C.s + ")");
            lop_memo_[key] = r;
        }
        r.neg = cneg;
        return r;
    }
    BV mux(const BV& s, const BV& x1, const BV& x0) {  // s ? x1 : x0
        if (x1 == x0) return x1;
        return lop3(0xCA, s, x1, x0);
    }
    // S-box as a circuit: output bit i of t[idx(b)], idx = 32 b0 + 16 b5 + 8 b1 + 4 b2 + 2 b3 + b4.
    // Three inputs feed 3-input cofactor functions (one LOP3 each), the other three drive a mux tree;
    // the split and the mux order with the fewest gates are chosen by counting.
    std::vector<BV> sbox(const std::vector<BV>& x, const std::vector<int32_t>& t) {
        auto tab = [&](int out, const int b[6]) {
            int idx = 32 * b[0] + 16 * b[5] + 8 * b[1] + 4 * b[2] + 2 * b[3] + b[4];
            return (t[idx] >> (3 - out)) & 1;
        };
        int best = 1 << 30;
        std::vector<int> bl, bs;
        for (int m = 0; m < 64; m++) {
            if (__builtin_popcount(m) != 3) continue;
            std::vector<int> lv, sv;
            for (int i = 0; i < 6; i++) (m >> i & 1 ? lv : sv).push_back(i);
            std::sort(sv.begin(), sv.end());
            do {
                // count distinct non-trivial cofactors and muxes (structural, without complements)
                std::set<int> cof;
                std::set<std::vector<int>> muxes;
                for (int out = 0; out < 4; out++) {
                    std::vector<int> lvl;
                    for (int sa = 0; sa < 8; sa++) {
                        int u = 0;
                        for (int p = 0; p < 8; p++) {
                            int b[6];
                            b[lv[0]] = p >> 2 & 1; b[lv[1]] = p >> 1 & 1; b[lv[2]] = p & 1;
                            b[sv[0]] = sa >> 2 & 1; b[sv[1]] = sa >> 1 & 1; b[sv[2]] = sa & 1;
                            u |= tab(out, b) << p;
                        }
                        int canon = std::min(u, 255 - u);
                        if (canon != 0 && canon != 0x0F && canon != 0x33 && canon != 0x55) cof.insert(canon);
                        lvl.push_back(u);
                    }
                    int id = 1000;
                    for (int d = 2; d >= 0; d--) {
                        std::vector<int> nx;
                        for (size_t k = 0; k < lvl.size(); k += 2) {
                            if (lvl[k] == lvl[k + 1]) { nx.push_back(lvl[k]); continue; }
                            std::vector<int> key = {d, lvl[k], lvl[k + 1]};
                            muxes.insert(key);
                            nx.push_back(id++ + out * 100000);
                        }
                        lvl = nx;
                    }
                }
                int cost = (int)cof.size() + (int)muxes.size();
                if (cost < best) { best = cost; bl = lv; bs = sv; }
            } while (std::next_permutation(sv.begin(), sv.end()));
        }
        std::vector<BV> y(4);
        for (int out = 0; out < 4; out++) {
            std::vector<BV> lvl;
            for (int sa = 0; sa < 8; sa++) {
                int u = 0;
                for (int p = 0; p < 8; p++) {
                    int b[6];
                    b[bl[0]] = p >> 2 & 1; b[bl[1]] = p >> 1 & 1; b[bl[2]] = p & 1;
                    b[bs[0]] = sa >> 2 & 1; b[bs[1]] = sa >> 1 & 1; b[bs[2]] = sa & 1;
                    u |= tab(out, b) << p;
                }
                lvl.push_back(lop3(u, x[bl[0]], x[bl[1]], x[bl[2]]));
            }
            for (int d = 2; d >= 0; d--) {   // mux on bs[d]: pairs (sa with bit (2-d) = 0 / 1)
                std::vector<BV> nx;
                for (size_t k = 0; k < lvl.size(); k += 2) nx.push_back(mux(x[bs[d]], lvl[k + 1], lvl[k]));
                lvl = nx;
            }
            y[out] = lvl[0];
        }
        return y;
    }
    // packed value of item `pos` of edge e (bit domain)
    BV bit(int e, int64_t pos) {
        Ref r = cur_R_->resolve(e, Lin::k(pos));
        if (r.k == Ref::ZERO) return zero();
        if (r.k != Ref::PHYS) throw Error(SG_E_UNSUPPORTED, "bitslice: non-constant position");
        if (r.edge == bedge_) {  // rolled loop: the state array
            const int64_t j = r.pos.c - blo_;
            if (j < 0 || j >= bm_) throw Error(SG_E_UNSUPPORTED, "bitslice: state position out of range");
            return {"S[" + std::to_string(j) + "]", false};
        }
        if (r.edge == ein_) throw Error(SG_E_UNSUPPORTED, "bitslice: a raw input word is used as a bit");
        const Edge& ed = f_.edges[r.edge];
        const int u = ed.src;
        const Node& n = f_.nodes[u];
        const int64_t q = r.pos.c - ed.pre, g = q / n.push, j = q % n.push;
        auto key = std::make_pair(u, g);
        auto it = memo_.find(key);
        if (it != memo_.end()) return it->second[j];
        std::vector<BV> y;
        switch (n.kind) {
        case SG_K_INTO_BITS: {
            Ref ri = R_.resolve(n.in[0], Lin::k(g * n.pop));
            if (ri.k != Ref::PHYS || ri.edge != ein_) throw Error(SG_E_UNSUPPORTED, "bitslice: INTO_BITS must read the boundary input");
            const int64_t c = ri.pos.c - off_in_;
            if (c < 0 || c >= PIN_) throw Error(SG_E_UNSUPPORTED, "bitslice: input column out of range");
            used_cols_.insert(c);
            for (int b = 0; b < 32; b++) y.push_back({"w" + std::to_string(c) + "[" + std::to_string(31 - b) + "]", false});
            break;
        }
        case SG_K_XOR: {
            const int64_t nn = n.iv[0];
            std::vector<BV> x(2 * nn);
            for (int64_t i = 0; i < 2 * nn; i++) x[i] = bit(n.in[0], g * n.pop + i);
            for (int64_t i = 0; i < nn; i++) {
                BV a = x[i], b = x[nn + i];
                if (a.s == "0u") { y.push_back({b.s, (bool)(b.neg ^ a.neg)}); continue; }
                if (b.s == "0u") { y.push_back({a.s, (bool)(a.neg ^ b.neg)}); continue; }
                BV r = fresh(a.s + " ^ " + b.s);
                r.neg = a.neg ^ b.neg;
                y.push_back(r);
            }
            break;
        }
        case SG_K_XOR_CONST: {
            auto ks = keyslot_.find(u);
            for (int64_t i = 0; i < n.iv[0]; i++) {
                BV a = bit(n.in[0], g * n.pop + i);
                if (ks != keyslot_.end()) {  // rolled loop: this round's key bit (0 or ~0) from the key table
                    BV r = fresh(a.s + " ^ kt[" + std::to_string(ks->second + i) + "]");
                    r.neg = a.neg;
                    y.push_back(r);
                    continue;
                }
                if (n.iv[1 + i] & 1) a.neg = !a.neg;
                y.push_back(a);
            }
            break;
        }
        case SG_K_SBOX: {
            std::vector<BV> x(6);
            for (int i = 0; i < 6; i++) x[i] = bit(n.in[0], g * n.pop + i);
            y = sbox(x, n.iv);
            break;
        }
        default:
            throw Error(SG_E_UNSUPPORTED, std::string("bitslice: ") + kind_name(n.kind) + " output used as a bit");
        }
        memo_[key] = y;
        return y[j];
    }
};

// ------------------------------------------------------------ feedback loops
// A feedback loop carries state from one iteration to the next, so its partition
// runs sequentially: one thread executes the loop graph's static schedule firing by firing (found
// at plan time, sg_graph.cpp go_loop), its internal FIFOs in shared memory (absolute stream
// positions, power-of-two rings), the outer input read and the outer output written in natural
// order.  Between launches (fragments) the FIFOs, the next firing index and a history of the last
// `halo` firings' outputs (re-emitted when a downstream peek window reaches back) live in a plan-
// owned state buffer, reset to the enqueued items at the start of every sg_run.
class LoopGen : public GenBase {
public:
    LoopGen(const Flat& outer, int v, int part) : GenBase(*outer.nodes[v].loop->sub, all_nodes(*outer.nodes[v].loop->sub), part),
                                                  of_(outer), v_(v), li_(*outer.nodes[v].loop) {}

    static std::vector<int> all_nodes(const Flat& f) {
        std::vector<int> a(f.nodes.size());
        std::iota(a.begin(), a.end(), 0);
        return a;
    }
    // Wavefront width: firing g reads an item of edge e written by firing g' <= g - floor(init_e / T_e)
    // (init_e = items queued at the stream start: enqueued items, DELAY prework), so the firings of any
    // window of W = min_e floor(init_e / T_e) consecutive firings are independent and run on W lanes.
    static int64_t wavefront(const LoopInfo& li) {
        const Flat& sf = *li.sub;
        int64_t W = 256;
        for (int e = 0; e < (int)sf.edges.size(); e++)
            if (li.init_level[e] > 0) W = std::min<int64_t>(W, li.init_level[e] / std::max<int64_t>(1, sf.edges[e].per_iter));
        return std::max<int64_t>(1, W);
    }
    // ring capacity of edge e when W firings are in flight: W * T_e beyond the simulated maximum
    static std::vector<int64_t> capacities(const LoopInfo& li, int64_t W) {
        const Flat& sf = *li.sub;
        std::vector<int64_t> cap(sf.edges.size(), 0);
        for (int e = 0; e < (int)sf.edges.size(); e++) {
            int64_t c = 1;
            while (c < li.cap[e] + (W - 1) * sf.edges[e].per_iter) c <<= 1;
            cap[e] = c;
        }
        return cap;
    }
    // state image layout (4-byte words): [0,2) next firing (int64), then each internal edge's ring, then history
    static std::vector<uint32_t> initial_state(const LoopInfo& li, const std::vector<int64_t>& cap, int64_t& hist_off,
                                               int64_t& hist_len, int64_t hist_items, std::vector<int64_t>& ring_off) {
        const Flat& sf = *li.sub;
        int64_t o = 2;
        ring_off.assign(sf.edges.size(), -1);
        for (int e = 0; e < (int)sf.edges.size(); e++) {
            if (e == sf.in_edge || e == sf.out_edge) continue;
            ring_off[e] = o;
            o += cap[e];
        }
        hist_off = o;
        hist_len = 1;
        while (hist_len < std::max<int64_t>(1, hist_items)) hist_len <<= 1;
        o += hist_len;
        std::vector<uint32_t> img((size_t)o, 0u);
        for (size_t k = 0; k < li.enq.size(); k++) img[ring_off[li.back] + (k & (cap[li.back] - 1))] = li.enq[k];
        return img;  // DELAY prework items are zeros (already 0)
    }

    KernelInfo run() {
        const Node& ln = of_.nodes[v_];
        const Flat& sf = *li_.sub;
        KernelInfo ki;
        ki.mode = 4;
        ki.name = "sg_part" + std::to_string(part_);
        ki.name_sync = ki.name;
        ki.tile = ki.tile_sync = 1 << 30;  // one CTA
        ki.in_edges = {ln.in[0]};
        ki.out_edges = {ln.out[0]};
        int64_t lo, ex;
        edge_window(of_, ln.in[0], lo, ex);
        ki.in_lo = {lo};
        ki.in_extra = {ex};
        edge_window(of_, ln.out[0], lo, ex);
        ki.out_lo = {lo};
        ki.out_extra = {ex};
        const int64_t OLO = lo, OEX = ex, OPI = of_.edges[ln.out[0]].per_iter;
        for (int u = 0; u < (int)sf.nodes.size(); u++) {
            int64_t a, b, c;
            node_work(sf, u, a, b, c);
            ki.flops_per_iter += a * ln.rep;
            ki.intops_per_iter += b * ln.rep;
            ki.dfma_per_iter += c * ln.rep;
        }
        int64_t W = wavefront(li_);
        if (const char* e = std::getenv("SG_LOOP_WAVEFRONT")) W = std::max<int64_t>(1, std::min<int64_t>(W, std::atoll(e)));
        std::vector<int64_t> cap;
        int64_t smem_words = 0;
        for (;; W = (W + 1) / 2) {  // shrink the wavefront until the rings fit in shared memory
            cap = capacities(li_, W);
            smem_words = 0;
            for (int e = 0; e < (int)sf.edges.size(); e++)
                if (e != sf.in_edge && e != sf.out_edge) smem_words += cap[e];
            if (smem_words * 4 <= 160 * 1024 || W == 1) break;
        }
        if (smem_words * 4 > 200 * 1024) throw Error(SG_E_SIZE, "feedback loop FIFOs exceed shared memory");
        const int NT = (int)std::min<int64_t>(256, (W + 31) / 32 * 32);
        const int64_t WB = std::min<int64_t>(W, NT);  // firings per wavefront step
        ki.threads = ki.threads_sync = NT;
        int64_t hist_off, hist_len;
        std::vector<int64_t> roff;
        auto img = initial_state(li_, cap, hist_off, hist_len, (ln.halo + WB) * li_.Q, roff);
        ki.state_words = (int64_t)img.size();
        ki.state_init = img;
        std::vector<int64_t> soff(sf.edges.size(), -1);
        int64_t so = 0;
        for (int e = 0; e < (int)sf.edges.size(); e++)
            if (roff[e] >= 0) { soff[e] = so; so += cap[e]; }
        ki.smem = (size_t)std::max<int64_t>(4, smem_words * 4);
        ki.smem_sync = ki.smem;
        // one firing of the loop = the static schedule with compile-time offsets
        std::ostringstream body;
        std::vector<int64_t> rd(sf.edges.size(), 0), wr(sf.edges.size(), 0);
        for (int e = 0; e < (int)sf.edges.size(); e++) wr[e] = li_.init_level[e];
        const std::string T = T_;
        // lane-local chains: if every queued edge holds exactly one step of items (init_e == WB * T_e), a
        // firing's cross-firing inputs come from the firing WB earlier -- the same lane, one step back
        // A slot of a ring (or of the history) is then only ever written by one lane iff its length is a
        // multiple of the items one step writes (WB * T_e; history: WB * Q) -- otherwise lanes of different
        // warps share slots and, with no barrier, a lagging warp could leave an older value in the saved
        // state, so such loops keep the per-step barrier.
        bool lane_local = !std::getenv("SG_LOOP_BARRIER");
        for (int e = 0; e < (int)sf.edges.size(); e++) {
            if (li_.init_level[e] > 0 && li_.init_level[e] != WB * sf.edges[e].per_iter) lane_local = false;
            if (roff[e] >= 0 && cap[e] % (WB * std::max<int64_t>(1, sf.edges[e].per_iter)) != 0) lane_local = false;
        }
        if (hist_len % (WB * std::max<int64_t>(1, li_.Q)) != 0) lane_local = false;
        // ... and then every item a firing reads is in a register: written earlier in the same firing
        // (edges without initial items) or carried from the lane's previous firing (queued edges, loaded
        // from the ring once, at the lane's first firing of the launch).  The rings of queued edges are
        // still written, so the state saved after the launch is exact.
        const bool fwd = lane_local && !std::getenv("SG_LOOP_NO_FWD");
        std::ostringstream decl, carry_in, carry_out;
        auto lv = [&](int e, int64_t c) { return "lv" + std::to_string(e) + "_" + std::to_string(c); };
        auto cr = [&](int e, int64_t c) { return "cr" + std::to_string(e) + "_" + std::to_string(c); };
        auto pos_ref = [&](int e, int64_t c) -> std::string {  // item at (firing-relative) position c of edge e
            const int64_t per = sf.edges[e].per_iter;
            if (e == sf.in_edge) return "cur[" + std::to_string(c) + "]";  // prefetched one wavefront step ahead
            return "q[" + std::to_string(soff[e]) + " + (int)((g * " + std::to_string(per) + "LL + " + std::to_string(c) +
                   "LL) & " + std::to_string(cap[e] - 1) + "LL)]";
        };
        for (int u : li_.sched) {
            const Node& n = sf.nodes[u];
            std::vector<std::string> xs;
            for (int e : n.in) {
                for (int64_t i = 0; i < sf.edges[e].pop; i++) {
                    const int64_t c = rd[e] + i;
                    if (!fwd || e == sf.in_edge) xs.push_back(pos_ref(e, c));
                    else xs.push_back(li_.init_level[e] > 0 ? cr(e, c) : lv(e, c));
                }
                rd[e] += sf.edges[e].pop;
            }
            std::vector<std::string> ys;  // per output item, in port order
            body << "        {\n";
            if (n.type == N_FILTER) {
                body << "          const " << T << " x_[" << std::max<size_t>(1, xs.size()) << "] = {";
                for (size_t i = 0; i < xs.size(); i++) body << (i ? ", " : "") << xs[i];
                body << "};\n          " << T << " y_[" << n.push << "];\n          ";
                body << firing_code(u) << "\n";
                for (int64_t j = 0; j < n.push; j++) ys.push_back("y_[" + std::to_string(j) + "]");
            } else {
                // splitters / joiners: pure data movement
                body << "          const " << T << " x_[" << xs.size() << "] = {";
                for (size_t i = 0; i < xs.size(); i++) body << (i ? ", " : "") << xs[i];
                body << "};\n";
                if (n.type == N_SPLIT_DUP) {
                    for (size_t k = 0; k < n.out.size(); k++) ys.push_back("x_[0]");
                } else {
                    for (size_t i = 0; i < xs.size(); i++) ys.push_back("x_[" + std::to_string(i) + "]");
                }
            }
            // pushes: splitter RR sends consecutive items per port; DUP sends x_[0] to every port
            size_t yi = 0;
            for (size_t k = 0; k < n.out.size(); k++) {
                const int e = n.out[k];
                for (int64_t j = 0; j < sf.edges[e].push; j++, yi++) {
                    const std::string val = n.type == N_SPLIT_DUP ? ys[k] : ys[yi];
                    if (e == sf.out_edge) {
                        const int64_t c = wr[e] + j;  // output item c of this firing
                        body << "          { const long long p = g * " << li_.Q << "LL + " << c << "LL; const " << T
                             << " val = " << val << ";\n            hist[(int)(p & " << hist_len - 1 << "LL)] = val;\n"
                             << "            if (p >= wlo && p < whi) gout[p - out_base] = val; }\n";
                    } else if (!fwd) {
                        body << "          " << pos_ref(e, wr[e] + j) << " = " << val << ";\n";
                    } else {
                        decl << "        " << T << " " << lv(e, wr[e] + j) << ";\n";
                        body << "          " << lv(e, wr[e] + j) << " = " << val << ";\n";
                        if (li_.init_level[e] > 0)
                            body << "          " << pos_ref(e, wr[e] + j) << " = " << lv(e, wr[e] + j) << ";\n";
                    }
                }
                wr[e] += sf.edges[e].push;
            }
            body << "        }\n";
        }
        std::ostringstream carry_decl;
        if (fwd)
            for (int e = 0; e < (int)sf.edges.size(); e++) {
                if (li_.init_level[e] == 0 || e == sf.in_edge || e == sf.out_edge) continue;
                const int64_t per = sf.edges[e].per_iter;
                for (int64_t c = 0; c < per; c++) {
                    carry_decl << "  " << T << " " << cr(e, c) << " = (" << T << ")0;\n";
                    carry_in << "          " << cr(e, c) << " = " << pos_ref(e, c) << ";\n";
                    carry_out << "        " << cr(e, c) << " = " << lv(e, WB * per + c) << ";\n";
                }
            }
        // Interior trips (every firing of the PD steps fires, prefetches in range, outputs inside the
        // launch window, carries in registers): one straight-line block of PD steps with no per-step
        // guards, so the address and store work of later steps overlaps the serial chain.
        // PD: prefetch distance = steps per unrolled trip.  Measured on echo64 (B200, iters/s): PD 8
        // 6.2e8, 16 9.8e8, 32 1.36e9, 64 1.78e9, 128 1.89e9.  Capped so the prefetch slots stay within
        // 128 registers and the unrolled trip within ~2048 firings.
        // registers: PD * P prefetch slots <= 128 (no floor: more would spill to local memory);
        // code size: the fast and the guarded trip are both unrolled PD steps, 2 * PD * |schedule| <= ~4096
        // firings of straight-line code
        int64_t PD = 128;
        PD = std::min<int64_t>(PD, std::max<int64_t>(1, 128 / std::max<int64_t>(1, li_.P)));
        PD = std::min<int64_t>(PD, std::max<int64_t>(1, 2048 / std::max<int64_t>(1, (int64_t)li_.sched.size())));
        if (const char* e = std::getenv("SG_LOOP_PD")) PD = std::max(1, std::atoi(e));
        std::string fast_trip;
        if (fwd && WB == NT) {
            std::string fb = body.str();
            const std::string guard = "if (p >= wlo && p < whi) ";
            for (size_t k; (k = fb.find(guard)) != std::string::npos;) fb.erase(k, guard.size());
            std::ostringstream ft;
            ft << "    if (gs >= next0 && gs + 2LL * PD * " << WB << " <= g1 && gs * " << li_.Q << "LL >= wlo && (gs + (long long)PD * "
               << WB << ") * " << li_.Q << "LL <= whi) {\n"
               << "      if (!fired) {\n        const long long g = gs + threadIdx.x;\n" << carry_in.str()
               << "          fired = true;\n      }\n"
               << "#pragma unroll\n"
               << "      for (int sd = 0; sd < PD; sd++) {\n"
               << "        const long long g = gs + (long long)sd * " << WB << " + threadIdx.x;\n"
               << "        " << T << " cur[" << li_.P << "];\n"
               << "        for (int c = 0; c < " << li_.P << "; c++) cur[c] = pf[sd][c];\n"
               << "        for (int c = 0; c < " << li_.P << "; c++) pf[sd][c] = gin[(g + (long long)PD * " << WB << ") * " << li_.P
               << "LL + c - in_base];\n"
               << decl.str() << fb << carry_out.str()
               << "      }\n"
               << "      continue;\n"
               << "    }\n";
            fast_trip = ft.str();
        }
        std::ostringstream s;
        s << header("feedback loop") << consts_.str() << args_struct_loop();
        s << "// wavefront: " << WB << " independent firings per step (loop delay " << wavefront(li_) << " firings)\n"
          << "extern \"C\" __global__ void __launch_bounds__(" << NT << ", 1) " << ki.name << "(const SgArgs a) {\n"
          << "  extern __shared__ __align__(16) unsigned char sg_smem[];\n"
          << "  " << T << "* q = reinterpret_cast<" << T << "*>(sg_smem);\n"
          << "  " << T << "* st = reinterpret_cast<" << T << "*>(SG_STATE);\n";
        for (int e = 0; e < (int)sf.edges.size(); e++)
            if (roff[e] >= 0)
                s << "  for (int i = threadIdx.x; i < " << cap[e] << "; i += " << NT << ") q[" << soff[e] << " + i] = st["
                  << roff[e] << " + i];\n";
        s << "  const long long next0 = *reinterpret_cast<const long long*>(st);\n"
          << "  __syncthreads();\n"
          << "  " << T << "* hist = st + " << hist_off << ";\n"
          << "  const " << T << "* gin = SG_IN(0);\n"
          << "  const long long in_base = SG_IN_BASE(0);\n"
          << "  " << T << "* gout = SG_OUT(0);\n"
          << "  const long long out_base = SG_OUT_BASE(0);\n"
          << "  const long long wlo = SG_K_BEGIN * " << OPI << "LL + (" << OLO << "LL);\n"
          << "  const long long whi = SG_K_END * " << OPI << "LL + (" << OLO + OEX << "LL);\n"
          << "  const long long g0 = SG_K_BEGIN * " << ln.rep << "LL + (" << ln.ninit - ln.halo << "LL);\n"
          << "  const long long g1 = SG_K_END * " << ln.rep << "LL + (" << ln.ninit << "LL);\n"
          << "  // the outer input of each lane's firings is loaded PD wavefront steps ahead (global latency\n"
          << "  // off the serial chain: a step is a few shared-memory round trips)\n"
          << "  constexpr int PD = " << PD << ";\n"
          << carry_decl.str() << (fwd ? "  bool fired = false;  // this lane's carries are in registers\n" : "")
          << "  " << T << " pf[PD][" << li_.P << "];\n"
          << "#pragma unroll\n"
          << "  for (int d = 0; d < PD; d++) {\n"
          << "    const long long g = g0 + (long long)d * " << WB << " + threadIdx.x;\n"
          << "    if (threadIdx.x < " << WB << " && g < g1 && g >= next0)\n"
          << "      for (int c = 0; c < " << li_.P << "; c++) pf[d][c] = gin[g * " << li_.P << "LL + c - in_base];\n"
          << "  }\n"
          << "  // PD steps per outer trip, unrolled: slot d is consumed and refilled at step d, so no\n"
          << "  // register rotation ever waits on a load still in flight\n"
          << "  for (long long gs = g0; gs < g1; gs += (long long)PD * " << WB << ") {\n"
          << fast_trip
          << "#pragma unroll\n"
          << "   for (int sd = 0; sd < PD; sd++) {\n"
          << "    const long long gb = gs + (long long)sd * " << WB << ";\n"
          << "    const long long g = gb + threadIdx.x;\n"
          << "    " << T << " cur[" << li_.P << "];\n"
          << "    for (int c = 0; c < " << li_.P << "; c++) cur[c] = pf[sd][c];\n"
          << "    {\n"
          << "      const long long gn = g + (long long)PD * " << WB << ";\n"
          << "      if (threadIdx.x < " << WB << " && gn < g1 && gn >= next0)\n"
          << "        for (int c = 0; c < " << li_.P << "; c++) pf[sd][c] = gin[gn * " << li_.P << "LL + c - in_base];\n"
          << "    }\n"
          << "    if (threadIdx.x < " << WB << " && g < g1) {\n"
          << "      if (g < next0) {  // before the stream start (zeros) or computed by an earlier launch (history)\n"
          << "        for (int j = 0; j < " << li_.Q << "; j++) {\n"
          << "          const long long p = g * " << li_.Q << "LL + j;\n"
          << "          if (p >= wlo && p < whi) gout[p - out_base] = g < 0 ? (" << T << ")0 : hist[(int)(p & " << hist_len - 1
          << "LL)];\n"
          << "        }\n"
          << "      } else {\n"
          << (fwd ? "        if (!fired) {\n" + carry_in.str() + "          fired = true;\n        }\n" : std::string())
          << decl.str()
          << body.str()
          << carry_out.str()
          << "      }\n"
          << "    }\n"
          << (lane_local ? "    // every cross-firing dependency is exactly one step back on the same lane: no barrier\n"
                         : "    __syncthreads();\n")
          << "   }\n"
          << "  }\n"
          << (lane_local ? "  __syncthreads();\n" : "")
          << "  if (threadIdx.x == 0) *reinterpret_cast<long long*>(st) = next0 > g1 ? next0 : g1;\n";
        for (int e = 0; e < (int)sf.edges.size(); e++)
            if (roff[e] >= 0)
                s << "  for (int i = threadIdx.x; i < " << cap[e] << "; i += " << NT << ") st[" << roff[e] << " + i] = q["
                  << soff[e] << " + i];\n";
        s << "}\n";
        ki.source = s.str();
        return ki;
    }

private:
    const Flat& of_;
    int v_;
    const LoopInfo& li_;

    std::string args_struct_loop() {
        // one boundary input and output (the outer edges), plus the state pointer
        std::ostringstream s;
        s << "struct SgArgs { long long v[8]; };\n"
          << "#define SG_IN(i) (reinterpret_cast<const " << T_ << "*>(a.v[0]))\n"
          << "#define SG_IN_BASE(i) (a.v[1])\n"
          << "#define SG_IN_LIMIT(i) (a.v[2])\n"
          << "#define SG_OUT(i) (reinterpret_cast<" << T_ << "*>(a.v[3]))\n"
          << "#define SG_OUT_BASE(i) (a.v[4])\n"
          << "#define SG_K_BEGIN (a.v[5])\n"
          << "#define SG_K_END (a.v[6])\n"
          << "#define SG_STATE (reinterpret_cast<void*>(a.v[7]))\n";
        return s.str();
    }
    // one firing of filter u of the loop graph: x_ -> y_ (compute kinds via work_call; data-movement kinds inline)
    std::string firing_code(int u) {
        const Node& n = f_.nodes[u];
        std::ostringstream c;
        switch (n.kind) {
        case SG_K_IDENTITY: case SG_K_DELAY: case SG_K_DECIMATE: c << "y_[0] = x_[0];"; break;
        case SG_K_EXPAND:
            c << "y_[0] = x_[0];";
            for (int64_t j = 1; j < n.push; j++) c << " y_[" << j << "] = (" << T_ << ")0;";
            break;
        case SG_K_FFT_REORDER: {
            int64_t nn = n.iv[0], o = 0;
            for (int64_t i = 0; i < nn; i += 2, o += 2) c << "y_[" << o << "] = x_[" << 2 * i << "]; y_[" << o + 1 << "] = x_[" << 2 * i + 1 << "]; ";
            for (int64_t i = 1; i < nn; i += 2, o += 2) c << "y_[" << o << "] = x_[" << 2 * i << "]; y_[" << o + 1 << "] = x_[" << 2 * i + 1 << "]; ";
            break;
        }
        case SG_K_PERMUTE:
            for (size_t k = 1; k < n.iv.size(); k++) c << "y_[" << k - 1 << "] = x_[" << n.iv[k] << "]; ";
            break;
        default: c << work_call(u);
        }
        return c.str();
    }
};

// --------------------------------------------------------------- gather mode
// A partition of views only (splitters, joiners, IDENTITY / DELAY / DECIMATE / EXPAND / PERMUTE /
// FFT_REORDER; e.g. the transposing join of a 2-D DCT, a joiner + duplicate splitter between the channel
// and beam halves of BeamFormer) computes nothing: every output position is one input position (or a
// zero).  Such a kernel is a straight global-to-global gather -- a grid-stride loop over the output
// window, each position resolved through the views by generated index arithmetic (64-bit positions,
// floor division), no tiles, no shared memory.  Positions outside an input's window (the stream start,
// prework) read as zero, exactly what the producer's firings g < 0 emit.
class GatherGen : public GenBase {
public:
    using GenBase::GenBase;

    KernelInfo run() {
        KernelInfo ki;
        ki.mode = 5;
        ki.name = "sg_part" + std::to_string(part_);
        ki.name_sync = ki.name;
        fill_io(ki);
        ki.threads = ki.threads_sync = 256;
        // iterations per grid-stride unit (grid sizing only): ~16k output items each, so a launch gets
        // enough CTAs to fill the GPU whatever the iteration size (BeamFormer: 49 152 items per frame)
        int64_t items = 0;
        for (int e : outs_) items += f_.edges[e].per_iter;
        ki.tile = ki.tile_sync = (int)std::max<int64_t>(1, std::min<int64_t>(64, 16384 / std::max<int64_t>(1, items)));
        ki.smem = ki.smem_sync = 0;
        ki.min_blocks = 1;
        for (int e : outs_) reader(e);
        std::ostringstream src;
        src << header("gather") << consts_.str() << args_struct();
        src << "__device__ __forceinline__ long long sg_fdiv64(long long a, long long b) {\n"
            << "  const long long q = a / b; return (a % b != 0 && ((a < 0) != (b < 0))) ? q - 1 : q;\n}\n";
        for (auto& r : order_) src << body_.at(r);
        src << "extern \"C\" __global__ void __launch_bounds__(256) " << ki.name << "(const SgArgs a) {\n"
            << "  const long long step = (long long)gridDim.x * 256;\n";
        for (size_t oi = 0; oi < outs_.size(); oi++) {
            const int e = outs_[oi];
            const Edge& ed = f_.edges[e];
            if (emit_periodic(src, oi, e, ki)) continue;
            src << "  { // boundary output " << oi << " (edge " << e << ")\n"
                << "    " << T_ << "* g = SG_OUT(" << oi << ");\n"
                << "    const long long ob = SG_OUT_BASE(" << oi << ");\n"
                << "    const long long p0 = SG_K_BEGIN * " << ed.per_iter << "LL + (" << ki.out_lo[oi] << "LL);\n"
                << "    const long long p1 = SG_K_END * " << ed.per_iter << "LL + (" << ki.out_lo[oi] + ki.out_extra[oi]
                << "LL);\n"
                << "    // four positions per trip, loads first: four gathers in flight per thread\n"
                << "    for (long long p = p0 + (long long)blockIdx.x * 256 + threadIdx.x; p < p1; p += 4 * step) {\n"
                << "      " << T_ << " v[4];\n"
                << "#pragma unroll\n"
                << "      for (int u = 0; u < 4; u++) { const long long q = p + u * step; v[u] = q < p1 ? " << name(e)
                << "(a, q) : (" << T_ << ")0; }\n"
                << "#pragma unroll\n"
                << "      for (int u = 0; u < 4; u++) { const long long q = p + u * step; if (q < p1) g[q - ob] = v[u]; }\n"
                << "    }\n"
                << "  }\n";
        }
        src << "}\n";
        ki.source = src.str();
        return ki;
    }

private:
    std::map<int, std::string> body_;
    std::vector<int> order_;  // callees first
    std::string name(int e) { return "sg_rdg" + std::to_string(e); }

    // Periodic form: the smallest period P (dividing the output's items per iteration, <= 32) for which
    // output position k*P + c resolves, for every residue c, to an affine position a_c*k + b_c of one
    // boundary input (or to a zero): each thread then copies one whole period with compile-time maps --
    // no per-item division or branch chain.  Longer periods keep the generic form: a thread copying a whole
    // period of P items makes a warp's accesses P items apart (uncoalesced), while the generic loop maps
    // consecutive threads to consecutive output positions.  Returns false when no such period exists.
    bool emit_periodic(std::ostringstream& src, size_t oi, int e, const KernelInfo& ki) {
        const int64_t per = f_.edges[e].per_iter;
        for (int64_t P = 1; P <= std::min<int64_t>(per, 32); P++) {
            if (per % P) continue;
            struct M { int in = -1; int64_t a = 0, b = 0; };
            std::vector<M> maps(P);
            bool ok = true;
            for (int64_t c = 0; c < P && ok; c++) {
                Ref r = R_.resolve(e, Lin::v("k", P, c));
                if (r.k == Ref::ZERO) continue;
                if (r.k == Ref::RUNTIME) { ok = false; break; }
                const int i = (int)(std::find(ins_.begin(), ins_.end(), r.edge) - ins_.begin());
                if (i >= (int)ins_.size()) { ok = false; break; }
                for (auto& t : r.pos.t) if (t.first != "k") ok = false;
                maps[c].in = i;
                maps[c].a = r.pos.coef("k");
                maps[c].b = r.pos.c;
            }
            if (!ok) continue;
            src << "  { // boundary output " << oi << " (edge " << e << "): period " << P << ", affine per residue\n"
                << "    " << T_ << "* g = SG_OUT(" << oi << ");\n"
                << "    const long long ob = SG_OUT_BASE(" << oi << ");\n"
                << "    const long long p0 = SG_K_BEGIN * " << per << "LL + (" << ki.out_lo[oi] << "LL);\n"
                << "    const long long p1 = SG_K_END * " << per << "LL + (" << ki.out_lo[oi] + ki.out_extra[oi] << "LL);\n"
                << "    const long long kb = sg_fdiv64(p0, " << P << "LL), ke = sg_fdiv64(p1 + " << P - 1 << "LL, " << P << "LL);\n"
                << "    for (long long k = kb + (long long)blockIdx.x * 256 + threadIdx.x; k < ke; k += step) {\n"
                << "      const long long pb = k * " << P << "LL;\n";
            for (int64_t c = 0; c < P; c++) {
                const M& m = maps[c];
                if (m.in < 0) { src << "      const " << T_ << " v" << c << " = (" << T_ << ")0;\n"; continue; }
                src << "      " << T_ << " v" << c << ";\n"
                    << "      { const long long q = " << m.a << "LL * k + (" << m.b << "LL) - SG_IN_BASE(" << m.in << ");\n"
                    << "        v" << c << " = (q >= 0 && q < SG_IN_LIMIT(" << m.in << ")) ? SG_IN(" << m.in << ")[q] : (" << T_
                    << ")0; }\n";
            }
            for (int64_t c = 0; c < P; c++)
                src << "      if (pb + " << c << " >= p0 && pb + " << c << " < p1) g[pb + " << c << " - ob] = v" << c << ";\n";
            src << "    }\n  }\n";
            return true;
        }
        return false;
    }

    void reader(int e) {
        if (body_.count(e)) return;
        body_[e] = "";
        std::ostringstream s;
        s << "__device__ __forceinline__ " << T_ << " " << name(e) << "(const SgArgs& a, long long p) {\n";
        const Edge& ed = f_.edges[e];
        const int i = (int)(std::find(ins_.begin(), ins_.end(), e) - ins_.begin());
        std::vector<int> deps;
        if (i < (int)ins_.size()) {  // a boundary input: its window, zero outside
            s << "  const long long q = p - SG_IN_BASE(" << i << ");\n"
              << "  return (q >= 0 && q < SG_IN_LIMIT(" << i << ")) ? SG_IN(" << i << ")[q] : (" << T_ << ")0;\n";
        } else {
            const Node& u = f_.nodes[ed.src];
            switch (u.type) {
            case N_SPLIT_DUP: s << "  return " << name(u.in[0]) << "(a, p);\n"; deps.push_back(u.in[0]); break;
            case N_SPLIT_RR: {
                int64_t w = u.w[ed.sport], P = 0;
                for (int k = 0; k < ed.sport; k++) P += u.w[k];
                s << "  const long long q = sg_fdiv64(p, " << w << "LL), r = p - q * " << w << "LL;\n"
                  << "  return " << name(u.in[0]) << "(a, q * " << u.wsum << "LL + " << P << "LL + r);\n";
                deps.push_back(u.in[0]);
                break;
            }
            case N_JOIN: {
                s << "  const long long q = sg_fdiv64(p, " << u.wsum << "LL), o = p - q * " << u.wsum << "LL;\n";
                int64_t P = 0;
                for (size_t b = 0; b < u.w.size(); b++) {
                    s << "  if (o < " << P + u.w[b] << "LL) return " << name(u.in[b]) << "(a, q * " << u.w[b] << "LL + o - "
                      << P << "LL);\n";
                    deps.push_back(u.in[b]);
                    P += u.w[b];
                }
                s << "  return (" << T_ << ")0;\n";
                break;
            }
            case N_FILTER: {
                const int in = u.in[0];
                deps.push_back(in);
                switch (u.kind) {
                case SG_K_IDENTITY: s << "  return " << name(in) << "(a, p);\n"; break;
                case SG_K_DELAY: s << "  return " << name(in) << "(a, p - " << u.iv[0] << "LL);\n"; break;
                case SG_K_DECIMATE: s << "  return " << name(in) << "(a, p * " << u.iv[0] << "LL);\n"; break;
                case SG_K_EXPAND:
                    s << "  const long long q = sg_fdiv64(p, " << u.iv[0] << "LL);\n  return (p - q * " << u.iv[0]
                      << "LL) == 0 ? " << name(in) << "(a, q) : (" << T_ << ")0;\n";
                    break;
                case SG_K_PERMUTE: {
                    const int64_t n = u.iv[0], m = (int64_t)u.iv.size() - 1;
                    const std::string tab = "SG_GP" + std::to_string(e);
                    consts_ << "__constant__ int " << tab << "[" << m << "] = {";
                    for (int64_t k = 0; k < m; k++) consts_ << (k ? "," : "") << (k % 16 == 0 ? "\n  " : "") << u.iv[1 + k];
                    consts_ << "};\n";
                    s << "  const long long q = sg_fdiv64(p, " << m << "LL), o = p - q * " << m << "LL;\n"
                      << "  return " << name(in) << "(a, q * " << n << "LL + " << tab << "[o]);\n";
                    break;
                }
                case SG_K_FFT_REORDER: {
                    const int64_t n = u.iv[0], F = 2 * n;
                    s << "  const long long q = sg_fdiv64(p, " << F << "LL), o = p - q * " << F << "LL;\n"
                      << "  const long long m = o >> 1, r = o & 1;\n"
                      << "  const long long sc = m < " << n / 2 << " ? 2 * m : 2 * (m - " << n / 2 << ") + 1;\n"
                      << "  return " << name(in) << "(a, q * " << F << "LL + 2 * sc + r);\n";
                    break;
                }
                default: throw Error(SG_E_UNSUPPORTED, "internal: gather through a compute filter");
                }
                break;
            }
            default: throw Error(SG_E_UNSUPPORTED, "internal: gather through a feedback loop");
            }
        }
        s << "}\n";
        for (int d : deps) reader(d);  // callees first
        body_[e] = s.str();
        order_.push_back(e);
    }
};

// -------------------------------------------------------------- staged mode
class StageGen : public GenBase {
public:
    using GenBase::GenBase;

    KernelInfo run(const CodegenOpts& opt) {
        KernelInfo ki;
        ki.mode = 2;
        ki.name = "sg_part" + std::to_string(part_);
        fill_io(ki);
        compute_levels();
        int NT = opt.threads > 0 ? opt.threads : 256;
        NT_ = NT;
        // ---------------- fused fast path (full tiles without stream-start firings)
        std::string fast, fast_start, prologue_fast;
        int WF = 0;
        size_t smem_fast = 0;
        if (opt.mode != -2) {
            try {
                fused_ = true;
                fused_analyze();
                size_t fb = opt.smem_budget > 0 ? (size_t)opt.smem_budget
                                                : (size_t)((opt.tile > 0 ? 227 : 110) * 1024);  // a forced tile may use it all
                for (int cand : fused_tile_candidates(opt.tile)) {
                    fused_layout(cand);
                    if (smem_bytes_ <= fb) { WF = cand; break; }
                }
                if (WF == 0) {
                    fused_layout(1);
                    if (smem_bytes_ <= 227 * 1024) WF = 1;
                }
                if (WF > 0 && opt.threads <= 0) {
                    fused_layout(WF);
                    if (smem_bytes_ > 113 * 1024) {  // one CTA per SM: give it 16 warps (32 for frame
                        // FIR partitions: their blocks fit 64 registers and the extra warps hide the
                        // shared-memory latency of the sample windows; BeamFormer 2.69 -> 2.57 ms)
                        bool frame = false;
                        for (auto& g : fg_) frame = frame || g.special;
                        // (opt-in FFMA2 frame FIRs, SG_FFMA2=1, need the 128 registers of 512-thread
                        // CTAs; measured slower: BeamFormer 2.88 ms vs 2.56 ms scalar at 1024 threads)
                        // (the sliding-window frame FIRs hold R-sample windows per plane: 512 threads)
                        NT_ = NT = (frame && !std::getenv("SG_FFMA2") && !beam_slide_on()) ? 1024 : 512;
                        int W2 = 0;
                        for (int cand : fused_tile_candidates(opt.tile)) {
                            fused_layout(cand);
                            if (smem_bytes_ <= 227 * 1024) { W2 = cand; break; }
                        }
                        if (W2 > 0) WF = W2;
                    }
                }
                if (WF > 0) {
                    fused_layout(WF);
                    // inputs: prefetch the next tile into a staging region with cp.async while
                    // this tile computes, if it fits at the same CTAs per SM; else issue every
                    // load of the tile asynchronously at its start (one wait instead of a
                    // round trip per load)
                    {
                        int64_t st = 0;
                        for (int e : ins_) {
                            int64_t lo, ex;
                            edge_window(f_, e, lo, ex);
                            st += (f_.edges[e].per_iter * WF + ex + 3) / 4 * 4 + 4;
                        }
                        auto blocks = [](size_t b) { return std::max(1, std::min(2, (int)((220 * 1024) / std::max<size_t>(1024, b)))); };
                        size_t with = smem_bytes_ + (size_t)st * 4;
                        prefetch_ = !ins_.empty() && !std::getenv("SG_NO_PREFETCH") && with <= 227 * 1024 &&
                                    blocks(with) == blocks(smem_bytes_);
                        if (prefetch_) {
                            int64_t o = (int64_t)(smem_bytes_ / 4 + 3) / 4 * 4;
                            stage_off_.clear();
                            for (int e : ins_) {
                                int64_t lo, ex;
                                edge_window(f_, e, lo, ex);
                                stage_off_[e] = o;
                                o += (f_.edges[e].per_iter * WF + ex + 3) / 4 * 4 + 4;
                            }
                            smem_bytes_ = (size_t)o * 4;
                        }
                    }
                    smem_fast = smem_bytes_;
                    fast = fused_emit(WF, false);
                    fast_start = fused_emit(WF, true);
                    prologue_fast = prologue_;
                    ki.flops_exec_per_iter = fused_flops_per_iter();
                    // frame-FIR levels: parallel efficiency of the chosen blocking (sliding-window form)
                    // and the level to split before when one level cannot fill the CTA
                    {
                        double id = 0, co = 0, worst = 2.0;
                        int wl = 0;
                        for (auto& kv : beam_slide_) {
                            if (kv.second.B <= 0 || kv.second.cost <= 0) continue;
                            id += kv.second.ideal;
                            co += kv.second.cost;
                            const double e = kv.second.ideal / kv.second.cost;
                            const int lv = level_.count(kv.first) ? level_.at(kv.first) : 0;
                            if (e < worst) { worst = e; wl = lv; }
                        }
                        if (co > 0) ki.par_eff = std::min(1.0, id / co);
                        ki.split_level = (worst < 0.6 && wl > 1) ? wl : 0;
                        for (int u : nodes_) ki.node_level.push_back({u, node_level_of(u)});
                    }
                }
            } catch (const FusedFail& ff) {
                if (std::getenv("SG_FUSED_DEBUG")) std::fprintf(stderr, "[sg codegen] partition %d: fused path declined (%s)\n", part_, ff.why);
                WF = 0;
                fast.clear();
            }
            fused_ = false;
        }
        // ---------------- slow (general) path: every compute filter materialised
        size_t budget = opt.smem_budget > 0 ? (size_t)opt.smem_budget : (size_t)(100 * 1024);
        int W = opt.tile;
        if (W <= 0) {
            W = 1;
            for (int cand : {1024, 512, 256, 128, 64, 32, 16, 8, 4, 2, 1}) {
                layout(cand);
                if (smem_bytes_ <= budget) { W = cand; break; }
            }
        }
        layout(W);
        if (WF == 0 && smem_bytes_ > 227 * 1024)
            throw Error(SG_E_SIZE, "partition " + std::to_string(part_) + " needs " + std::to_string(smem_bytes_) +
                                       " B of shared memory for one iteration");
        W_ = W;
        std::ostringstream slow;
        if (WF == 0) {
        emit_loads(slow);
        for (int L = 1; L <= nlev_; L++) {
            slow << "    // ---- level " << L << "\n";
            int64_t rot = 0;
            for (int v : nodes_) {
                if (is_view_node(f_.nodes[v]) || level_[v] != L) continue;
                emit_stage(slow, v, rot);
                rot += f_.nodes[v].halo + (int64_t)W * f_.nodes[v].rep;
            }
            slow << "    __syncthreads();\n";
        }
        emit_stores(slow);
        slow << "    __syncthreads();  // stores of this tile read buffers the next tile's loads may reuse\n";
        }
        size_t smem_slow = smem_bytes_;
        ki.n_levels = nlev_;
        int64_t ksafe = 0;
        for (int v : nodes_) {
            const Node& n = f_.nodes[v];
            int64_t F0 = n.ninit - n.halo;
            if (F0 < 0) ksafe = std::max(ksafe, (-F0 + n.rep - 1) / n.rep);
        }
        const int WT = WF > 0 ? WF : W;
        ki.threads = NT;
        ki.tile = WT;
        ki.smem = WF > 0 ? smem_fast : smem_slow;
        ki.min_blocks = std::max(1, std::min(2, (int)((220 * 1024) / std::max<size_t>(1024, ki.smem))));
        if (const char* mb = std::getenv("SG_MINB")) ki.min_blocks = std::max(1, std::atoi(mb));
        ki.fused = WF > 0;
        ki.ksafe = ksafe;
        std::ostringstream src;
        src << header("staged") << consts_.str() << args_struct(1, WT);
        src << "#define NT " << NT << "\n";
        src << readers_.str();
        auto kernel = [&](const std::string& name, const std::string& body, bool fusedk) {
            src << "extern \"C\" __global__ void __launch_bounds__(NT, " << ki.min_blocks << ") " << name
                << "(const SgArgs a) {\n"
                << "  extern __shared__ __align__(16) unsigned char sg_smem[];\n"
                << "  " << T_ << "* sm = reinterpret_cast<" << T_ << "*>(sg_smem);\n"
                << "  const int tid = threadIdx.x;\n"
                << (fusedk ? prologue_fast : std::string())
                << "  for (long long kt = SG_K_BEGIN + (long long)blockIdx.x * " << (fusedk ? "SG_WR" : std::to_string(WT))
                << "; kt < SG_K_END; kt += (long long)gridDim.x * " << (fusedk ? "SG_WR" : std::to_string(WT)) << ") {\n"
                << "    const int Wtt = (int)min((long long)" << (fusedk ? "SG_WR" : std::to_string(WT)) << ", SG_K_END - kt);\n";
            if (fusedk)
                src << "    const long long k0 = kt;\n    const int Wt = Wtt;\n" << body << "  }\n}\n";
            else
                src << "    for (long long k0 = kt; k0 < kt + Wtt; k0 += " << W << ") {\n"
                    << "      const int Wt = (int)min((long long)" << W << ", kt + Wtt - k0);\n"
                    << body << "    }\n  }\n}\n";
        };
        if (WF > 0) {
            // steady state: tiles with kt >= ksafe; stream start (firings g < 0 emit zeros): the rest
            kernel(ki.name, fast, true);
            ki.name_start = ki.name + "_start";
            kernel(ki.name_start, fast_start, true);
        } else {
            kernel(ki.name, slow.str(), false);
        }
        ki.source = src.str();
        return ki;
    }

private:
    std::map<int, int> level_;      // compute node -> level (1..)
    int nlev_ = 0;
    std::map<int, int64_t> off_;    // phys edge -> smem offset (items)
    std::map<int, int64_t> wb_;     // phys edge -> window base (local position)
    std::map<int, int64_t> size_;   // phys edge -> items at the chosen W
    size_t smem_bytes_ = 0;
    int W_ = 1, NT_ = 256;
    std::ostringstream readers_;
    std::set<int> reader_done_;

    // ======================================================= fused fast path
    // Compute filters whose every output item is read once by a single consumer
    // are inlined into it (SSA registers, no buffer); the rest ("roots") are
    // materialised in shared memory, compacted to their live firings (dead-firing
    // elimination, e.g. FIR outputs dropped by a decimator).  Sibling roots that
    // read the same buffers form one group and share one register window;
    // reductions (ADD, FIR) are emitted transposed across a block of B firings.
    bool fused_ = false;
    bool prefetch_ = false;               // inputs of the next tile prefetched into a staging region
    std::map<int, int64_t> stage_off_;    // input edge -> staging offset (items)
    std::string prologue_;                // emitted before the tile loop (first prefetch, tables)
    int nctr_ = 0;                        // shared work counters used by the fused body (dynamic items)
    std::map<int, int64_t> ctab_off_;     // frame FIR -> coefficient table offset (items)
    std::vector<std::pair<int64_t, std::vector<float>>> ctab_vals_;
    std::map<int, int64_t> plP_, plQ_;  // phys edge -> planar layout: period P, row length Q (odd)
    std::map<int, int64_t> cs_;    // phys edge -> compaction stride (live firings of the producer)
    std::map<int, int64_t> cf0_;   // phys edge -> first live local firing of the producer
    std::set<int> inl_;            // inlined compute nodes
    struct FGroup {
        std::vector<int> roots;
        bool special = false;
        int B = 1;
        int level = 0;
        std::set<int> srcs;
        int64_t NB = 0;
        int64_t flops_block = 0;   // dry-run work of one block (cost model)
    };
    std::vector<FGroup> fg_;
    int flev_ = 0;
    std::map<int, std::vector<Lin>> patterns_;   // materialised edge -> positions read (forms in "jb")
    std::set<int> full_read_;                    // edges read densely (stores, frame FIRs)
    std::map<int, int64_t> NL_;                  // root -> live firings per fast tile
    std::vector<char> inpart_v_;

    struct Sym {
        bool dry = true;
        std::ostringstream* os = nullptr;
        std::map<std::string, std::string> loads;
        std::map<std::string, std::vector<std::string>> firings;
        std::map<std::string, std::vector<std::string>> values;   // CSE: (kind, params, inputs) -> outputs
        bool lockstep = false;                     // every thread runs the block (act: stores)
        int64_t sync_every = 0, since = 0;         // fetch-locality barriers every ~sync_every FP ops
        std::map<int, std::set<std::string>> touched;
        std::map<int, std::vector<Lin>> reads;
        int64_t nloads = 0, flops = 0;
        bool runtime = false;
        int* nv = nullptr;
        std::string ind = "        ";
        bool guarded = false;                      // stream-start variant: firings g < 0 emit zeros
        std::map<int, int64_t> node_flops, node_firings;
    };
    int nvar_ = 0;

    bool in_part(int v) const { return v >= 0 && inpart_v_[v]; }
    bool compute_node(int v) const { return in_part(v) && !is_view_node(f_.nodes[v]); }
    bool special(int v) const { return f_.nodes[v].type == N_FILTER && f_.nodes[v].kind == SG_K_BEAM_FIR; }
    // edge whose producer is not inlined: a shared-memory buffer in the fused layout
    bool materialised(int e) const {
        if (!R_.phys(e)) return false;
        int s = f_.edges[e].src;
        return s < 0 || !in_part(s) || !inl_.count(s);
    }
    void consumers_of(int e, std::set<int>& comp, bool& boundary) const {
        const Edge& ed = f_.edges[e];
        if (ed.dst < 0 || !in_part(ed.dst)) { boundary = true; return; }
        const Node& w = f_.nodes[ed.dst];
        if (is_view_node(w)) { for (int o : w.out) consumers_of(o, comp, boundary); return; }
        comp.insert(ed.dst);
    }
    void sources_of(int e, std::set<int>& out) const {
        if (R_.phys(e)) {
            if (materialised(e)) { out.insert(e); return; }
            sources_of(f_.nodes[f_.edges[e].src].in[0], out);
            return;
        }
        for (int i : f_.nodes[f_.edges[e].src].in) sources_of(i, out);
    }
    std::string zero() const { return "(" + T_ + ")0"; }
    static bool is_zero(const std::string& x) { return x == "0"; }

    std::string sym_value(Sym& c, int e, const Lin& pos) {
        Ref r = R_.resolve(e, pos);
        if (r.k == Ref::ZERO) return "0";
        if (r.k == Ref::RUNTIME) {
            static const bool dbg = std::getenv("SG_FUSED_DEBUG") != nullptr;
            if (dbg && !c.runtime)
                std::fprintf(stderr, "[sg codegen] runtime view: edge %d position %s (resolved to edge %d at %s)\n", e,
                             pos.str().c_str(), r.edge, r.pos.str().c_str());
            c.runtime = true;
            return "0";
        }
        int pe = r.edge;
        const Edge& ed = f_.edges[pe];
        if (materialised(pe)) {
            c.reads[pe].push_back(r.pos);
            std::string key = std::to_string(pe) + "@" + r.pos.str();
            auto it = c.loads.find(key);
            if (it != c.loads.end()) return it->second;
            c.nloads++;
            std::string name = "l" + std::to_string((*c.nv)++);
            if (!c.dry) *c.os << c.ind << "const " << T_ << " " << name << " = sm[" << buf_index(pe, r.pos).str() << "];\n";
            c.loads[key] = name;
            return name;
        }
        const Node& w = f_.nodes[ed.src];
        Lin q = r.pos.plus(-ed.pre);
        if (!q.divisible(w.push)) { c.runtime = true; return "0"; }
        Lin fw = q.divf(w.push);
        int64_t j = q.modc(w.push);
        auto outs = sym_firing(c, ed.src, fw);
        return outs[j];
    }
    std::vector<std::string> sym_firing(Sym& c, int v, const Lin& lf) {
        std::string key = std::to_string(v) + ":" + lf.str();
        auto it = c.firings.find(key);
        if (it != c.firings.end()) return it->second;
        c.touched[v].insert(key);
        const Node& n = f_.nodes[v];
        std::vector<std::string> x(n.peek);
        int64_t use = n.kind == SG_K_FIR ? n.iv[0] : n.peek;
        for (int64_t i = 0; i < use; i++) x[i] = sym_value(c, n.in[0], lf.scaled(n.pop).plus(i));
        for (int64_t i = use; i < n.peek; i++) x[i] = "0";
        // common-subexpression elimination: a firing of a filter with the same kind and
        // parameters on the same input values (e.g. FMRadio's band edges: the high
        // low-pass of band i is the low low-pass of band i+1) is the same value; reuse it
        // so the emitted code and the pruned work count agree
        std::string vkey;
        {
            std::ostringstream k;
            k << n.kind << "|" << n.rep << "|" << n.ninit << "|" << lf.str() << "|";
            for (auto q : n.iv) k << q << ",";
            k << "|";
            for (auto q : n.fv) k << hexf(q) << ",";
            k << "|";
            for (auto& q : x) k << q << ",";
            vkey = k.str();
            auto vit = c.values.find(vkey);
            if (vit != c.values.end()) {
                c.firings[key] = vit->second;
                return vit->second;
            }
        }
        std::vector<std::string> y(n.push);
        for (auto& s : y) s = "y" + std::to_string((*c.nv)++);
        std::ostringstream& o = *c.os;
        const int64_t flops_before = c.flops;
        c.node_firings[v]++;
        if (n.kind == SG_K_FIR) {
            int64_t nz = 0;
            for (int64_t i = 0; i < n.iv[0]; i++) if (!is_zero(x[i])) nz++;
            c.flops += 2 * nz;
            if (nz == 0) { y[0] = "0"; }
            else if (!c.dry) {
                o << c.ind << "float " << y[0] << " = 0.0f;\n";
                for (int64_t i = 0; i < n.iv[0]; i++)
                    if (!is_zero(x[i])) o << c.ind << y[0] << " = fmaf(" << x[i] << ", " << hexf(n.fv[i]) << ", " << y[0] << ");\n";
            }
        } else if (n.kind == SG_K_ADD) {
            c.flops += n.iv[0];
            if (!c.dry) {
                o << c.ind << T_ << " " << y[0] << " = " << zero() << ";\n";
                for (int64_t i = 0; i < n.iv[0]; i++) {
                    if (is_zero(x[i])) continue;
                    if (T_ == "float") o << c.ind << y[0] << " = " << y[0] << " + " << x[i] << ";\n";
                    else o << c.ind << y[0] << " = (int)((unsigned)" << y[0] << " + (unsigned)" << x[i] << ");\n";
                }
            }
        } else {
            int64_t a, b2, d;
            node_work(f_, v, a, b2, d);
            c.flops += n.rep ? a / n.rep : 0;
            if (!c.dry) {
                o << c.ind << T_ << " ";
                for (size_t jj = 0; jj < y.size(); jj++) o << (jj ? ", " : "") << y[jj];
                o << ";\n" << c.ind << "{ const " << T_ << " x_[" << n.peek << "] = {";
                for (int64_t i = 0; i < n.peek; i++) o << (i ? ", " : "") << (is_zero(x[i]) ? zero() : x[i]);
                o << "}; " << T_ << " y_[" << n.push << "]; " << work_call(v);
                for (size_t jj = 0; jj < y.size(); jj++) o << " " << y[jj] << " = y_[" << jj << "];";
                o << " }\n";
            }
        }
        c.node_flops[v] += c.flops - flops_before;
        if (c.guarded && !c.dry)
            for (auto& yy : y)
                if (!is_zero(yy))
                    o << c.ind << yy << " = (k0 * " << n.rep << "LL + " << lf.str() << " < 0) ? " << zero() << " : " << yy << ";\n";
        c.firings[key] = y;
        c.values[vkey] = y;
        return y;
    }
    int64_t root_S(int r) const { auto it = cs_.find(f_.nodes[r].out[0]); return it == cs_.end() ? 1 : it->second; }
    int64_t root_F0L(int r) const {
        int e = f_.nodes[r].out[0];
        auto it = cf0_.find(e);
        return it == cf0_.end() ? f_.nodes[r].ninit - f_.nodes[r].halo : it->second;
    }
    void sym_fir_chunk(Sym& c, const FGroup& g, const std::vector<int>& roots, bool emit_stores) {
        std::ostringstream& o = *c.os;
        const int64_t B = g.B;
        int64_t maxL = 0;
        std::vector<std::vector<Lin>> lf(roots.size(), std::vector<Lin>(B));
        std::vector<std::vector<std::string>> acc(roots.size(), std::vector<std::string>(B));
        for (size_t k = 0; k < roots.size(); k++) {
            int r = roots[k];
            const int64_t S = root_S(r), F0L = root_F0L(r);
            maxL = std::max<int64_t>(maxL, f_.nodes[r].iv[0]);
            c.node_firings[r] += B;
            for (int64_t be = 0; be < B; be++) {
                lf[k][be] = Lin::v("jb", S * B, F0L + S * be);
                acc[k][be] = "a" + std::to_string((*c.nv)++);
                if (!c.dry) o << c.ind << "float " << acc[k][be] << " = 0.0f;\n";
            }
        }
        // Two roots reading the same window (sibling FIRs of a duplicate splitter, FilterBank's 64 band FIRs):
        // their two accumulators form one float2 and every tap is ONE packed FFMA2 (Blackwell fp32x2; each
        // lane an IEEE fma, so each accumulator's tap order and rounding are those of fmaf) with the
        // coefficient pair from a constant table and the sample broadcast (ptxas: `R.F32` operand) -- half the FMA
        // instructions of the level.  Opt-in (SG_FIR_FFMA2=1): FFMA2 takes no 64-bit immediate, so every
        // coefficient pair comes through a uniform-register load (LDCU), and FilterBank measured 0.203 ->
        // 0.252 ms against the scalar immediate-coefficient FFMAs (r02x).
        static const bool ffma2 = std::getenv("SG_FIR_FFMA2") && std::atoi(std::getenv("SG_FIR_FFMA2")) != 0;
        const bool packed = ffma2 && T_ == "float" && roots.size() == 2;
        std::vector<std::string> pk(B);
        if (packed && !c.dry) {
            for (int64_t be = 0; be < B; be++) {
                pk[be] = "p" + std::to_string((*c.nv)++);
                o << c.ind << "float2 " << pk[be] << " = make_float2(" << acc[0][be] << ", " << acc[1][be] << ");\n";
            }
        }
        std::vector<float> cp;  // coefficient pairs of this chunk's packed taps, in emission order
        std::ostringstream po;  // packed tap statements (the table name is known once all pairs are)
        for (int64_t i = 0; i < maxL; i++)
            for (int64_t be = 0; be < B; be++) {
                std::string xs[2];
                for (size_t k = 0; k < roots.size(); k++) {
                    const Node& n = f_.nodes[roots[k]];
                    if (i >= n.iv[0]) continue;
                    xs[k] = sym_value(c, n.in[0], lf[k][be].scaled(n.pop).plus(i));
                }
                const bool both = packed && !xs[0].empty() && xs[0] == xs[1] && !is_zero(xs[0]);
                for (size_t k = 0; k < roots.size(); k++) {
                    const Node& n = f_.nodes[roots[k]];
                    if (i >= n.iv[0] || xs[k].empty() || is_zero(xs[k])) continue;
                    c.flops += 2;
                    c.node_flops[roots[k]] += 2;
                    if (c.dry || both) continue;
                    const std::string a = packed ? pk[be] + (k ? ".y" : ".x") : acc[k][be];
                    po << c.ind << a << " = fmaf(" << xs[k] << ", " << hexf(n.fv[i]) << ", " << a << ");\n";
                }
                if (both && !c.dry) {
                    auto it = dup_.find(xs[0]);
                    std::string d;
                    if (it == dup_.end()) {
                        d = "d" + std::to_string((*c.nv)++);
                        dup_[xs[0]] = d;
                        po << c.ind << "const float2 " << d << " = make_float2(" << xs[0] << ", " << xs[0] << ");\n";
                    } else {
                        d = it->second;
                    }
                    po << c.ind << pk[be] << " = __ffma2_rn(" << d << ", @CP[" << cp.size() / 2 << "], " << pk[be] << ");\n";
                    cp.push_back(f_.nodes[roots[0]].fv[i]);
                    cp.push_back(f_.nodes[roots[1]].fv[i]);
                }
            }
        if (!c.dry) {
            std::string txt = po.str();
            if (!cp.empty()) {
                const std::string tn = "SG_CP" + std::to_string(nvar_++);
                consts_ << "__constant__ float2 " << tn << "[" << cp.size() / 2 << "] = {";
                for (size_t q = 0; q < cp.size(); q += 2) consts_ << (q ? ", " : "") << "{" << hexf(cp[q]) << ", " << hexf(cp[q + 1]) << "}";
                consts_ << "};\n";
                for (size_t p = txt.find("@CP"); p != std::string::npos; p = txt.find("@CP", p)) txt.replace(p, 3, tn);
            }
            o << txt;
            if (packed)
                for (int64_t be = 0; be < B; be++)
                    o << c.ind << acc[0][be] << " = " << pk[be] << ".x; " << acc[1][be] << " = " << pk[be] << ".y;\n";
        }
        if (c.dry || !emit_stores) return;
        for (size_t k = 0; k < roots.size(); k++) {
            const Node& n = f_.nodes[roots[k]];
            const int r = roots[k];
            for (int64_t be = 0; be < B; be++) {
                std::string val = acc[k][be];
                if (c.guarded)
                    val = "((k0 * " + std::to_string(n.rep) + "LL + " + lf[k][be].str() + " < 0) ? " + zero() + " : " + val + ")";
                Lin pos = lf[k][be].scaled(n.push).plus(f_.edges[n.out[0]].pre);
                o << c.ind << guard_store(r, B, be, c.lockstep) << "sm[" << buf_index(n.out[0], pos).str() << "] = " << val << ";\n";
            }
        }
    }
    std::map<std::string, std::string> dup_;  // window value -> its duplicated float2 (one block's scope)
    // One block of a group: roots' live firings F0L + S*(jb*B + beta), beta < B.
    void sym_block(Sym& c, const FGroup& g, bool emit_stores) {
        std::ostringstream& o = *c.os;
        dup_.clear();
        // Sibling FIR roots (one shared window) are emitted in chunks of SG_PAIRS roots with
        // their taps interleaved (taps outer, chunk roots and block firings inner): each warp
        // gets that many independent accumulation chains, while the store guards between
        // chunks keep ptxas from interleaving the whole group (which scatters the warps of an
        // SMSP over the group's straight-line code).  SG_INTERLEAVE=1: one chunk (all roots).
        static const int pairs_env = std::getenv("SG_PAIRS") ? std::atoi(std::getenv("SG_PAIRS")) : 2;
        static const bool interleave = std::getenv("SG_INTERLEAVE") != nullptr;
        bool all_fir = g.roots.size() > 1 && (interleave || pairs_env > 1);
        for (int r : g.roots) all_fir = all_fir && f_.nodes[r].kind == SG_K_FIR;
        if (all_fir) {
            const size_t P = interleave ? g.roots.size() : (size_t)pairs_env;
            for (size_t k0 = 0; k0 < g.roots.size(); k0 += P) {
                std::vector<int> chunk(g.roots.begin() + k0, g.roots.begin() + std::min(g.roots.size(), k0 + P));
                sym_fir_chunk(c, g, chunk, emit_stores);
                fetch_sync(c, 0);
            }
            return;
        }
        for (int r : g.roots) {
            const Node& n = f_.nodes[r];
            const int64_t S = root_S(r), F0L = root_F0L(r), B = g.B;
            std::vector<Lin> lf(B);
            for (int64_t be = 0; be < B; be++) lf[be] = Lin::v("jb", S * B, F0L + S * be);
            std::vector<std::vector<std::string>> outs(B);
            if (n.kind == SG_K_FIR || (n.kind == SG_K_ADD && T_ == "float")) {
                const bool fir = n.kind == SG_K_FIR;
                const int64_t terms = fir ? n.iv[0] : n.iv[0];
                std::vector<std::string> acc(B);
                for (int64_t be = 0; be < B; be++) {
                    acc[be] = "a" + std::to_string((*c.nv)++);
                    if (!c.dry) o << c.ind << "float " << acc[be] << " = 0.0f;\n";
                }
                c.node_firings[r] += B;
                for (int64_t i = 0; i < terms; i++) {
                    const int64_t f0 = c.flops;
                    for (int64_t be = 0; be < B; be++) {
                        std::string x = sym_value(c, n.in[0], lf[be].scaled(n.pop).plus(i));
                        if (is_zero(x)) continue;
                        c.flops += fir ? 2 : 1;
                        c.node_flops[r] += fir ? 2 : 1;
                        if (c.dry) continue;
                        if (fir) o << c.ind << acc[be] << " = fmaf(" << x << ", " << hexf(n.fv[i]) << ", " << acc[be] << ");\n";
                        else o << c.ind << acc[be] << " = " << acc[be] << " + " << x << ";\n";
                    }
                    fetch_sync(c, (c.flops - f0 + 1) / 2);
                }
                for (int64_t be = 0; be < B; be++) outs[be] = {acc[be]};
            } else {
                for (int64_t be = 0; be < B; be++) outs[be] = sym_firing(c, r, lf[be]);
            }
            if (c.dry || !emit_stores) continue;
            const int e = n.out[0];
            for (int64_t be = 0; be < B; be++)
                for (int64_t j = 0; j < n.push; j++) {
                    std::string val = is_zero(outs[be][j]) ? zero() : outs[be][j];
                    if (c.guarded && !is_zero(outs[be][j]))
                        val = "((k0 * " + std::to_string(n.rep) + "LL + " + lf[be].str() + " < 0) ? " + zero() + " : " + val + ")";
                    Lin pos = lf[be].scaled(n.push).plus(f_.edges[e].pre + j);
                    o << c.ind << guard_store(r, B, be, c.lockstep) << "sm[" << buf_index(e, pos).str() << "] = " << val << ";\n";
                }
            fetch_sync(c, 0);
        }
    }
    // Per-store range guards.  The branch they compile to splits a block's code into one
    // basic block per root, so ptxas keeps each root's accumulation chain contiguous;
    // without it (SG_NO_GUARD=1; safe, the buffers are padded) ptxas interleaves every
    // chain of a wide group and the warps of an SMSP drift apart in straight-line code
    // far larger than the instruction caches: FilterBank measured 0.225 ms guarded vs
    // 0.262 ms unguarded (45% of stall samples "no instruction").
    void fetch_sync(Sym& c, int64_t ops) {
        if (c.dry || !c.lockstep || c.sync_every <= 0) return;
        c.since += ops;
        if (c.since >= c.sync_every) {
            *c.os << c.ind << "__syncthreads();  // fetch locality\n";
            c.since = 0;
        }
    }
    static std::string guard_store(int r, int64_t B, int64_t be, bool lockstep = false) {
        static const bool on = std::getenv("SG_NO_GUARD") == nullptr;
        if (lockstep) return "if (act && jb * " + std::to_string(B) + " + " + std::to_string(be) + " < NL" + std::to_string(r) + ") ";
        if (!on) return "";
        return "if (jb * " + std::to_string(B) + " + " + std::to_string(be) + " < NL" + std::to_string(r) + ") ";
    }
    bool dry_ok(const FGroup& g, Sym& c) {
        c = Sym();
        c.dry = true;
        std::ostringstream sink;
        c.os = &sink;
        c.nv = &nvar_;
        sym_block(c, g, false);
        return !c.runtime;
    }
    void fused_analyze() {
        inpart_v_.assign(f_.nodes.size(), 0);
        for (int v : nodes_) inpart_v_[v] = 1;
        inl_.clear();
        cs_.clear();
        cf0_.clear();
        patterns_.clear();
        full_read_.clear();
        fg_.clear();
        // ---- inline decisions, consumers first
        for (auto it = nodes_.rbegin(); it != nodes_.rend(); ++it) {
            int u = *it;
            if (!compute_node(u) || special(u)) continue;
            std::set<int> comp;
            bool boundary = false;
            consumers_of(f_.nodes[u].out[0], comp, boundary);
            if (boundary || comp.size() != 1) continue;
            int v = *comp.begin();
            if (special(v)) continue;
            // opt-in (A/B): keep an accumulate chain's partial sums materialised, one level per group
            static const bool keep_acc = std::getenv("SG_KEEP_ACC") != nullptr;
            if (keep_acc && f_.nodes[u].kind == SG_K_ADD && f_.nodes[v].kind == SG_K_ADD) continue;
            inl_.insert(u);
            FGroup g;
            g.roots = {v};
            bool ok = false;
            int Bn = 0;
            Sym c;
            for (int B : {1, 2, 4, 8, 16, 32, 64}) {
                g.B = B;
                if (dry_ok(g, c)) { Bn = B; ok = true; break; }
            }
            if (!ok) { inl_.erase(u); continue; }
            g.B = std::max(Bn, 8);
            if (!dry_ok(g, c)) g.B = Bn, dry_ok(g, c);
            int64_t c1 = c.touched[u].size();
            g.B *= 16;
            if (!dry_ok(g, c)) { inl_.erase(u); continue; }
            int64_t cK = c.touched[u].size();
            if (!(c1 * 16 <= 1.25 * cK)) inl_.erase(u);
        }
        // ---- roots, their sources and levels
        std::vector<int> roots;
        for (int v : nodes_) if (compute_node(v) && !inl_.count(v)) roots.push_back(v);
        std::map<int, int> lvl;
        std::map<int, std::set<int>> srcs;
        flev_ = 0;
        for (int r : roots) {
            sources_of(f_.nodes[r].in[0], srcs[r]);
            int L = 0;
            for (int e : srcs[r]) {
                int sp = f_.edges[e].src;
                if (sp >= 0 && in_part(sp)) L = std::max(L, lvl.at(sp));
            }
            lvl[r] = L + 1;
            flev_ = std::max(flev_, L + 1);
        }
        // stores and frame FIRs read densely
        for (int e : outs_) {
            std::set<int> s2;
            if (R_.phys(e)) s2.insert(e); else sources_of(e, s2);
            if (!R_.phys(e)) {
                // views between the buffer and the store: positions may be strided; keep dense
            }
            for (int x : s2) full_read_.insert(x);
        }
        for (int r : roots) if (special(r)) for (int e : srcs[r]) full_read_.insert(e);
        // ---- levels from the top: live strides, groups, block sizes, read patterns
        for (int L = flev_; L >= 1; L--) {
            std::vector<int> here;
            for (int r : roots) if (lvl[r] == L) here.push_back(r);
            for (int r : here) {
                const Node& n = f_.nodes[r];
                const int e = n.out[0];
                const Edge& ed = f_.edges[e];
                int64_t S = 1, rho = 0;
                auto pit = patterns_.find(e);
                if (!special(r) && n.push == 1 && !full_read_.count(e) && pit != patterns_.end() && !pit->second.empty()) {
                    int64_t g = 0, c0 = pit->second[0].c;
                    for (auto& lp : pit->second) {
                        for (auto& t : lp.t) g = std::gcd(g, std::llabs(t.second));
                        g = std::gcd(g, std::llabs(lp.c - c0));
                    }
                    if (g > 1 && n.rep % g == 0) { S = g; rho = fmodp(c0 - ed.pre, S); }
                }
                const int64_t F0 = n.ninit - n.halo;
                cs_[e] = S;
                cf0_[e] = F0 + fmodp(rho - F0, S);
            }
            // group siblings: same rep, stride, sources (non-special)
            std::map<std::string, FGroup> bysig;
            std::vector<FGroup> singles;
            for (int r : here) {
                FGroup g;
                g.roots = {r};
                g.level = L;
                g.srcs = srcs[r];
                if (special(r)) { g.special = true; singles.push_back(g); continue; }
                std::ostringstream sig;
                sig << f_.nodes[r].rep << "/" << root_S(r) << "/" << f_.nodes[r].push << "/" << f_.nodes[r].halo << "/"
                    << f_.nodes[r].ninit << ":";
                for (int e : srcs[r]) sig << e << ",";
                auto it = bysig.find(sig.str());
                if (it == bysig.end()) bysig[sig.str()] = g;
                else it->second.roots.push_back(r);
            }
            for (auto& kv : bysig) singles.push_back(kv.second);
            for (auto& g : singles) {
                if (!g.special) {
                    Sym c;
                    int B0 = 0;
                    for (int B : {1, 2, 4, 8, 16, 32, 64}) {
                        g.B = B;
                        if (dry_ok(g, c)) { B0 = B; break; }
                    }
                    if (!B0) throw FusedFail{"site 1"};
                    g.B = B0;
                    static const int bmax = std::getenv("SG_FUSED_BMAX") ? std::atoi(std::getenv("SG_FUSED_BMAX")) : 16;
                    dry_ok(g, c);
                    // blocking only pays when consecutive firings share loaded items (peek
                    // windows, inlined producers); without sharing it only cuts the
                    // parallelism and multiplies the lane stride (bank conflicts)
                    bool shares = true;
                    {
                        FGroup h = g;
                        h.B = g.B * 2;
                        Sym c2;
                        if (dry_ok(h, c2) && c2.nloads >= 2 * c.nloads) shares = false;
                    }
                    while (shares && g.B * 2 <= bmax) {
                        FGroup h = g;
                        h.B = g.B * 2;
                        Sym c2;
                        static const int64_t fcap = std::getenv("SG_FUSED_FLOPCAP") ? std::atoll(std::getenv("SG_FUSED_FLOPCAP")) : 2048;
                        if (!dry_ok(h, c2) || c2.flops > fcap || c2.nloads > 96) break;
                        g.B = h.B;
                        c = c2;
                    }
                    dry_ok(g, c);
                    g.flops_block = c.flops + c.nloads;
                    for (auto& kv : c.reads) for (auto& lp : kv.second) patterns_[kv.first].push_back(lp);
                }
                fg_.push_back(g);
            }
        }
        std::stable_sort(fg_.begin(), fg_.end(), [](const FGroup& a, const FGroup& b) { return a.level < b.level; });
        // planar layouts for buffers read by frame FIRs: period P = gcd of every reader's and
        // writer's position strides, so that per-thread blocks of odd length hit distinct banks
        plP_.clear();
        std::map<int, int64_t> gP;
        std::set<int> special_read;
        auto acc = [&](int e, int64_t a) { gP[e] = std::gcd(gP[e], std::llabs(a)); };
        for (auto& g : fg_) {
            if (!g.special) continue;
            for (int r : g.roots) {
                const Node& n = f_.nodes[r];
                Lin pr = Lin::v("lf", n.pop, 0);
                pr.t.push_back({"s0", 2});
                for (int k = 0; k < 2; k++) {
                    Ref rf = R_.resolve(n.in[0], pr.plus(k));
                    if (rf.k != Ref::PHYS || !materialised(rf.edge)) continue;
                    special_read.insert(rf.edge);
                    for (auto& t : rf.pos.t) acc(rf.edge, t.second);
                }
                acc(n.out[0], n.push);   // its own output: positions j*push + 2*t
                acc(n.out[0], 2);
            }
        }
        for (auto& kv : patterns_)
            for (auto& lp : kv.second)
                for (auto& t : lp.t) acc(kv.first, t.second);
        for (auto& g : fg_) {
            if (g.special) continue;
            for (int r : g.roots) acc(f_.nodes[r].out[0], f_.nodes[r].push * root_S(r) * g.B);
        }
        // frame-FIR outputs too (their readers -- beamforming, magnitudes -- then load re and im from two
        // planes at unit stride instead of stride 2: no 2-way bank conflicts); SG_PLANAR_OUT=0 turns it off
        static const bool planar_out = !std::getenv("SG_PLANAR_OUT") || std::atoi(std::getenv("SG_PLANAR_OUT")) != 0;
        if (planar_out)
            for (auto& g : fg_)
                if (g.special)
                    for (int r : g.roots)
                        if (materialised(f_.nodes[r].out[0])) special_read.insert(f_.nodes[r].out[0]);
        for (int e : special_read) {
            int64_t P = gP[e];
            if (P > 1 && P <= 64 && (!cs_.count(e) || cs_[e] == 1)) plP_[e] = P;
        }
    }
    void fused_layout(int W) {
        W_ = W;
        beam_B_.clear();
        beam_slide_.clear();
        off_.clear();
        wb_.clear();
        size_.clear();
        NL_.clear();
        struct Buf { int e; int64_t size; int birth, death; };
        std::map<int, Buf> bufs;
        auto note = [&](int e, int64_t size, int birth) {
            if (!bufs.count(e)) bufs[e] = {e, size, birth, birth};
        };
        for (size_t i = 0; i < ins_.size(); i++) {
            int e = ins_[i];
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            wb_[e] = lo;
            note(e, f_.edges[e].per_iter * W + ex, 0);
        }
        for (auto& g : fg_) {
            for (int r : g.roots) {
                const Node& n = f_.nodes[r];
                const int e = n.out[0];
                const int64_t S = root_S(r), F0 = n.ninit - n.halo, F0L = root_F0L(r);
                const int64_t end = F0 + n.halo + (int64_t)W * n.rep;  // exclusive
                const int64_t NL = end > F0L ? (end - 1 - F0L) / S + 1 : 0;
                NL_[r] = NL;
                wb_[e] = f_.edges[e].pre + F0L * n.push;
            }
        }
        for (auto& g : fg_) {
            int64_t nb = 0;
            for (int r : g.roots) nb = std::max(nb, (NL_[r] + g.B - 1) / g.B);
            g.NB = g.special ? 0 : nb;
            // every root buffer has room for all NB * B firings of its group (the tail is
            // never read), so block stores may go unguarded (see guard_store)
            for (int r : g.roots) {
                const Node& n = f_.nodes[r];
                note(n.out[0], std::max(NL_[r], g.special ? 0 : g.NB * g.B) * n.push, g.level);
            }
        }
        // extents read by the first and last block of every group; liveness
        for (auto& g : fg_) {
            for (int e : g.srcs) if (bufs.count(e)) bufs[e].death = std::max(bufs[e].death, g.level);
            if (g.special || g.NB == 0) continue;
            Sym c;
            dry_ok(g, c);
            for (auto& kv : c.reads) {
                int e = kv.first;
                if (!bufs.count(e)) continue;
                for (auto& lp : kv.second)
                    for (int64_t jb : {(int64_t)0, g.NB - 1}) {
                        int64_t pos = lp.c + lp.coef("jb") * jb;
                        int64_t idx;
                        auto it = cs_.find(e);
                        if (it != cs_.end() && it->second > 1) {
                            int64_t q = pos - f_.edges[e].pre - cf0_.at(e);
                            if (fmodp(q, it->second) != 0) throw FusedFail{"site 2"};
                            idx = fdiv(q, it->second);
                        } else {
                            idx = pos - wb_.at(e);
                        }
                        if (idx < 0) throw FusedFail{"site 3"};
                        bufs[e].size = std::max(bufs[e].size, idx + 1);
                    }
            }
        }
        for (int e : outs_) {
            std::set<int> s2;
            if (R_.phys(e)) s2.insert(e); else sources_of(e, s2);
            for (int x : s2) if (bufs.count(x)) bufs[x].death = flev_ + 1;
        }
        plQ_.clear();
        for (auto& kv : bufs) {
            auto it = plP_.find(kv.first);
            if (it == plP_.end()) continue;
            int64_t P = it->second, Q = (kv.second.size + P - 1) / P;
            if (Q % 2 == 0) Q++;
            plQ_[kv.first] = Q;
            kv.second.size = P * Q;
        }
        std::vector<Buf> list;
        for (auto& kv : bufs) list.push_back(kv.second);
        std::stable_sort(list.begin(), list.end(), [](const Buf& a, const Buf& b) { return a.size > b.size; });
        std::vector<Buf> placed;
        int64_t top = 0;
        for (auto& b : list) {
            int64_t sz = (b.size + 3) / 4 * 4;
            std::vector<std::pair<int64_t, int64_t>> busy;
            for (auto& q : placed)
                if (!(q.death < b.birth || b.death < q.birth))
                    busy.push_back({off_[q.e], off_[q.e] + (q.size + 3) / 4 * 4});
            std::sort(busy.begin(), busy.end());
            int64_t o = 0;
            for (auto& iv : busy) {
                if (o + sz <= iv.first) break;
                o = std::max(o, iv.second);
            }
            off_[b.e] = o;
            size_[b.e] = b.size;
            top = std::max(top, o + sz);
            placed.push_back(b);
        }
        // frame-FIR coefficient tables ((cr, ci) interleaved, read as 128-bit broadcasts)
        ctab_off_.clear();
        ctab_vals_.clear();
        {
            std::map<std::vector<float>, int64_t> seen;
            top = (top + 3) / 4 * 4;
            for (auto& g : fg_) {
                if (!g.special) continue;
                for (int r : g.roots) {
                    const Node& n = f_.nodes[r];
                    const int64_t L = n.iv[0];
                    std::vector<float> t(2 * L);
                    for (int64_t i = 0; i < L; i++) { t[2 * i] = n.fv[i]; t[2 * i + 1] = n.fv[L + i]; }
                    auto it = seen.find(t);
                    if (it == seen.end()) {
                        seen[t] = top;
                        ctab_vals_.push_back({top, t});
                        ctab_off_[r] = top;
                        top += (2 * L + 3) / 4 * 4;
                    } else {
                        ctab_off_[r] = it->second;
                    }
                }
            }
        }
        smem_bytes_ = (size_t)std::max<int64_t>(top, 4) * 4;
    }
    // live root firings in a tile of W iterations
    int64_t nl_of(int r, int64_t W) const {
        const Node& n = f_.nodes[r];
        const int64_t S = root_S(r), F0 = n.ninit - n.halo, F0L = root_F0L(r);
        return (F0 + n.halo - 1 - F0L + W * n.rep) / S + 1;
    }
    // Tile sizes ordered by a cost model: per level, ceil(blocks / NT) rounds of
    // the heaviest block, summed, per iteration; candidates include the sizes that
    // make a group's block count a multiple of NT (no straggler round).
    std::vector<int> fused_tile_candidates(int forced) {
        if (forced > 0) return {forced};
        std::set<int64_t> cand;
        for (int64_t w = 1; w <= 4096; w *= 2) cand.insert(w);
        for (auto& g : fg_) {
            if (g.special) continue;
            for (int64_t k = 1; k <= 16; k++) {
                int64_t lo = 1, hi = 8192;  // largest W with NB_g(W) <= k*NT
                if ((nl_of(g.roots[0], 1) + g.B - 1) / g.B > k * NT_) continue;
                while (lo < hi) {
                    int64_t mid = (lo + hi + 1) / 2;
                    int64_t nb = 0;
                    for (int r : g.roots) nb = std::max(nb, (nl_of(r, mid) + g.B - 1) / g.B);
                    if (nb <= k * NT_) lo = mid; else hi = mid - 1;
                }
                if (lo >= 1 && lo <= 8192) cand.insert(lo);
            }
        }
        std::vector<std::pair<double, int>> scored;
        for (int64_t W : cand) {
            double tile = 0;
            for (int L = 1; L <= flev_; L++) {
                int64_t items = 0, worst = 1;
                for (auto& g : fg_) {
                    if (g.level != L) continue;
                    if (g.special) {
                        for (int r : g.roots) {
                            const Node& n = f_.nodes[r];
                            int64_t per = (n.iv[2] / n.iv[1] + 3) / 4;
                            items += (n.halo + W * n.rep) * per;
                            worst = std::max<int64_t>(worst, 32LL * n.iv[0]);
                        }
                        continue;
                    }
                    int64_t nb = 0;
                    for (int r : g.roots) nb = std::max(nb, (nl_of(r, W) + g.B - 1) / g.B);
                    items += nb;
                    worst = std::max(worst, g.flops_block);
                }
                tile += (double)((items + NT_ - 1) / NT_) * (double)worst + 200.0;
            }
            scored.push_back({tile / (double)W, (int)W});
        }
        // equal cost per iteration (e.g. a partition of views only, no compute level): the larger tile
        // amortises the per-tile halo, barriers and loop overhead
        std::sort(scored.begin(), scored.end(), [](const std::pair<double, int>& a, const std::pair<double, int>& b) {
            return a.first != b.first ? a.first < b.first : a.second > b.second;
        });
        std::vector<int> out;
        for (auto& p : scored) out.push_back(p.second);
        return out;
    }
    // Fused tile body for a runtime Wt <= W.  guarded: the stream-start variant.
    std::string fused_emit(int W, bool guarded) {
        std::ostringstream b;
        nctr_ = 0;
        std::ostringstream body;
        std::string r = fused_emit_body(W, guarded, body);
        if (nctr_ > 0)  // work counters: zeroed at tile start (the previous tile ended with a barrier,
                        // the post-load barrier orders the reset before the first level)
            b << "    __shared__ int sg_ctr[" << nctr_ << "];\n"
              << "    if (tid < " << nctr_ << ") sg_ctr[tid] = 0;\n";
        b << r;
        return b.str();
    }
    std::string fused_emit_body(int W, bool guarded, std::ostringstream& b) {
        {
            std::ostringstream pb;
            for (auto& kv : ctab_vals_) {
                std::string name = const_array(kv.second);
                pb << "  for (int j = tid; j < " << kv.second.size() << "; j += NT) sm[" << kv.first << " + j] = " << name
                   << "[j];  // frame-FIR coefficient table\n";
            }
            if (prefetch_) {
                pb << "  int sg_pm[" << std::max<size_t>(1, ins_.size()) << "];  // staging misalignment (items) per input\n";
                emit_issue(pb, "SG_K_BEGIN + (long long)blockIdx.x * SG_WR", true);
            }
            prologue_ = pb.str();
        }
        emit_loads(b);
        for (int L = 1; L <= flev_; L++) {
            b << "    // ---- fused level " << L << "\n";
            int64_t rot = 0;
            emit_specials(b, L, rot);
            for (auto& g : fg_) {
                if (g.level != L) continue;
                if (g.special) continue;
                b << "    { // group of " << g.roots.size() << " root(s) [" << kind_name(f_.nodes[g.roots[0]].kind)
                  << "], B = " << g.B << ", blocks per full tile = " << g.NB << "\n";
                b << "      int NBg = 0;\n";
                for (int r : g.roots) {
                    const Node& n = f_.nodes[r];
                    const int64_t S = root_S(r), F0 = n.ninit - n.halo, F0L = root_F0L(r);
                    b << "      const int NL" << r << " = (" << F0 + n.halo - 1 - F0L << " + Wt * " << n.rep << ") / " << S
                      << " + 1;\n"
                      << "      NBg = max(NBg, (NL" << r << " + " << g.B - 1 << ") / " << g.B << ");\n";
                }
                // lockstep: a level with one large group whose blocks fit one round runs every
                // thread through the block once (idle threads recompute the last block and
                // store nothing) with __syncthreads() every ~512 FP instructions, so the warps
                // of a CTA stay within a few KB of straight-line code (instruction-fetch
                // locality; FilterBank's levels are 35-46 KB of code each)
                int nlev_groups = 0;
                for (auto& h : fg_) if (h.level == L) nlev_groups++;
                static const bool fetchbar = std::getenv("SG_FETCHBAR") != nullptr;  // measured neutral-to-worse
                const bool lockstep = fetchbar && nlev_groups == 1 && g.NB <= NT_ && g.flops_block >= 2048;
                // warp sub-groups: a group of many sibling roots (FilterBank: 64 FIR_H on one window) is
                // split into K contiguous root ranges, warp w running range w mod K over every block, so
                // each warp scheduler streams ~1/K of the level's straight-line code (instruction-fetch
                // locality: L0 ~6 KB, L1.5 ~32 KB per SM) at the cost of K reloads of the shared window
                static const int ksub_env = std::getenv("SG_SUBGROUPS") ? std::atoi(std::getenv("SG_SUBGROUPS")) : 0;
                const int ksub = ksub_env;
                if (!lockstep && ksub > 1 && (int)g.roots.size() >= 2 * ksub && NT_ % (32 * ksub) == 0) {
                    b << "      const int sgw = (tid >> 5) % " << ksub << ";\n"
                      << "      const int tsg = ((tid >> 5) / " << ksub << ") * 32 + (tid & 31);\n";
                    const size_t nr = g.roots.size();
                    for (int q = 0; q < ksub; q++) {
                        FGroup h = g;
                        h.roots.assign(g.roots.begin() + nr * q / ksub, g.roots.begin() + nr * (q + 1) / ksub);
                        Sym cq;
                        cq.dry = false;
                        cq.os = &b;
                        cq.nv = &nvar_;
                        cq.guarded = guarded;
                        b << "      " << (q ? "else " : "") << "if (sgw == " << q << ") {\n"
                          << "      for (int jb = tsg; jb < NBg; jb += " << NT_ / ksub << ") {\n";
                        sym_block(cq, h, true);
                        if (cq.runtime) throw FusedFail{"site 4"};
                        b << "      }\n      }\n";
                    }
                    b << "    }\n";
                    rot += g.NB;
                    continue;
                }
                Sym c;
                c.dry = false;
                c.os = &b;
                c.nv = &nvar_;
                c.guarded = guarded;
                if (lockstep) {
                    b << "      if (NBg > 0) {\n"
                      << "      const bool act = tid < NBg;\n"
                      << "      const int jb = act ? tid : NBg - 1;\n";
                    c.lockstep = true;
                    static const int every = std::getenv("SG_FETCHBAR_OPS") ? std::atoi(std::getenv("SG_FETCHBAR_OPS")) : 512;
                    c.sync_every = every;
                } else {
                    b << "      int jb = tid - " << rot % NT_ << "; if (jb < 0) jb += NT;\n"
                      << "      for (; jb < NBg; jb += NT) {\n";
                }
                sym_block(c, g, true);
                if (c.runtime) throw FusedFail{"site 5"};
                b << "      }\n    }\n";
                rot += g.NB;
            }
            b << "    __syncthreads();\n";
        }
        emit_stores(b);
        b << "    __syncthreads();\n";
        return b.str();
    }
    // frame-FIR stages of one level, peers sharing one body where possible
    void emit_specials(std::ostringstream& b, int L, int64_t& rot) {
        std::vector<int> sp;
        for (auto& g : fg_)
            if (g.special && g.level == L)
                for (int r : g.roots) sp.push_back(r);
        std::vector<char> done(sp.size(), 0);
        for (size_t a = 0; a < sp.size(); a++) {
            if (done[a]) continue;
            std::vector<int> peers{sp[a]};
            done[a] = 1;
            for (size_t c = a + 1; c < sp.size(); c++)
                if (!done[c] && f_.nodes[sp[c]].iv == f_.nodes[sp[a]].iv && f_.nodes[sp[c]].fv == f_.nodes[sp[a]].fv) {
                    peers.push_back(sp[c]);
                    done[c] = 1;
                }
            std::vector<int64_t> din, dout;
            if (peers.size() > 1 && beam_peer_offsets(peers, din, dout)) {
                const Node& n = f_.nodes[peers[0]];
                b << "    { // " << peers.size() << " peer frame FIRs (shared body)\n"
                  << "      const int nf = " << n.halo << " + Wt * " << n.rep << ";\n"
                  << "      const long long gf = k0 * " << n.rep << "LL;\n";
                emit_beam_fir(b, peers[0], n.ninit - n.halo, rot, peers, din, dout);
                b << "    }\n";
                rot += (int64_t)peers.size() * (n.halo + (int64_t)W_ * n.rep);
            } else {
                for (int r : peers) {
                    emit_stage(b, r, rot);
                    rot += f_.nodes[r].halo + (int64_t)W_ * f_.nodes[r].rep;
                }
            }
        }
    }
    // Algorithmic fp32 work per iteration of the fused plan: dead firings and zero
    // taps removed, recomputed (halo / inlining overlap) firings not counted.
    int64_t fused_flops_per_iter() {
        double tot = 0;
        for (auto& g : fg_) {
            if (g.special) {  // live taps only: x[s < 0] = 0 before the frame start (skipped chunks)
                for (int r : g.roots) {
                    const Node& n = f_.nodes[r];
                    const int64_t L = n.iv[0], DEC = n.iv[1], OUT = n.iv[2] / n.iv[1];
                    int64_t taps = 0;
                    for (int64_t t = 0; t < OUT; t++) taps += std::min<int64_t>(L, t * DEC + 1);
                    tot += 8.0 * (double)taps * (double)n.rep;
                }
                continue;
            }
            Sym c;
            dry_ok(g, c);
            for (auto& kv : c.node_flops) {
                int v = kv.first;
                int64_t nf = c.node_firings[v];
                if (nf <= 0) continue;
                const Node& n = f_.nodes[v];
                int64_t S = inl_.count(v) ? 1 : root_S(v);
                tot += (double)kv.second / nf * (double)n.rep / S;
            }
        }
        return (int64_t)(tot + 0.5);
    }
    int producer_level(int e) {
        const Edge& ed = f_.edges[e];
        if (!R_.phys(e)) throw Error(SG_E_UNSUPPORTED, "internal");
        if (ed.src < 0 || std::find(ins_.begin(), ins_.end(), e) != ins_.end()) return 0;
        return level_.at(ed.src);
    }
    void compute_levels() {
        nlev_ = 0;
        for (int v : nodes_) {  // topological order
            const Node& n = f_.nodes[v];
            if (is_view_node(n)) continue;
            std::set<int> src;
            R_.sources(n.in[0], src);
            int L = 0;
            for (int e : src) L = std::max(L, producer_level(e));
            level_[v] = L + 1;
            nlev_ = std::max(nlev_, L + 1);
        }
    }
    // buffers, windows and liveness-based placement for tile W
    void layout(int W) {
        off_.clear();
        wb_.clear();
        size_.clear();
        struct Buf { int e; int64_t size; int birth, death; };
        std::vector<Buf> bufs;
        std::map<int, int> death;
        auto note_reads = [&](int e_in, int lvl) {
            std::set<int> src;
            R_.sources(e_in, src);
            for (int s : src) death[s] = std::max(death[s], lvl);
        };
        for (int v : nodes_) {
            const Node& n = f_.nodes[v];
            if (is_view_node(n)) continue;
            note_reads(n.in[0], level_[v]);
        }
        for (int e : outs_) note_reads(e, nlev_ + 1);
        for (size_t i = 0; i < ins_.size(); i++) {
            int e = ins_[i];
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            int64_t sz = f_.edges[e].per_iter * W + ex;
            wb_[e] = lo;
            bufs.push_back({e, sz, 0, death.count(e) ? death[e] : 0});
        }
        for (int v : nodes_) {
            const Node& n = f_.nodes[v];
            if (is_view_node(n)) continue;
            int e = n.out[0];
            const Edge& ed = f_.edges[e];
            wb_[e] = ed.pre + (n.ninit - n.halo) * n.push;
            int64_t sz = (n.halo + (int64_t)W * n.rep) * n.push;
            bufs.push_back({e, sz, level_[v], death.count(e) ? death[e] : level_[v]});
        }
        std::vector<int> order(bufs.size());
        std::iota(order.begin(), order.end(), 0);
        std::stable_sort(order.begin(), order.end(), [&](int a, int b) { return bufs[a].size > bufs[b].size; });
        std::vector<int> placed;
        int64_t top = 0;
        for (int bi : order) {
            Buf& b = bufs[bi];
            int64_t sz = (b.size + 3) / 4 * 4;
            // candidate offsets: 0 and the end of every live-overlapping placed buffer
            std::vector<std::pair<int64_t, int64_t>> busy;
            for (int pj : placed) {
                Buf& q = bufs[pj];
                bool overlap = !(q.death < b.birth || b.death < q.birth);
                if (overlap) busy.push_back({off_[q.e], off_[q.e] + (q.size + 3) / 4 * 4});
            }
            std::sort(busy.begin(), busy.end());
            int64_t o = 0;
            for (auto& iv : busy) {
                if (o + sz <= iv.first) break;
                o = std::max(o, iv.second);
            }
            off_[b.e] = o;
            size_[b.e] = b.size;
            top = std::max(top, o + sz);
            placed.push_back(bi);
        }
        smem_bytes_ = (size_t)std::max<int64_t>(top, 4) * 4;
    }
    std::string rd_name(int e) { return "sg_rd" + std::to_string(e); }
    // runtime reader through views (fallback when static resolution fails)
    void gen_reader(int e) {
        if (reader_done_.count(e)) return;
        reader_done_.insert(e);
        std::ostringstream s;
        s << "__device__ __forceinline__ " << T_ << " " << rd_name(e) << "(const " << T_ << "* sm, int lp) {\n";
        if (R_.phys(e)) {
            s << "  return sm[" << off_.at(e) - wb_.at(e) << " + lp];\n}\n";
            readers_ << s.str();
            return;
        }
        const Edge& ed = f_.edges[e];
        const Node& u = f_.nodes[ed.src];
        std::vector<int> deps;
        switch (u.type) {
        case N_SPLIT_DUP: s << "  return " << rd_name(u.in[0]) << "(sm, lp);\n"; deps.push_back(u.in[0]); break;
        case N_SPLIT_RR: {
            int64_t w = u.w[ed.sport], P = 0;
            for (int i = 0; i < ed.sport; i++) P += u.w[i];
            s << "  const int q = sg_fdiv32(lp, " << w << "), r = lp - q * " << w << ";\n";
            s << "  return " << rd_name(u.in[0]) << "(sm, q * " << u.wsum << " + " << P << " + r);\n";
            deps.push_back(u.in[0]);
            break;
        }
        case N_JOIN: {
            s << "  const int q = sg_fdiv32(lp, " << u.wsum << "), o = lp - q * " << u.wsum << ";\n";
            int64_t P = 0;
            for (size_t b = 0; b < u.w.size(); b++) {
                s << "  if (o < " << P + u.w[b] << ") return " << rd_name(u.in[b]) << "(sm, q * " << u.w[b] << " + o - "
                  << P << ");\n";
                deps.push_back(u.in[b]);
                P += u.w[b];
            }
            s << "  return (" << T_ << ")0;\n";
            break;
        }
        case N_FILTER: {
            int in = u.in[0];
            deps.push_back(in);
            switch (u.kind) {
            case SG_K_IDENTITY: s << "  return " << rd_name(in) << "(sm, lp);\n"; break;
            case SG_K_DELAY: s << "  return " << rd_name(in) << "(sm, lp - " << u.iv[0] << ");\n"; break;
            case SG_K_DECIMATE: s << "  return " << rd_name(in) << "(sm, lp * " << u.iv[0] << ");\n"; break;
            case SG_K_EXPAND:
                s << "  const int q = sg_fdiv32(lp, " << u.iv[0] << ");\n  return (lp - q * " << u.iv[0] << ") == 0 ? "
                  << rd_name(in) << "(sm, q) : (" << T_ << ")0;\n";
                break;
            case SG_K_PERMUTE: {
                const int64_t n = u.iv[0], m = (int64_t)u.iv.size() - 1;
                std::string tab = "SG_PI" + std::to_string(ipool_n_++);
                consts_ << "__constant__ int " << tab << "[" << m << "] = {";
                for (int64_t k = 0; k < m; k++) consts_ << (k ? "," : "") << (k % 16 == 0 ? "\n  " : "") << u.iv[1 + k];
                consts_ << "};\n";
                s << "  const int q = sg_fdiv32(lp, " << m << "), o = lp - q * " << m << ";\n"
                  << "  return " << rd_name(in) << "(sm, q * " << n << " + " << tab << "[o]);\n";
                break;
            }
            case SG_K_FFT_REORDER: {
                int64_t n = u.iv[0], F = 2 * n;
                s << "  const int q = sg_fdiv32(lp, " << F << "), o = lp - q * " << F << ";\n"
                  << "  const int m = o >> 1, r = o & 1;\n"
                  << "  const int sc = m < " << n / 2 << " ? 2 * m : 2 * (m - " << n / 2 << ") + 1;\n"
                  << "  return " << rd_name(in) << "(sm, q * " << F << " + 2 * sc + r);\n";
                break;
            }
            default: throw Error(SG_E_UNSUPPORTED, "internal: reader for compute node");
            }
            break;
        }
        }
        s << "}\n";
        for (int d : deps) gen_reader(d);  // callees first
        readers_ << s.str();
    }
    struct FusedFail {
        const char* why = "";
    };
    // shared-memory index of position `pos` of physical edge e in the current layout
    Lin buf_index(int e, const Lin& pos) {
        auto pit = plP_.find(e);
        if (fused_ && pit != plP_.end() && pit->second > 1) {  // planar: [P][Q], Q odd
            const int64_t P = pit->second, Q = plQ_.at(e);
            Lin j = pos.plus(-wb_.at(e));
            if (!j.divisible(P)) throw FusedFail{"site 6"};
            return j.divf(P).plus(j.modc(P) * Q + off_.at(e));
        }
        auto it = cs_.find(e);
        if (fused_ && it != cs_.end() && it->second > 1) {
            const Edge& ed = f_.edges[e];
            Lin q = pos.plus(-(ed.pre + cf0_.at(e)));
            if (!q.divisible(it->second) || q.modc(it->second) != 0) throw FusedFail{"site 7"};
            return q.divf(it->second).plus(off_.at(e));
        }
        return pos.plus(off_.at(e) - wb_.at(e));
    }
    std::string read_expr(int e, const Lin& pos) {
        Ref r = R_.resolve(e, pos);
        if (r.k == Ref::ZERO) return "(" + T_ + ")0";
        if (r.k == Ref::RUNTIME) {
            if (fused_) {
                // a view map that is not affine in the loop index (e.g. the transposing joins of a 2-D DCT
                // in a store): generated index readers over dense, uncompacted buffers
                std::set<int> src;
                R_.sources(r.edge, src);
                for (int pe : src) {
                    const bool dense = materialised(pe) && off_.count(pe) && wb_.count(pe) &&
                                       !(cs_.count(pe) && cs_.at(pe) > 1) && !(plP_.count(pe) && plP_.at(pe) > 1);
                    if (!dense) throw FusedFail{"site 8"};
                }
            }
            gen_reader(r.edge);
            return rd_name(r.edge) + "(sm, " + r.pos.str() + ")";
        }
        return "sm[" + buf_index(r.edge, r.pos).str() + "]";
    }
    // cp.async of the input windows of the tile starting at `kexpr` (fused path)
    void emit_issue(std::ostringstream& b, const std::string& kexpr, bool staging) {
        b << "    { // issue loads of the tile at " << kexpr << (staging ? " into the staging region" : "") << "\n"
          << "      const long long kn = " << kexpr << ";\n"
          << "      if (kn < SG_K_END) {\n"
          << "        const int Wn = (int)min((long long)SG_WR, SG_K_END - kn);\n";
        for (size_t i = 0; i < ins_.size(); i++) {
            int e = ins_[i];
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            int64_t P = f_.edges[e].per_iter;
            std::string dst = "s + j";
            auto pit = plP_.find(e);
            if (!staging && pit != plP_.end())
                dst = "s + (j % " + std::to_string(pit->second) + ") * " + std::to_string(plQ_.at(e)) + " + j / " +
                      std::to_string(pit->second);
            if (staging) {
                // 16-byte cp.async over the 16-byte-aligned superset of the window; the
                // misalignment m (items) is kept for the staging -> tile copy; partial
                // quads at the stream ends go item by item with zero fill
                b << "        {\n"
                  << "          const " << T_ << "* g = SG_IN(" << i << ");\n"
                  << "          const long long gb = kn * " << P << "LL + (" << lo << "LL) - SG_IN_BASE(" << i << ");\n"
                  << "          const long long lim = SG_IN_LIMIT(" << i << ");\n"
                  << "          const int n = Wn * " << P << " + " << ex << ";\n"
                  << "          const int m = (int)(((unsigned long long)g / 4ull + (unsigned long long)gb) & 3ull);\n"
                  << "          sg_pm[" << i << "] = m;\n"
                  << "          const long long ga = gb - m;\n"
                  << "          const int nq = (n + m + 3) >> 2;\n"
                  << "          " << T_ << "* s = sm + " << stage_off_.at(e) << ";\n"
                  << "          for (int q = tid; q < nq; q += NT) {\n"
                  << "            const long long gi = ga + 4LL * q;\n"
                  << "            if (gi >= 0 && gi + 3 < lim) sg_cp_async16(s + 4 * q, g + gi);\n"
                  << "            else for (int r = 0; r < 4; r++) { const bool ok = gi + r >= 0 && gi + r < lim;\n"
                  << "              sg_cp_async4(s + 4 * q + r, g + (ok ? gi + r : 0LL), ok ? 4u : 0u); }\n"
                  << "          }\n"
                  << "        }\n";
                continue;
            }
            b << "        {\n"
              << "          const " << T_ << "* g = SG_IN(" << i << ");\n"
              << "          const long long gb = kn * " << P << "LL + (" << lo << "LL) - SG_IN_BASE(" << i << ");\n"
              << "          const long long lim = SG_IN_LIMIT(" << i << ");\n"
              << "          const int n = Wn * " << P << " + " << ex << ";\n"
              << "          " << T_ << "* s = sm + " << off_.at(e) << ";\n"
              << "          for (int j = tid; j < n; j += NT) { const long long gi = gb + j; const bool ok = gi >= 0 && gi < lim;\n"
              << "            sg_cp_async4(" << dst << ", g + (ok ? gi : 0LL), ok ? 4u : 0u); }\n"
              << "        }\n";
        }
        b << "      }\n      sg_cp_async_commit();\n    }\n";
    }
    std::string fused_prologue() const { return prologue_; }
    void emit_loads(std::ostringstream& b) {
        if (fused_ && !ins_.empty()) {
            if (prefetch_) {
                b << "    sg_cp_async_wait_all();\n    __syncthreads();\n";
                for (size_t i = 0; i < ins_.size(); i++) {
                    int e = ins_[i];
                    int64_t lo, ex;
                    edge_window(f_, e, lo, ex);
                    int64_t P = f_.edges[e].per_iter;
                    auto pit = plP_.find(e);
                    std::string dst = "s[j]";
                    if (pit != plP_.end())
                        dst = "s[(j % " + std::to_string(pit->second) + ") * " + std::to_string(plQ_.at(e)) + " + j / " +
                              std::to_string(pit->second) + "]";
                    b << "    { // boundary input " << i << " (edge " << e << "): staging -> tile buffer\n"
                      << "      const int n = Wt * " << P << " + " << ex << ";\n"
                      << "      " << T_ << "* s = sm + " << off_.at(e) << ";\n"
                      << "      const " << T_ << "* st = sm + " << stage_off_.at(e) << " + sg_pm[" << i << "];\n"
                      << "      for (int j = tid; j < n; j += NT) " << dst << " = st[j];\n"
                      << "    }\n";
                }
                b << "    __syncthreads();\n";
                emit_issue(b, "kt + (long long)gridDim.x * SG_WR", true);
            } else {
                emit_issue(b, "k0", false);
                b << "    sg_cp_async_wait_all();\n    __syncthreads();\n";
            }
            return;
        }
        for (size_t i = 0; i < ins_.size(); i++) {
            int e = ins_[i];
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            int64_t P = f_.edges[e].per_iter;
            b << "    { // load boundary input " << i << " (edge " << e << ")\n"
              << "      const " << T_ << "* g = SG_IN(" << i << ");\n"
              << "      const long long gb = k0 * " << P << "LL + (" << lo << "LL) - SG_IN_BASE(" << i << ");\n"
              << "      const long long lim = SG_IN_LIMIT(" << i << ");\n"
              << "      const int n = Wt * " << P << " + " << ex << ";\n"
              << "      " << T_ << "* s = sm + " << off_.at(e) << ";\n";
            auto pit = plP_.find(e);
            std::string dst = "s[j]";
            if (fused_ && pit != plP_.end())
                dst = "s[(j % " + std::to_string(pit->second) + ") * " + std::to_string(plQ_.at(e)) + " + j / " +
                      std::to_string(pit->second) + "]";
            b << "      for (int j = tid; j < n; j += NT) { const long long gi = gb + j; " << dst
              << " = (gi >= 0 && gi < lim) ? g[gi] : (" << T_ << ")0; }\n"
              << "    }\n";
        }
        b << "    __syncthreads();\n";
    }
    // choose a store period PER so that every position resolves statically
    int store_period(int e, int64_t lo) {
        for (int per : {1, 2, 4, 8, 16, 32, 64}) {
            bool ok = true;
            for (int c = 0; c < per && ok; c++) {
                Ref r = R_.resolve(e, Lin::v("q", per, lo + c));
                ok = r.k != Ref::RUNTIME;
                if (ok && r.k == Ref::PHYS && fused_) {
                    try { buf_index(r.edge, r.pos); } catch (const FusedFail&) { ok = false; }
                }
            }
            if (ok) return per;
        }
        return 1;
    }
    void emit_stores(std::ostringstream& b) {
        for (size_t i = 0; i < outs_.size(); i++) {
            int e = outs_[i];
            int64_t lo, ex;
            edge_window(f_, e, lo, ex);
            int64_t P = f_.edges[e].per_iter;
            int per = store_period(e, lo);
            b << "    { // store boundary output " << i << " (edge " << e << ")\n"
              << "      " << T_ << "* g = SG_OUT(" << i << ");\n"
              << "      const long long gb = k0 * " << P << "LL + (" << lo << "LL) - SG_OUT_BASE(" << i << ");\n"
              << "      const int n = Wt * " << P << " + " << ex << ";\n"
              << "      const int nq = (n + " << per - 1 << ") / " << per << ";\n"
              << "      for (int q = tid; q < nq; q += NT) {\n";
            for (int c = 0; c < per; c++) {
                std::string val = read_expr(e, Lin::v("q", per, lo + c));
                b << "        if (" << per << " * q + " << c << " < n) g[gb + " << per << " * q + " << c << "] = " << val
                  << ";\n";
            }
            b << "      }\n";
            b << "    }\n";
        }
    }
    void emit_stage(std::ostringstream& b, int v, int64_t rot) {
        const Node& n = f_.nodes[v];
        int eo = n.out[0];
        int64_t F0 = n.ninit - n.halo;
        int64_t r = rot % NT_;
        b << "    { // " << kind_name(n.kind) << " node " << v << "\n"
          << "      const int nf = " << n.halo << " + Wt * " << n.rep << ";\n"
          << "      const long long gf = k0 * " << n.rep << "LL;\n"
          << "      " << T_ << "* o_ = sm + " << off_.at(eo) << ";\n";
        if (n.kind == SG_K_BEAM_FIR) {
            emit_beam_fir(b, v, F0, r);
        } else if (n.kind == SG_K_FIR && n.iv[0] >= 4 && emit_fir_blocked(b, v, F0, r)) {
        } else {
            b << "      int j = tid - " << r << "; if (j < 0) j += NT;\n"
              << "      for (; j < nf; j += NT) {\n"
              << "        const int lf = " << F0 << " + j;\n";
            emit_firing(b, v, "        ");
            b << "      }\n";
        }
        b << "    }\n";
    }
    // one firing at local index `lf`, output slot j
    void emit_firing(std::ostringstream& b, int v, const std::string& ind) {
        const Node& n = f_.nodes[v];
        b << ind << "if (gf + lf < 0) {";
        for (int64_t jj = 0; jj < n.push; jj++) b << " o_[j * " << n.push << " + " << jj << "] = (" << T_ << ")0;";
        b << " } else {\n";
        b << ind << "  " << T_ << " x_[" << n.peek << "];\n";
        for (int64_t i = 0; i < n.peek; i++)
            b << ind << "  x_[" << i << "] = " << read_expr(n.in[0], Lin::v("lf", n.pop, i)) << ";\n";
        b << ind << "  " << T_ << " y_[" << n.push << "]; " << work_call(v) << "\n";
        for (int64_t jj = 0; jj < n.push; jj++)
            b << ind << "  o_[j * " << n.push << " + " << jj << "] = y_[" << jj << "];\n";
        b << ind << "}\n";
    }
    // Register-blocked FIR: a thread computes B consecutive firings from one
    // window of (B-1)*pop + L inputs held in registers; per output the taps are
    // accumulated in order i = 0..L-1 (the FIR semantics).
    bool emit_fir_blocked(std::ostringstream& b, int v, int64_t F0, int64_t rot) {
        const Node& n = f_.nodes[v];
        int64_t L = n.iv[0], pop = n.pop;
        // probe: positions lf0*pop + k must map to one physical buffer, affine in lf0 and k
        Ref r0 = R_.resolve(n.in[0], Lin::v("lf0", pop, 0));
        Ref r1 = R_.resolve(n.in[0], Lin::v("lf0", pop, 1));
        if (r0.k != Ref::PHYS || r1.k != Ref::PHYS || r0.edge != r1.edge) return false;
        int64_t a = r0.pos.coef("lf0"), s = r1.pos.c - r0.pos.c;
        if (r0.pos.t.size() != (a ? 1u : 0u) || a != pop * s || s == 0) return false;
        int B = 1;
        for (int cand : {9, 7, 5, 3}) {
            if ((cand - 1) * pop + L > 100) continue;
            if (((cand * pop * s) & 1) == 0 && cand != 3) continue;
            B = cand;
            break;
        }
        if (B == 1) return false;
        int64_t NW = (B - 1) * pop + L;
        for (int64_t k = 0; k < NW; k++) {  // verify the whole window is affine
            Ref rk = R_.resolve(n.in[0], Lin::v("lf0", pop, k));
            if (rk.k != Ref::PHYS || rk.edge != r0.edge || rk.pos.coef("lf0") != a || rk.pos.c != r0.pos.c + s * k)
                return false;
        }
        std::string C = const_array(n.fv);
        int64_t base = off_.at(r0.edge) - wb_.at(r0.edge) + r0.pos.c;
        b << "      const int nb = (nf + " << B - 1 << ") / " << B << ";\n"
          << "      int jb = tid - " << rot % NT_ << "; if (jb < 0) jb += NT;\n"
          << "      for (; jb < nb; jb += NT) {\n"
          << "        const int j0 = jb * " << B << ";\n"
          << "        const int lf0 = " << F0 << " + j0;\n"
          << "        if (j0 + " << B << " <= nf && gf + lf0 >= 0) {\n"
          << "          const " << T_ << "* w_ = sm + (" << base << " + " << a << " * lf0);\n"
          << "          float w[" << NW << "];\n"
          << "#pragma unroll\n"
          << "          for (int k = 0; k < " << NW << "; k++) w[k] = w_[k * " << s << "];\n"
          << "          float acc[" << B << "];\n"
          << "#pragma unroll\n"
          << "          for (int bb = 0; bb < " << B << "; bb++) acc[bb] = 0.0f;\n"
          << "#pragma unroll\n"
          << "          for (int i = 0; i < " << L << "; i++) {\n"
          << "            const float c = " << C << "[i];\n"
          << "#pragma unroll\n"
          << "            for (int bb = 0; bb < " << B << "; bb++) acc[bb] = fmaf(w[bb * " << pop << " + i], c, acc[bb]);\n"
          << "          }\n"
          << "#pragma unroll\n"
          << "          for (int bb = 0; bb < " << B << "; bb++) o_[j0 + bb] = acc[bb];\n"
          << "        } else {\n"
          << "          for (int j = j0; j < min(j0 + " << B << ", nf); j++) {\n"
          << "            const int lf = " << F0 << " + j;\n";
        emit_firing(b, v, "            ");
        b << "          }\n        }\n      }\n";
        return true;
    }
    // Frame-granular complex FIR: items = (firing, block of B outputs); taps in
    // chunks of TC with the sample window in registers; x[s<0] = 0.
    // Frame-granular complex FIR: items = (firing, block of B consecutive outputs);
    // taps in chunks of TC with the sample window in registers; x[s<0] = 0.
    // B odd (lanes 3/5/7.. samples apart hit distinct banks of planar buffers),
    // chosen with the other frame FIRs of the same level to avoid straggler
    // rounds; interior chunks skip the boundary checks; short filters are fully
    // unrolled so coefficients become immediates.
    std::map<int, int64_t> beam_B_;
    std::map<int, bool> beam_pair_, beam_f2_;
    // chunks of TC taps a block of B outputs starting at output t0 runs: taps whose
    // window lies wholly before the frame start (x = 0) are skipped -- exact, the
    // accumulators start at +0 and adding +-0 never changes them (reading 14)
    static int64_t beam_chunks(int64_t t0, int64_t B, int64_t DEC, int64_t L, int64_t TC) {
        int64_t lim = std::min<int64_t>(L, (t0 + B - 1) * DEC + 1);
        return (lim + TC - 1) / TC;
    }
    static int64_t beam_tc(int64_t L) {
        for (int64_t c : {16, 8, 4, 2, 1})
            if (L % c == 0) return c;
        return 1;
    }
    // Block size B (odd: lanes B samples apart hit distinct banks of the planar
    // buffers) and pairing (an item runs blocks p and NB-1-p, so the triangular work
    // of long filters -- few live taps early in the frame -- is even per item),
    // chosen by simulating the round-robin assignment of all peer items of the level
    // to the CTA's threads and minimising the busiest thread's issue slots.
    int64_t beam_block(int v, int64_t W) {
        auto it = beam_B_.find(v);
        if (it != beam_B_.end()) return it->second;
        const Node& n = f_.nodes[v];
        int64_t peers = 0;
        for (int u : nodes_)
            if (compute_node(u) && special(u) && f_.nodes[u].iv == n.iv && level_of_special(u) == level_of_special(v)) peers++;
        const int64_t OUT = n.iv[2] / n.iv[1], L = n.iv[0], DEC = n.iv[1], TC = beam_tc(L);
        const int64_t nf = n.halo + W * n.rep;
        int64_t best = 3;
        bool bestp = false, bestf2 = false;
        double bestc = 1e300;
        const bool dynsched = fused_ && !std::getenv("SG_STATIC_ITEMS");
        // FFMA2 mode (fused, dynamic scheduling, coefficient table): a thread runs blocks
        // blk and blk + 32 as the two halves of packed fp32x2 FMAs (Blackwell FFMA2)
        if (dynsched && std::getenv("SG_FFMA2") && L % 2 == 0 && NT_ <= 512)
            for (int64_t B : {1, 3, 5}) {
                const int64_t NB = (OUT + B - 1) / B, NBH = (NB + 63) / 64 * 32;
                const int64_t NWIN = (B - 1) * DEC + beam_tc(L);
                double sum = 0, mx = 0;
                for (int64_t q = 0; q < NBH; q++) {
                    const int64_t a = q / 32 * 64 + q % 32, bb = std::min(a + 32, NB - 1);
                    const int64_t ch = beam_chunks(bb * B, B, DEC, L, TC);
                    const double c = (double)ch * ((double)TC * B * 4 + 4.0 * NWIN + TC / 2.0 + 8) + 8.0 * B + 16;
                    sum += c;
                    mx = std::max(mx, c);
                }
                sum *= (double)peers * nf;
                const double cost = std::max(sum / NT_, mx) + mx * 0.5;
                if (cost < bestc * 0.98) { bestc = cost; best = B; bestp = false; bestf2 = true; }
            }
        for (int64_t B : {1, 3, 5, 7, 9})
            for (bool pair : {false, true}) {
                const int64_t NB = (OUT + B - 1) / B, NBP = pair ? (NB + 1) / 2 : NB;
                const int64_t NWIN = (B - 1) * DEC + TC;
                auto blk_cost = [&](int64_t blk) {
                    int64_t ch = beam_chunks(blk * B, B, DEC, L, TC);
                    return (double)ch * ((double)TC * B * 4 + 2.0 * NWIN + TC / 2.0 + 8) + 4.0 * B + 12;
                };
                std::vector<double> per(NBP);
                for (int64_t q = 0; q < NBP; q++) {
                    per[q] = blk_cost(q);
                    if (pair && NB - 1 - q != q) per[q] += blk_cost(NB - 1 - q);
                }
                const int64_t items = peers * nf * NBP;
                double cost = 0;
                if (fused_ && !std::getenv("SG_STATIC_ITEMS")) {
                    // dynamic scheduling: warps take 32-item chunks until the level is done
                    double sum = 0, mx = 0;
                    for (int64_t k = 0; k < items; k++) { sum += per[k % NBP]; mx = std::max(mx, per[k % NBP]); }
                    cost = std::max(sum / NT_, mx) + mx * 0.5;
                } else {
                    std::vector<double> th(std::min<int64_t>(NT_, items), 0.0);
                    for (int64_t k = 0; k < items; k++) th[k % NT_] += per[k % NBP];
                    for (double c : th) cost = std::max(cost, c);
                }
                if (cost < bestc * 0.98) { bestc = cost; best = B; bestp = pair; bestf2 = false; }
            }
        beam_B_[v] = best;
        beam_pair_[v] = bestp;
        beam_f2_[v] = bestf2;
        return best;
    }
    // fused level of a node of the partition: compute nodes their level, views the largest level of the
    // compute nodes feeding them (a cut at a level boundary is then convex)
    int node_level_of(int u) {
        const Node& n = f_.nodes[u];
        if (compute_node(u)) return level_.count(u) ? level_.at(u) : 0;
        int L = 0;
        for (int e : n.in) {
            std::set<int> src;
            R_.sources(e, src);
            for (int pe : src) {
                const int s = f_.edges[pe].src;
                if (s >= 0 && std::find(nodes_.begin(), nodes_.end(), s) != nodes_.end() && compute_node(s))
                    L = std::max(L, level_.count(s) ? level_.at(s) : 0);
            }
        }
        return L;
    }
    std::map<int, int> special_level_;
    int level_of_special(int v) {
        auto it = special_level_.find(v);
        if (it != special_level_.end()) return it->second;
        int L = level_.count(v) ? level_.at(v) : 0;
        for (auto& g : fg_)
            for (int r : g.roots)
                if (r == v) L = g.level;
        special_level_[v] = L;
        return L;
    }
    // peers: frame FIRs with identical parameters whose reads/writes differ only by a
    // constant offset; one body serves all of them (item -> peer, firing, block).
    bool beam_peer_offsets(const std::vector<int>& peers, std::vector<int64_t>& din, std::vector<int64_t>& dout) {
        const Node& n0 = f_.nodes[peers[0]];
        const int64_t L = n0.iv[0], DEC = n0.iv[1], TC = 16, B = 9;
        const int64_t NWIN = (B - 1) * DEC + TC;
        din.assign(peers.size(), 0);
        dout.assign(peers.size(), 0);
        for (size_t q = 0; q < peers.size(); q++) {
            const Node& n = f_.nodes[peers[q]];
            if (n.iv != n0.iv || n.fv != n0.fv || n.halo != n0.halo || n.ninit != n0.ninit || n.rep != n0.rep) return false;
            for (int64_t k = 0; k < NWIN; k += NWIN - 1)
                for (int r = 0; r < 2; r++) {
                    Lin pr = Lin::v("lf", n.pop, 2 * k + r);
                    pr.t.push_back({"s0", 2});
                    Lin p0 = pr;
                    Ref a = R_.resolve(n0.in[0], p0), c = R_.resolve(n.in[0], pr);
                    if (a.k != Ref::PHYS || c.k != Ref::PHYS) return false;
                    Lin ia = buf_index(a.edge, a.pos), ic = buf_index(c.edge, c.pos);
                    if (ia.vars() != ic.vars()) return false;
                    int64_t d = ic.c - ia.c;
                    if (k == 0 && r == 0) din[q] = d;
                    else if (d != din[q]) return false;
                }
            Lin pos = Lin::v("j", n.push, f_.edges[n.out[0]].pre + (n.ninit - n.halo) * n.push);
            pos.t.push_back({"(t0 + bb)", 2});
            Lin oa = buf_index(n0.out[0], pos), oc = buf_index(n.out[0], pos);
            Lin oa1 = buf_index(n0.out[0], pos.plus(1)), oc1 = buf_index(n.out[0], pos.plus(1));
            if (oa.vars() != oc.vars() || oc.c - oa.c != oc1.c - oa1.c) return false;
            dout[q] = oc.c - oa.c;
            (void)L;
        }
        return true;
    }
    // FFMA2 variant of the frame FIR: item = (peer, frame, slot q); the thread computes the
    // B-output blocks a = (q / 32) * 64 + q % 32 and a + 32 together, the two halves of
    // packed fp32x2 registers: every tap is 4 FFMA2 (= the 8 fmaf of two sg_cmac, same
    // order, same rounding) with the coefficient broadcast from the shared table.  Lanes
    // stay B samples apart (odd B: distinct banks); chunks run to block a+32's triangle
    // limit, block a's extra taps read zeros (exact, reading 14).
    static std::string subst_s0(const std::string& e, const std::string& to) {
        std::string r;
        for (size_t i = 0; i < e.size();) {
            if (e.compare(i, 2, "s0") == 0 && (i == 0 || !(isalnum((unsigned char)e[i - 1]) || e[i - 1] == '_')) &&
                (i + 2 >= e.size() || !(isalnum((unsigned char)e[i + 2]) || e[i + 2] == '_'))) {
                r += to;
                i += 2;
            } else {
                r += e[i++];
            }
        }
        return r;
    }
    void emit_beam_fir_f2(std::ostringstream& b, int v, int64_t F0, int64_t NP, const std::string& DINT,
                          const std::string& DOUTT, int64_t ctoff) {
        const Node& n = f_.nodes[v];
        const int64_t L = n.iv[0], DEC = n.iv[1], FR = n.iv[2], OUT = FR / DEC;
        const int64_t TC = beam_tc(L), B = beam_B_[v];
        const int64_t NB = (OUT + B - 1) / B, NBH = (NB + 63) / 64 * 32, NWIN = (B - 1) * DEC + TC;
        const int slot = nctr_++;
        b << "      const int items = nf * " << NBH * NP << ";\n"
          << "      for (int it0 = 0;;) {\n"
          << "        if ((tid & 31) == 0) it0 = atomicAdd(&sg_ctr[" << slot << "], 32);\n"
          << "        it0 = __shfl_sync(0xffffffffu, it0, 0);\n"
          << "        if (it0 >= items) break;\n"
          << "        const int it = it0 + (tid & 31);\n"
          << "        if (it < items) {\n"
          << "        const int pq = it / (nf * " << NBH << ");\n"
          << "        const int itp = it - pq * (nf * " << NBH << ");\n"
          << "        const int j = itp / " << NBH << ";\n"
          << "        const int q = " << NBH - 1 << " - (itp - j * " << NBH << ");  // longest first\n"
          << "        const int blka = (q >> 5) * 64 + (q & 31), blkb = blka + 32;\n"
          << "        const int t0 = blka * " << B << ", t0b = blkb * " << B << ";\n"
          << "        const int ilim = min(" << L << ", (t0b + " << B - 1 << ") * " << DEC << " + 1);\n"
          << "        const int lf = " << F0 << " + j;\n"
          << "        " << T_ << "* smi = sm + " << (NP > 1 ? DINT + "[pq]" : std::string("0")) << ";\n"
          << "        " << T_ << "* smo = sm + " << (NP > 1 ? DOUTT + "[pq]" : std::string("0")) << ";\n"
          << "        (void)pq; (void)smi; (void)smo;\n"
          << "        float2 RE[" << B << "], IM[" << B << "];\n"
          << "#pragma unroll\n"
          << "        for (int bb = 0; bb < " << B << "; bb++) { RE[bb] = make_float2(0.0f, 0.0f); IM[bb] = RE[bb]; }\n"
          << "        if (gf + lf >= 0) {\n"
          << "#pragma unroll 1\n"
          << "          for (int i0 = 0; i0 < ilim; i0 += " << TC << ") {\n"
          << "            const int s0 = t0 * " << DEC << " - i0 - " << TC - 1 << ";\n"
          << "            const int s0b = t0b * " << DEC << " - i0 - " << TC - 1 << ";\n"
          << "            float2 XR[" << NWIN << "], XI[" << NWIN << "];\n"
          << "            if (s0 >= 0 && s0b + " << NWIN - 1 << " < " << FR << ") {\n";
        auto window = [&](bool checked) {
            for (int64_t k = 0; k < NWIN; k++) {
                Lin pr = Lin::v("lf", n.pop, 2 * k);
                pr.t.push_back({"s0", 2});
                Lin pi = pr.plus(1);
                std::string er = "smi" + read_expr(n.in[0], pr).substr(2), ei = "smi" + read_expr(n.in[0], pi).substr(2);
                std::string erb = subst_s0(er, "s0b"), eib = subst_s0(ei, "s0b");
                if (checked)
                    b << "              { const bool oa = s0 + " << k << " >= 0 && s0 + " << k << " < " << FR
                      << ", ob = s0b + " << k << " >= 0 && s0b + " << k << " < " << FR << ";\n"
                      << "                XR[" << k << "] = make_float2(oa ? " << er << " : 0.0f, ob ? " << erb << " : 0.0f);\n"
                      << "                XI[" << k << "] = make_float2(oa ? " << ei << " : 0.0f, ob ? " << eib << " : 0.0f); }\n";
                else
                    b << "              XR[" << k << "] = make_float2(" << er << ", " << erb << "); XI[" << k << "] = make_float2(" << ei
                      << ", " << eib << ");\n";
            }
        };
        window(false);
        b << "            } else {\n";
        window(true);
        b << "            }\n"
          << "#pragma unroll\n"
          << "            for (int ii = 0; ii < " << TC << "; ii += 2) {\n"
          << "              const float4 c4 = reinterpret_cast<const float4*>(sm + " << ctoff << ")[(i0 + ii) >> 1];\n"
          << "              const float2 cr0 = make_float2(c4.x, c4.x), ci0 = make_float2(c4.y, c4.y);\n"
          << "              const float2 cr1 = make_float2(c4.z, c4.z), ci1 = make_float2(c4.w, c4.w);\n"
          << "#pragma unroll\n"
          << "              for (int bb = 0; bb < " << B << "; bb++) {\n"
          << "                const int k = bb * " << DEC << " - ii + " << TC - 1 << ";\n"
          << "                RE[bb] = __ffma2_rn(XR[k], cr0, RE[bb]);\n"
          << "                RE[bb] = __ffma2_rn(make_float2(-XI[k].x, -XI[k].y), ci0, RE[bb]);\n"
          << "                IM[bb] = __ffma2_rn(XR[k], ci0, IM[bb]);\n"
          << "                IM[bb] = __ffma2_rn(XI[k], cr0, IM[bb]);\n"
          << "              }\n"
          << "#pragma unroll\n"
          << "              for (int bb = 0; bb < " << B << "; bb++) {\n"
          << "                const int k = bb * " << DEC << " - ii + " << TC - 2 << ";\n"
          << "                RE[bb] = __ffma2_rn(XR[k], cr1, RE[bb]);\n"
          << "                RE[bb] = __ffma2_rn(make_float2(-XI[k].x, -XI[k].y), ci1, RE[bb]);\n"
          << "                IM[bb] = __ffma2_rn(XR[k], ci1, IM[bb]);\n"
          << "                IM[bb] = __ffma2_rn(XI[k], cr1, IM[bb]);\n"
          << "              }\n"
          << "            }\n"
          << "          }\n"
          << "        }\n";
        const int eo = n.out[0];
        Lin pos = Lin::v("j", n.push, f_.edges[eo].pre + F0 * n.push);
        pos.t.push_back({"(t0 + bb)", 2});
        Lin posb = Lin::v("j", n.push, f_.edges[eo].pre + F0 * n.push);
        posb.t.push_back({"(t0b + bb)", 2});
        b << "#pragma unroll\n"
          << "        for (int bb = 0; bb < " << B << "; bb++) {\n"
          << "          if (t0 + bb < " << OUT << ") {\n"
          << "            smo[" << buf_index(eo, pos).str() << "] = RE[bb].x;\n"
          << "            smo[" << buf_index(eo, pos.plus(1)).str() << "] = IM[bb].x;\n"
          << "          }\n"
          << "          if (blkb < " << NB << " && t0b + bb < " << OUT << ") {\n"
          << "            smo[" << buf_index(eo, posb).str() << "] = RE[bb].y;\n"
          << "            smo[" << buf_index(eo, posb.plus(1)).str() << "] = IM[bb].y;\n"
          << "          }\n"
          << "        }\n"
          << "        }\n"
          << "      }\n";
    }
    // ---- sliding-window frame FIR (fused kernels; the default, SG_BEAM_NOSLIDE=1 restores the chunked form)
    // An item is (peer, firing, block of B consecutive outputs t0..t0+B-1).  At tap i output t0+b reads
    // sample (t0+b)*DEC - i, so from one tap to the next the lane needs ONE new sample (per plane): the
    // window lives in R registers per plane, sample S0 + rel (S0 = t0*DEC - i0, i0 = first tap of an
    // R-tap group) in slot rel mod R -- compile-time slots, no register moves.  Per tap and lane: 4B FFMA,
    // 2 scalar shared loads (re, im; lanes B*DEC samples apart), one constant-cache coefficient pair.
    // Taps run i = 0..L-1 per output in the FIR's order (bit-identical to the chunked form); groups past
    // the block's triangle limit (x[s < 0] = 0, reading 14) are skipped, so L % R == 0.
    struct BeamSlide { int64_t B = 0, R = 0, PF = 2; bool pair = false; double cost = 0, ideal = 0; };
    std::map<int, BeamSlide> beam_slide_;
    static bool beam_slide_on() { return std::getenv("SG_BEAM_NOSLIDE") == nullptr; }
    BeamSlide beam_slide_cfg(int v) {
        auto it = beam_slide_.find(v);
        if (it != beam_slide_.end()) return it->second;
        const Node& n = f_.nodes[v];
        int64_t peers = 0;
        for (int u : nodes_)
            if (compute_node(u) && special(u) && f_.nodes[u].iv == n.iv && level_of_special(u) == level_of_special(v)) peers++;
        const int64_t L = n.iv[0], DEC = n.iv[1], OUT = n.iv[2] / n.iv[1];
        const int64_t nf = n.halo + (int64_t)W_ * n.rep;
        const int64_t nwarps = std::max(1, NT_ / 32);
        BeamSlide best;
        double bestc = 1e300;
        // A/B override: SG_BEAM_B="level/B,level/B" (odd B) for the frame FIRs of the given fused levels
        int64_t bforce = 0;
        if (const char* e = std::getenv("SG_BEAM_B")) {
            const std::string sp(e);
            const int lv = level_of_special(v);
            for (size_t p = 0; p < sp.size();) {
                size_t q = sp.find(',', p);
                if (q == std::string::npos) q = sp.size();
                const std::string tok = sp.substr(p, q - p);
                const size_t c = tok.find('/');
                // "level/B", or "t<taps>x<dec>/B" for every frame FIR of that shape
                const bool shape = !tok.empty() && tok[0] == 't';
                const std::string key = tok.substr(shape ? 1 : 0, c == std::string::npos ? 0 : c - (shape ? 1 : 0));
                const bool hit = shape ? key == std::to_string(n.iv[0]) + "x" + std::to_string(n.iv[1])
                                       : std::atoi(key.c_str()) == lv;
                if (c != std::string::npos && hit) bforce = std::atoll(tok.c_str() + c + 1);
                p = q + 1;
            }
        }
        for (int64_t B = 1; B <= 15; B += 2) {
            if (bforce && B != bforce) continue;
            BeamSlide c;
            c.B = B;
            static const int64_t pf_env = std::getenv("SG_BEAM_PF") ? std::atoll(std::getenv("SG_BEAM_PF")) : 0;
            if (pf_env > 0) c.PF = pf_env;
            for (int64_t R : {4, 8, 16, 32})
                if (R >= (B - 1) * DEC + c.PF + 1 && L % R == 0) { c.R = R; break; }
            if (c.R == 0 || 2 * c.R + 2 * B > (NT_ <= 512 ? 104 : 44)) continue;  // register budget
            for (bool pair : {false, true}) {
                const int64_t NB = (OUT + B - 1) / B, NBP = pair ? (NB + 1) / 2 : NB;
                auto blk_cost = [&](int64_t blk) {
                    int64_t lim = std::min<int64_t>(L, (blk * B + B - 1) * DEC + 1);
                    lim = std::min<int64_t>(L, (lim + c.R - 1) / c.R * c.R);
                    return (double)lim * (4.0 * B + 3.5) + 4.0 * B + 40.0;
                };
                std::vector<double> per(NBP);
                for (int64_t q = 0; q < NBP; q++) {
                    const int64_t blk = pair ? q : NB - 1 - q;  // longest first
                    per[q] = blk_cost(blk);
                    if (pair && NB - 1 - q != q) per[q] += blk_cost(NB - 1 - q);
                }
                // dynamic scheduling: warps take 32 consecutive items; list-schedule the chunks
                const int64_t items = peers * nf * NBP;
                std::vector<double> wl(nwarps, 0.0);
                for (int64_t k0 = 0; k0 < items; k0 += 32) {
                    double cmax = 0;
                    for (int64_t k = k0; k < std::min(items, k0 + 32); k++)
                        cmax = std::max(cmax, per[pair ? k / (peers * nf) : k % NBP]);  // item order as emitted
                    *std::min_element(wl.begin(), wl.end()) += cmax;
                }
                // a warp issues at most one instruction per cycle; warp w shares scheduler w % 4,
                // which needs about four busy warps to hide the FFMA / shared-load latencies (measured on
                // BeamFormer's matched filter: B = 1 over 16 warps beats B = 3 over 11, 2.37 vs 2.59 ms)
                // (co-resident CTAs of the same kernel -- shared memory permitting -- add their warps)
                const double ctas = (double)std::max(1, std::min(2, (int)((220 * 1024) / std::max<size_t>(1024, smem_bytes_))));
                double cost = *std::max_element(wl.begin(), wl.end());
                for (int s = 0; s < 4; s++) {
                    double t = 0;
                    int busy = 0;
                    for (int64_t w = s; w < nwarps; w += 4) { t += wl[w]; busy += wl[w] > 0; }
                    cost = std::max(cost, t / std::min(1.0, busy * ctas / 4.0));
                }
                if (cost < bestc * 0.98) { bestc = cost; best = c; best.pair = pair; best.cost = cost; }
            }
        }
        // the level's pure FFMA issue (live taps, 4 FFMA per complex tap, 32 lanes, 4 schedulers): the
        // parallel efficiency ideal / cost feeds the PEE (pee_refine) and the planner's level split
        double taps = 0;
        for (int64_t t = 0; t < OUT; t++) taps += (double)std::min<int64_t>(L, t * DEC + 1);
        best.ideal = taps * 4.0 * (double)(peers * nf) / 128.0;
        beam_slide_[v] = best;
        return best;
    }
    std::map<std::vector<float>, std::string> beam_ct_;
    std::string beam_const_table(const Node& n) {
        auto it = beam_ct_.find(n.fv);
        if (it != beam_ct_.end()) return it->second;
        const int64_t L = n.iv[0];
        std::string nm = "SG_CTS" + std::to_string(nvar_++);
        consts_ << "__constant__ float2 " << nm << "[" << L << "] = {";
        for (int64_t i = 0; i < L; i++)
            consts_ << (i ? ", " : "") << "{" << hexf(n.fv[i]) << ", " << hexf(n.fv[L + i]) << "}";
        consts_ << "};\n";
        beam_ct_[n.fv] = nm;
        return nm;
    }
    std::map<std::vector<float>, std::string> beam_cq_;
    std::string beam_const_table4(const Node& n) {  // per tap {wr, wi, -wi, wr}: the two FFMA2 coefficient pairs
        auto it = beam_cq_.find(n.fv);
        if (it != beam_cq_.end()) return it->second;
        const int64_t L = n.iv[0];
        std::string nm = "SG_CTQ" + std::to_string(nvar_++);
        consts_ << "__constant__ float4 " << nm << "[" << L << "] = {";
        for (int64_t i = 0; i < L; i++)
            consts_ << (i ? ", " : "") << "{" << hexf(n.fv[i]) << ", " << hexf(n.fv[L + i]) << ", " << hexf(-n.fv[L + i])
                    << ", " << hexf(n.fv[i]) << "}";
        consts_ << "};\n";
        beam_cq_[n.fv] = nm;
        return nm;
    }
    void emit_beam_fir_slide(std::ostringstream& b, int v, int64_t F0, int64_t rot, int64_t NP, const std::string& DINT,
                             const std::string& DOUTT) {
        const Node& n = f_.nodes[v];
        // packed complex MACs: (re, im) as one float2, per tap two FFMA2 with the sample broadcast --
        // (re, im) += xr * (wr, wi), then (re, im) += xi * (-wi, wr): lane by lane the fmaf sequence of sg_cmac
        // (xi * -wi is exactly -(xi * wi)), so bit-identical; half the FMA instructions.  Opt-in (SG_BEAM_FFMA2=1):
        // in the bench's step it measured slower (BeamFormer 1.707 -> 2.016 ms; the packed chains' longer latency
        // with one or two warps per scheduler), although each kernel timed alone looked faster.
        static const bool f2 = std::getenv("SG_BEAM_FFMA2") && std::atoi(std::getenv("SG_BEAM_FFMA2")) != 0;
        const int64_t L = n.iv[0], DEC = n.iv[1], FR = n.iv[2], OUT = FR / DEC;
        const BeamSlide cfg = beam_slide_cfg(v);
        const int64_t B = cfg.B, R = cfg.R, PF = cfg.PF;
        const int64_t NB = (OUT + B - 1) / B, NBP = cfg.pair ? (NB + 1) / 2 : NB;
        static const bool ct_smem = std::getenv("SG_BEAM_CT_SMEM") != nullptr;
        auto ct = ctab_off_.find(v);
        std::string coef;  // expression of the (cr, ci) pair of tap `i0 + u`
        if (ct_smem && ct != ctab_off_.end())
            coef = "reinterpret_cast<const float2*>(sm + " + std::to_string(ct->second) + ")";
        else
            coef = beam_const_table(n);
        auto slot = [&](int64_t rel) { return ((rel % R) + R) % R; };
        auto sample = [&](int64_t rel, bool im, const std::string& var) {  // shared-memory read of sample var + rel
            Lin p = Lin::v("lf", n.pop, 2 * rel + (im ? 1 : 0));
            p.t.push_back({var, 2});
            return "smi" + read_expr(n.in[0], p).substr(2);
        };
        b << "      const int items = nf * " << NBP * NP << ";  // sliding window: B = " << B << ", R = " << R
          << (cfg.pair ? ", paired blocks" : "") << "\n";
        // Every lane of a warp runs the same tap groups (trip count = the warp's largest triangle limit;
        // a lane's extra taps read x[s < 0] = 0, exact by DESIGN.md reading 14), so the tap index is
        // warp-uniform: the coefficient pair is a uniform-register operand of the FFMAs (LDCU), not a
        // third vector register.  Items past the end are clamped to a valid one and not stored.
        const int slot_c = nctr_++;
        (void)rot;
        b << "      for (int it0 = 0;;) {\n"
          << "        if ((tid & 31) == 0) it0 = atomicAdd(&sg_ctr[" << slot_c << "], 32);\n"
          << "        it0 = __shfl_sync(0xffffffffu, it0, 0);\n"
          << "        if (it0 >= items) break;\n"
          << "        const int itr = it0 + (tid & 31);\n"
          << "        const bool valid = itr < items;\n"
          << "        const int it = valid ? itr : items - 1;\n";
        // paired blocks (long triangular filters): block-pair-major order, so the lanes of a warp run pairs
        // of nearly equal triangle limits (the warp's trip count is its largest limit)
        static const bool pmajor = std::getenv("SG_BEAM_PMAJOR") ? std::atoi(std::getenv("SG_BEAM_PMAJOR")) != 0 : true;
        if (cfg.pair && pmajor)
            b << "        const int pb = it / (nf * " << NP << ");\n"
              << "        const int itq = it - pb * (nf * " << NP << ");\n"
              << "        const int pq = itq / nf;\n"
              << "        const int j = itq - pq * nf;\n";
        else
            b << "        const int pq = it / (nf * " << NBP << ");\n"
              << "        const int itp = it - pq * (nf * " << NBP << ");\n"
              << "        const int j = itp / " << NBP << ";\n"
              << "        const int pb = itp - j * " << NBP << ";\n";
        b
          << "        const int lf = " << F0 << " + j;\n"
          << "        const bool live = valid && gf + lf >= 0;  // firings before the stream start emit zeros\n"
          << "        " << T_ << "* smi = sm + " << (NP > 1 ? DINT + "[pq]" : std::string("0")) << ";\n"
          << "        " << T_ << "* smo = sm + " << (NP > 1 ? DOUTT + "[pq]" : std::string("0")) << ";\n"
          << "        (void)pq; (void)smi; (void)smo;\n";
        if (cfg.pair)
            b << "#pragma unroll 1\n"
              << "        for (int half = 0; half < 2; half++) {\n"
              << "        const int blk = half ? " << NB - 1 << " - pb : pb;\n"
              << "        const bool hs = valid && !(half && blk == pb), hv = hs && live;\n";
        else
            b << "        { const int blk = " << NB - 1 << " - pb;  // longest first\n"
              << "        const bool hs = valid, hv = live;\n";
        b << "        const int t0 = blk * " << B << ";\n"
          << "        const int S0 = t0 * " << DEC << ";\n"
          << "        const int ilim = min(" << L << ", (min(" << L << ", S0 + " << (B - 1) * DEC << " + 1) + " << R - 1
          << ") / " << R << " * " << R << ");\n"
          << "        const int ilimw = __reduce_max_sync(0xffffffffu, hv ? ilim : 0);\n"
          << (f2 ? "        float2 ac[" + std::to_string(B) + "];\n" : "        float re[" + std::to_string(B) + "], im[" +
                                                                          std::to_string(B) + "];\n");
        for (int64_t bb = 0; bb < B; bb++)
            b << (f2 ? "        ac[" + std::to_string(bb) + "] = make_float2(0.0f, 0.0f);\n"
                     : "        re[" + std::to_string(bb) + "] = 0.0f; im[" + std::to_string(bb) + "] = 0.0f;\n");
        b << "        {\n"
          << "          float xr[" << R << "], xi[" << R << "];\n";
        // prologue: rel in [-(PF-1), (B-1)*DEC] relative to S0
        auto prologue = [&](bool checked) {
            for (int64_t rel = -(PF - 1); rel <= (B - 1) * DEC; rel++) {
                const int64_t s = slot(rel);
                if (checked)
                    b << "            { const int s = S0 + " << rel << "; const bool ok = s >= 0 && s < " << FR << ";\n"
                      << "              xr[" << s << "] = ok ? " << sample(rel, false, "S0") << " : 0.0f;\n"
                      << "              xi[" << s << "] = ok ? " << sample(rel, true, "S0") << " : 0.0f; }\n";
                else
                    b << "            xr[" << s << "] = " << sample(rel, false, "S0") << "; xi[" << s << "] = "
                      << sample(rel, true, "S0") << ";\n";
            }
        };
        // guard decisions are warp-uniform too (one lane near the frame start would otherwise split the warp
        // into a serialised few-lane pass over the guarded copy; the guarded copy is exact for every lane)
        b << "          if (__all_sync(0xffffffffu, S0 - " << PF - 1 << " >= 0 && S0 + " << (B - 1) * DEC << " < " << FR
          << ")) {\n";
        prologue(false);
        b << "          } else {\n";
        prologue(true);
        b << "          }\n"
          << "#pragma unroll 1\n"
          << "          for (int i0 = 0; i0 < ilimw; i0 += " << R << ") {\n"
          << "            const int sb = S0 - i0;\n";
        auto body = [&](bool checked) {
            for (int64_t u = 0; u < R; u++) {
                const int64_t rl = -(u + PF), sl = slot(rl);
                if (f2)
                    b << "            { const float4 c4 = " << beam_const_table4(n) << "[i0 + " << u << "];\n"
                      << "              const float2 ca = make_float2(c4.x, c4.y), cb = make_float2(c4.z, c4.w);\n";
                else
                    b << "            { const float2 c = " << coef << "[i0 + " << u << "];\n";
                if (checked)
                    b << "              { const bool ok = sb - " << u + PF << " >= 0;\n"
                      << "                xr[" << sl << "] = ok ? " << sample(rl, false, "sb") << " : 0.0f;\n"
                      << "                xi[" << sl << "] = ok ? " << sample(rl, true, "sb") << " : 0.0f; }\n";
                else
                    b << "              xr[" << sl << "] = " << sample(rl, false, "sb") << "; xi[" << sl << "] = "
                      << sample(rl, true, "sb") << ";\n";
                for (int64_t bb = 0; bb < B; bb++) {
                    const int64_t s = slot(bb * DEC - u);
                    if (f2)
                        b << "              ac[" << bb << "] = __ffma2_rn(make_float2(xr[" << s << "], xr[" << s << "]), ca, ac["
                          << bb << "]); ac[" << bb << "] = __ffma2_rn(make_float2(xi[" << s << "], xi[" << s << "]), cb, ac["
                          << bb << "]);\n";
                    else
                        b << "              sg_cmac(re[" << bb << "], im[" << bb << "], xr[" << s << "], xi[" << s
                          << "], c.x, c.y);\n";
                }
                b << "            }\n";
            }
        };
        b << "            if (__all_sync(0xffffffffu, sb - " << R - 1 + PF << " >= 0)) {\n";
        body(false);
        b << "            } else {\n";
        body(true);
        b << "            }\n"
          << "          }\n"
          << "        }\n";
        const int eo = n.out[0];
        Lin pos = Lin::v("j", n.push, f_.edges[eo].pre + F0 * n.push);
        pos.t.push_back({"(t0 + bb)", 2});
        b << "        if (hs) {\n"
          << "#pragma unroll\n"
          << "        for (int bb = 0; bb < " << B << "; bb++)\n"
          << "          if (t0 + bb < " << OUT << ") {\n"
          << "            smo[" << buf_index(eo, pos).str() << "] = hv ? " << (f2 ? "ac[bb].x" : "re[bb]") << " : 0.0f;\n"
          << "            smo[" << buf_index(eo, pos.plus(1)).str() << "] = hv ? " << (f2 ? "ac[bb].y" : "im[bb]") << " : 0.0f;\n"
          << "          }\n"
          << "        }\n"
          << "        }\n"
          << "      }\n";
    }
    void emit_beam_fir(std::ostringstream& b, int v, int64_t F0, int64_t rot, const std::vector<int>& peers = {},
                       const std::vector<int64_t>& din = {}, const std::vector<int64_t>& dout = {}) {
        const Node& n = f_.nodes[v];
        const int64_t NP = peers.empty() ? 1 : (int64_t)peers.size();
        int64_t L = n.iv[0], DEC = n.iv[1], FR = n.iv[2], OUT = FR / DEC;
        const int64_t TC = beam_tc(L);
        const int64_t B = beam_block(v, W_);
        const bool pair = beam_pair_[v];
        int64_t NB = (OUT + B - 1) / B, NWIN = (B - 1) * DEC + TC;
        const int64_t NBP = pair ? (NB + 1) / 2 : NB;
        auto ct = ctab_off_.find(v);
        const bool ctab = fused_ && ct != ctab_off_.end() && TC % 2 == 0;
        const bool unroll = false;  // rolled tap loop: small code (I-cache) beats immediates here
        std::vector<float> wr(n.fv.begin(), n.fv.begin() + L), wi(n.fv.begin() + L, n.fv.end());
        std::string WR = unroll ? "" : const_array(wr), WI = unroll ? "" : const_array(wi);
        std::string DINT, DOUTT;
        if (NP > 1) {
            DINT = "SG_DIN" + std::to_string(v) + "_" + std::to_string(nvar_++);
            DOUTT = "SG_DOUT" + std::to_string(v) + "_" + std::to_string(nvar_++);
            consts_ << "__constant__ int " << DINT << "[" << NP << "] = {";
            for (int64_t q = 0; q < NP; q++) consts_ << (q ? ", " : "") << din[q];
            consts_ << "};\n__constant__ int " << DOUTT << "[" << NP << "] = {";
            for (int64_t q = 0; q < NP; q++) consts_ << (q ? ", " : "") << dout[q];
            consts_ << "};\n";
        }
        if (fused_ && beam_slide_on() && !std::getenv("SG_FFMA2") && beam_slide_cfg(v).B > 0) {
            emit_beam_fir_slide(b, v, F0, rot, NP, DINT, DOUTT);
            return;
        }
        if (beam_f2_[v] && ctab) {
            emit_beam_fir_f2(b, v, F0, NP, DINT, DOUTT, ct->second);
            return;
        }
        b << "      const int items = nf * " << NBP * NP << ";\n";
        // dynamic item scheduling (fused kernels): warps grab 32 consecutive items from a
        // shared counter, so warps the scheduler favours (highest warp id first) take more
        // items and the level's tail is one item per thread, not a whole static share
        const bool dyn = fused_ && !std::getenv("SG_STATIC_ITEMS");
        if (dyn) {
            const int slot = nctr_++;
            b << "      for (int it0 = 0;;) {\n"
              << "        if ((tid & 31) == 0) it0 = atomicAdd(&sg_ctr[" << slot << "], 32);\n"
              << "        it0 = __shfl_sync(0xffffffffu, it0, 0);\n"
              << "        if (it0 >= items) break;\n"
              << "        const int it = it0 + (tid & 31);\n"
              << "        if (it < items) {\n";
        } else {
            b << "      int it = tid - " << rot % NT_ << "; if (it < 0) it += NT;\n"
              << "      for (; it < items; it += NT) {\n";
        }
        b
          << "        const int pq = it / (nf * " << NBP << ");\n"
          << "        const int itp = it - pq * (nf * " << NBP << ");\n"
          << "        const int j = itp / " << NBP << ";\n"
          << "        const int pb = itp - j * " << NBP << ";\n";
        if (pair)
            b << "        for (int half = 0; half < 2; half++) {\n"
              << "        const int blk = half ? " << NB - 1 << " - pb : pb;\n"
              << "        if (half && blk == pb) break;\n";
        else if (dyn)  // longest blocks (most live taps) first: the dynamic tail is short
            b << "        { const int blk = " << NB - 1 << " - pb;\n";
        else
            b << "        { const int blk = pb;\n";
        b << "        const int t0 = blk * " << B << ";\n"
          << "        const int ilim = min(" << L << ", (t0 + " << B - 1 << ") * " << DEC << " + 1);\n"
          << "        const int lf = " << F0 << " + j;\n"
          << "        " << T_ << "* smi = sm + " << (NP > 1 ? DINT + "[pq]" : std::string("0")) << ";\n"
          << "        " << T_ << "* smo = sm + " << (NP > 1 ? DOUTT + "[pq]" : std::string("0")) << ";\n"
          << "        (void)pq; (void)smi; (void)smo;\n"
          << "        float re[" << B << "], im[" << B << "];\n"
          << "#pragma unroll\n"
          << "        for (int bb = 0; bb < " << B << "; bb++) { re[bb] = 0.0f; im[bb] = 0.0f; }\n"
          << "        if (gf + lf >= 0) {\n";
        auto chunk = [&](const std::string& i0expr, bool checked, const std::string& cr_of, const std::string& ci_of) {
            b << "          {\n"
              << "            const int s0 = t0 * " << DEC << " - (" << i0expr << ") - " << TC - 1 << ";\n"
              << "            float xr[" << NWIN << "], xi[" << NWIN << "];\n";
            for (int64_t k = 0; k < NWIN; k++) {
                Lin pr = Lin::v("lf", n.pop, 2 * k);
                pr.t.push_back({"s0", 2});
                Lin pi = pr.plus(1);
                std::string er = "smi" + read_expr(n.in[0], pr).substr(2), ei = "smi" + read_expr(n.in[0], pi).substr(2);
                if (checked)
                    b << "            { const int s = s0 + " << k << "; const bool ok = s >= 0 && s < " << FR << ";\n"
                      << "              xr[" << k << "] = ok ? " << er << " : 0.0f;\n"
                      << "              xi[" << k << "] = ok ? " << ei << " : 0.0f; }\n";
                else
                    b << "            xr[" << k << "] = " << er << "; xi[" << k << "] = " << ei << ";\n";
            }
            if (ctab && !unroll) {  // (cr, ci) pairs of two taps per 128-bit shared-memory broadcast
                b << "#pragma unroll\n"
                  << "            for (int ii = 0; ii < " << TC << "; ii += 2) {\n"
                  << "              const float4 c4 = reinterpret_cast<const float4*>(sm + " << ct->second << ")[(" << i0expr
                  << " + ii) >> 1];\n"
                  << "#pragma unroll\n"
                  << "              for (int bb = 0; bb < " << B << "; bb++) {\n"
                  << "                const int k = bb * " << DEC << " - ii + " << TC - 1 << ";\n"
                  << "                sg_cmac(re[bb], im[bb], xr[k], xi[k], c4.x, c4.y);\n"
                  << "              }\n"
                  << "#pragma unroll\n"
                  << "              for (int bb = 0; bb < " << B << "; bb++) {\n"
                  << "                const int k = bb * " << DEC << " - ii + " << TC - 2 << ";\n"
                  << "                sg_cmac(re[bb], im[bb], xr[k], xi[k], c4.z, c4.w);\n"
                  << "              }\n"
                  << "            }\n"
                  << "          }\n";
                return;
            }
            b << "#pragma unroll\n"
              << "            for (int ii = 0; ii < " << TC << "; ii++) {\n"
              << "              const float cr = " << cr_of << ", ci = " << ci_of << ";\n"
              << "#pragma unroll\n"
              << "              for (int bb = 0; bb < " << B << "; bb++) {\n"
              << "                const int k = bb * " << DEC << " - ii + " << TC - 1 << ";\n"
              << "                sg_cmac(re[bb], im[bb], xr[k], xi[k], cr, ci);\n"
              << "              }\n"
              << "            }\n"
              << "          }\n";
        };
        if (unroll) {
            for (int64_t i0 = 0; i0 < L; i0 += TC) {
                // immediates: a switch-free table via a constexpr lambda index is not available in NVRTC C++17
                // device code, so emit the chunk's TC coefficients as an initialised local array
                std::string cr = const_array(std::vector<float>(wr.begin() + i0, wr.begin() + i0 + TC));
                std::string ci = const_array(std::vector<float>(wi.begin() + i0, wi.begin() + i0 + TC));
                b << "          if (t0 * " << DEC << " - " << i0 + TC - 1 << " >= 0 && t0 * " << DEC << " + " << (B - 1) * DEC
                  << " - " << i0 << " < " << FR << ") {\n";
                chunk(std::to_string(i0), false, cr + "[ii]", ci + "[ii]");
                b << "          } else {\n";
                chunk(std::to_string(i0), true, cr + "[ii]", ci + "[ii]");
                b << "          }\n";
            }
        } else {
            b << "#pragma unroll 1\n"
              << "          for (int i0 = 0; i0 < ilim; i0 += " << TC << ") {\n"
              << "            if (t0 * " << DEC << " - i0 - " << TC - 1 << " >= 0 && t0 * " << DEC << " + " << (B - 1) * DEC
              << " - i0 < " << FR << ") {\n";
            chunk("i0", false, WR + "[i0 + ii]", WI + "[i0 + ii]");
            b << "            } else {\n";
            chunk("i0", true, WR + "[i0 + ii]", WI + "[i0 + ii]");
            b << "            }\n          }\n";
        }
        b << "        }\n"
          << "#pragma unroll\n"
          << "        for (int bb = 0; bb < " << B << "; bb++)\n"
          << "          if (t0 + bb < " << OUT << ") {\n";
        {
            const int eo = n.out[0];
            Lin pos = Lin::v("j", n.push, f_.edges[eo].pre + F0 * n.push);
            pos.t.push_back({"(t0 + bb)", 2});
            b << "            smo[" << buf_index(eo, pos).str() << "] = re[bb];\n"
              << "            smo[" << buf_index(eo, pos.plus(1)).str() << "] = im[bb];\n";
        }
        b << "          }\n"
          << "        }\n";
        if (dyn) b << "        }\n";
        b << "      }\n";
    }
};

KernelInfo generate_kernel(const Flat& f, const std::vector<int>& nodes, int part_id, const CodegenOpts& opt) {
    for (int v : nodes)
        if (f.nodes[v].type == N_LOOP) {
            if (nodes.size() != 1) throw Error(SG_E_PLAN, "a feedback loop must be a partition of its own");
            LoopGen g(f, v, part_id);
            return g.run();
        }
    std::string why;
    bool reg_ok = register_mode_eligible(f, nodes, &why);
    int mode = opt.mode;
    if (mode == 1 && !reg_ok) throw Error(SG_E_UNSUPPORTED, "register mode not possible: " + why);
    if (mode == 0) mode = reg_ok ? 1 : 2;
    if (mode == 1 && opt.mode == 0 && !std::getenv("SG_NO_BITSLICE") && bitslice_eligible(f, nodes, nullptr)) {
        try {
            BitGen g(f, nodes, part_id);
            return g.run(opt);
        } catch (const Error&) {
            // bit kinds whose words cross the partition boundary (e.g. a lone XOR): plain register mode
        }
    }
    if (mode == 1) {
        RegGen g(f, nodes, part_id);
        return g.run(opt);
    }
    if (mode == 2 && opt.mode == 0 && !std::getenv("SG_NO_GATHER")) {
        bool views_only = true;
        for (int v : nodes) views_only = views_only && is_view_node(f.nodes[v]);
        if (views_only) {
            GatherGen g(f, nodes, part_id);
            return g.run();
        }
    }
    StageGen g(f, nodes, part_id);
    CodegenOpts o2 = opt;
    if (mode == 3) o2.mode = -2;  // staged without the fused fast path (general path only)
    return g.run(o2);
}

}  // namespace sg
