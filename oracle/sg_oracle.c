/*
 * sg_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, sequential CPU interpreter of a synchronous-dataflow stream
 * program.  Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load it.  It shares no code with the CUDA path
 * (paper_conf_cgo_nguyenl16_b200/); it reads the neutral program text written by
 * workloads/spec.py and the same input bytes.
 *
 * What it computes (PAPER.md is the authority):
 *   - a stream graph: filters composed by pipeline and split-join
 *     (section 2.1.1; section 3.1);
 *   - every filter fires when its input holds `peek` items, reads them, pops
 *     `pop`, pushes `push` (push/pop "rates");
 *   - the method partitions / maps / pipelines the graph but must reach exactly
 *     the output of executing the graph (fragments are independent,
 *     PAPER.md:560-561, section 3.2.3).  The oracle is that definition: it feeds
 *     the input in chunks and, after each chunk, fires every node in a
 *     topological order as often as its inputs allow (a Kahn process network;
 *     any fair schedule gives the same output stream).
 *   - the repetition vector ("firing rate ... number of times a filter has to be
 *     executed in order to match its input and output rates")
 *     is solved separately by orc_rates(), with rational arithmetic.
 *
 * Filter-kind arithmetic follows the readings of SURVEY.md 8(c)-3 (the paper
 * is silent on every filter body); they are listed in DESIGN.md "Readings".
 * Built with -O2 -ffp-contract=off (no FMA contraction, no fast-math):
 * every fused multiply-add below is an explicit fmaf().
 *
 * Pins: tests/test_oracle.py (DFT, convolution, sorting, closed-form rates,
 * Kahn determinism, chunked == whole, ...).
 */
#include <math.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#define ORC_OK 0
#define ORC_E_PARSE -1
#define ORC_E_RATE -3
#define ORC_E_KIND -4
#define ORC_E_NOMEM -5

typedef union {
    float f;
    int32_t i;
    uint32_t u;
} word;

enum { K_IDENTITY, K_FIR, K_DELAY, K_DECIMATE, K_EXPAND, K_COMPARE_EXCHANGE, K_FFT_REORDER,
       K_COMBINE_DFT, K_FM_DEMOD, K_SUBTRACT, K_AMPLIFY, K_ADD, K_BEAM_FIR, K_BEAMFORM,
       K_MAGNITUDE, K_MULTIPLY, K_PERMUTE, K_XOR, K_XOR_CONST, K_SBOX, K_INTO_BITS, K_BITS_TO_INT,
       K_COUNT };
static const char* KIND_NAMES[K_COUNT] = {
    "IDENTITY", "FIR", "DELAY", "DECIMATE", "EXPAND", "COMPARE_EXCHANGE", "FFT_REORDER",
    "COMBINE_DFT", "FM_DEMOD", "SUBTRACT", "AMPLIFY", "ADD", "BEAM_FIR", "BEAMFORM", "MAGNITUDE",
    "MULTIPLY", "PERMUTE", "XOR", "XOR_CONST", "SBOX", "INTO_BITS", "BITS_TO_INT"};

enum { T_FILTER, T_SPLIT_DUP, T_SPLIT_RR, T_JOIN_RR };

typedef struct {
    word* a;
    long long head, tail, cap; /* items a[head..tail) */
} fifo;

typedef struct {
    int type, kind;
    int ni, nf;
    int* iv;
    float* fv;
    int nw;
    int* w; /* split / join weights */
    int pop, push, peek, prework;
    int prework_done;
    int n_in, n_out;
    int* in;  /* edge ids */
    int* out; /* edge ids */
    /* twiddles for COMBINE_DFT */
    float* tw_r;
    float* tw_i;
} node;

typedef struct {
    int src, dst; /* node ids, -1 = graph boundary */
    fifo q;
} edge;

typedef struct {
    int is_i32;
    int n_nodes, cap_nodes;
    node* nodes;
    int n_edges, cap_edges;
    edge* edges;
    int in_edge, out_edge;
    /* parser */
    const char* p;
    int err;
} graph;

/* ------------------------------------------------------------------ fifo */
static int fifo_reserve(fifo* q, long long extra) {
    if (q->tail + extra <= q->cap) return 0;
    long long live = q->tail - q->head;
    if (q->head > 0 && live + extra <= q->cap) {
        memmove(q->a, q->a + q->head, (size_t)live * sizeof(word));
        q->head = 0;
        q->tail = live;
        return 0;
    }
    long long ncap = q->cap ? q->cap : 256;
    while (ncap < live + extra) ncap *= 2;
    word* na = (word*)malloc((size_t)ncap * sizeof(word));
    if (!na) return -1;
    if (live) memcpy(na, q->a + q->head, (size_t)live * sizeof(word));
    free(q->a);
    q->a = na;
    q->cap = ncap;
    q->head = 0;
    q->tail = live;
    return 0;
}
static long long fifo_avail(const fifo* q) { return q->tail - q->head; }
static void fifo_push(fifo* q, word v) {
    if (fifo_reserve(q, 1)) { fprintf(stderr, "oracle: out of memory\n"); abort(); }
    q->a[q->tail++] = v;
}
static word fifo_peek(const fifo* q, long long i) { return q->a[q->head + i]; }
static void fifo_pop(fifo* q, long long n) { q->head += n; }

/* ---------------------------------------------------------------- parser */
static void skip_ws(graph* g) {
    while (*g->p == ' ' || *g->p == '\n' || *g->p == '\t' || *g->p == '\r') g->p++;
}
static int next_tok(graph* g, char* buf, int n) {
    skip_ws(g);
    int k = 0;
    while (*g->p && *g->p != ' ' && *g->p != '\n' && *g->p != '\t' && *g->p != '\r') {
        if (k < n - 1) buf[k++] = *g->p;
        g->p++;
    }
    buf[k] = 0;
    return k;
}
static long long next_int(graph* g) {
    char b[64];
    if (!next_tok(g, b, 64)) { g->err = ORC_E_PARSE; return 0; }
    char* e;
    long long v = strtoll(b, &e, 10);
    if (*e) g->err = ORC_E_PARSE;
    return v;
}
static float next_float(graph* g) {
    char b[64];
    if (!next_tok(g, b, 64)) { g->err = ORC_E_PARSE; return 0; }
    char* e;
    double v = strtod(b, &e); /* hex floats, exact */
    if (*e) g->err = ORC_E_PARSE;
    return (float)v;
}

static int new_edge(graph* g, int src) {
    if (g->n_edges == g->cap_edges) {
        g->cap_edges = g->cap_edges ? 2 * g->cap_edges : 64;
        g->edges = (edge*)realloc(g->edges, (size_t)g->cap_edges * sizeof(edge));
    }
    edge* e = &g->edges[g->n_edges];
    memset(e, 0, sizeof(*e));
    e->src = src;
    e->dst = -1;
    return g->n_edges++;
}
static int new_node(graph* g) {
    if (g->n_nodes == g->cap_nodes) {
        g->cap_nodes = g->cap_nodes ? 2 * g->cap_nodes : 64;
        g->nodes = (node*)realloc(g->nodes, (size_t)g->cap_nodes * sizeof(node));
    }
    node* n = &g->nodes[g->n_nodes];
    memset(n, 0, sizeof(*n));
    return g->n_nodes++;
}

/* Rates of a filter kind, from its parameters. */
static int filter_rates(graph* g, node* n) {
    int* iv = n->iv;
    int ni = n->ni, nf = n->nf;
    n->prework = 0;
    switch (n->kind) {
    case K_IDENTITY: n->pop = 1; n->push = 1; n->peek = 1; break;
    case K_FIR:
        if (ni < 2 || iv[0] < 1 || iv[1] < 1 || nf != iv[0] || g->is_i32) return ORC_E_KIND;
        n->peek = iv[0] > iv[1] ? iv[0] : iv[1];
        n->pop = iv[1];
        n->push = 1;
        break;
    case K_DELAY:
        if (ni < 1 || iv[0] < 0) return ORC_E_KIND;
        n->pop = n->push = n->peek = 1;
        n->prework = iv[0];
        break;
    case K_DECIMATE:
        if (ni < 1 || iv[0] < 1) return ORC_E_KIND;
        n->pop = n->peek = iv[0]; n->push = 1;
        break;
    case K_EXPAND:
        if (ni < 1 || iv[0] < 1) return ORC_E_KIND;
        n->pop = n->peek = 1; n->push = iv[0];
        break;
    case K_COMPARE_EXCHANGE: n->pop = n->peek = n->push = 2; break;
    case K_FFT_REORDER:
        if (ni < 1 || iv[0] < 2 || (iv[0] & 1) || g->is_i32) return ORC_E_KIND;
        n->pop = n->peek = n->push = 2 * iv[0];
        break;
    case K_COMBINE_DFT:
        if (ni < 1 || iv[0] < 2 || (iv[0] & 1) || g->is_i32) return ORC_E_KIND;
        n->pop = n->peek = n->push = 2 * iv[0];
        break;
    case K_FM_DEMOD:
        if (nf < 1 || g->is_i32) return ORC_E_KIND;
        n->peek = 2; n->pop = 1; n->push = 1;
        break;
    case K_SUBTRACT: if (g->is_i32) return ORC_E_KIND; n->pop = n->peek = 2; n->push = 1; break;
    case K_AMPLIFY: if (nf < 1 || g->is_i32) return ORC_E_KIND; n->pop = n->peek = n->push = 1; break;
    case K_ADD:
        if (ni < 1 || iv[0] < 1) return ORC_E_KIND;
        n->pop = n->peek = iv[0]; n->push = 1;
        break;
    case K_BEAM_FIR:
        if (ni < 3 || iv[0] < 1 || iv[1] < 1 || iv[2] < 1 || iv[2] % iv[1] || nf != 2 * iv[0] || g->is_i32)
            return ORC_E_KIND;
        n->pop = n->peek = 2 * iv[2];
        n->push = 2 * (iv[2] / iv[1]);
        break;
    case K_BEAMFORM:
        if (ni < 1 || iv[0] < 1 || nf != 2 * iv[0] || g->is_i32) return ORC_E_KIND;
        n->pop = n->peek = 2 * iv[0]; n->push = 2;
        break;
    case K_MAGNITUDE: if (g->is_i32) return ORC_E_KIND; n->pop = n->peek = 2; n->push = 1; break;
    case K_MULTIPLY: if (g->is_i32) return ORC_E_KIND; n->pop = n->peek = 2; n->push = 1; break;
    /* DES (Fig. 4.2c; StreamIt bit-per-item form) */
    case K_PERMUTE: /* {n, idx[m]}: y[k] = x[idx[k]] */
        if (ni < 2 || iv[0] < 1) return ORC_E_KIND;
        for (int k = 1; k < ni; k++) if (iv[k] < 0 || iv[k] >= iv[0]) return ORC_E_KIND;
        n->pop = n->peek = iv[0]; n->push = ni - 1;
        break;
    case K_XOR: /* {n}: y[i] = x[i] ^ x[n+i] */
        if (ni < 1 || iv[0] < 1 || !g->is_i32) return ORC_E_KIND;
        n->pop = n->peek = 2 * iv[0]; n->push = iv[0];
        break;
    case K_XOR_CONST: /* {n, k[n]}: y[i] = x[i] ^ k[i] */
        if (ni < 1 || iv[0] < 1 || ni != 1 + iv[0] || !g->is_i32) return ORC_E_KIND;
        n->pop = n->peek = n->push = iv[0];
        break;
    case K_SBOX: /* {t[64]}: 6 bits in, 4 bits out */
        if (ni != 64 || !g->is_i32) return ORC_E_KIND;
        for (int k = 0; k < 64; k++) if (iv[k] < 0 || iv[k] > 15) return ORC_E_KIND;
        n->pop = n->peek = 6; n->push = 4;
        break;
    case K_INTO_BITS: if (!g->is_i32) return ORC_E_KIND; n->pop = n->peek = 1; n->push = 32; break;
    case K_BITS_TO_INT: if (!g->is_i32) return ORC_E_KIND; n->pop = n->peek = 32; n->push = 1; break;
    default: return ORC_E_KIND;
    }
    if (n->kind == K_COMBINE_DFT) {
        /* w_k = exp(-2 pi i k / j), k < j/2, computed directly in double, rounded to float */
        int j = iv[0];
        n->tw_r = (float*)malloc(sizeof(float) * (size_t)(j / 2));
        n->tw_i = (float*)malloc(sizeof(float) * (size_t)(j / 2));
        for (int k = 0; k < j / 2; k++) {
            double a = 2.0 * M_PI * (double)k / (double)j;
            n->tw_r[k] = (float)cos(a);
            n->tw_i[k] = (float)(-sin(a));
        }
    }
    return ORC_OK;
}

/* Build the flattened graph for one stream; returns its output edge. */
static int build(graph* g, int in_edge) {
    char tok[64];
    if (g->err) return -1;
    if (!next_tok(g, tok, 64)) { g->err = ORC_E_PARSE; return -1; }
    if (tok[0] == 'F' && tok[1] == 0) {
        char kname[64];
        next_tok(g, kname, 64);
        int id = new_node(g);
        node* n = &g->nodes[id];
        n->type = T_FILTER;
        n->kind = -1;
        for (int k = 0; k < K_COUNT; k++)
            if (!strcmp(kname, KIND_NAMES[k])) n->kind = k;
        if (n->kind < 0) { g->err = ORC_E_KIND; return -1; }
        n->ni = (int)next_int(g);
        n->iv = (int*)calloc((size_t)n->ni + 1, sizeof(int));
        for (int k = 0; k < n->ni; k++) n->iv[k] = (int)next_int(g);
        n->nf = (int)next_int(g);
        n->fv = (float*)calloc((size_t)n->nf + 1, sizeof(float));
        for (int k = 0; k < n->nf; k++) n->fv[k] = next_float(g);
        if (g->err) return -1;
        int rc = filter_rates(g, n);
        if (rc) { g->err = rc; return -1; }
        n->n_in = 1; n->n_out = 1;
        n->in = (int*)malloc(sizeof(int));
        n->out = (int*)malloc(sizeof(int));
        n->in[0] = in_edge;
        g->edges[in_edge].dst = id;
        int oe = new_edge(g, id);
        g->nodes[id].out[0] = oe;
        return oe;
    }
    if (tok[0] == 'P' && tok[1] == 0) {
        long long cnt = next_int(g);
        int e = in_edge;
        for (long long k = 0; k < cnt && !g->err; k++) e = build(g, e);
        return e;
    }
    if (tok[0] == 'J' && tok[1] == 0) {
        char sk[8];
        next_tok(g, sk, 8);
        int nb = (int)next_int(g);
        if (nb < 1 || g->err) { g->err = ORC_E_PARSE; return -1; }
        int sid = new_node(g);
        node* s = &g->nodes[sid];
        s->type = (sk[0] == 'D') ? T_SPLIT_DUP : T_SPLIT_RR;
        s->nw = nb;
        s->w = (int*)calloc((size_t)nb, sizeof(int));
        if (s->type == T_SPLIT_RR)
            for (int b = 0; b < nb; b++) s->w[b] = (int)next_int(g);
        int* jw = (int*)calloc((size_t)nb, sizeof(int));
        for (int b = 0; b < nb; b++) jw[b] = (int)next_int(g);
        s->n_in = 1; s->n_out = nb;
        s->in = (int*)malloc(sizeof(int));
        s->out = (int*)malloc(sizeof(int) * (size_t)nb);
        s->in[0] = in_edge;
        g->edges[in_edge].dst = sid;
        int* outs = (int*)malloc(sizeof(int) * (size_t)nb);
        for (int b = 0; b < nb; b++) {
            int be = new_edge(g, sid);
            g->nodes[sid].out[b] = be;
            outs[b] = build(g, be);
            if (g->err) { free(outs); free(jw); return -1; }
        }
        int jid = new_node(g);
        node* jn = &g->nodes[jid];
        jn->type = T_JOIN_RR;
        jn->nw = nb;
        jn->w = jw;
        jn->n_in = nb; jn->n_out = 1;
        jn->in = outs;
        jn->out = (int*)malloc(sizeof(int));
        for (int b = 0; b < nb; b++) g->edges[outs[b]].dst = jid;
        int oe = new_edge(g, jid);
        g->nodes[jid].out[0] = oe;
        return oe;
    }
    if (tok[0] == 'L' && tok[1] == 0) {
        /* feedback loop ("pipeline ..., split-join ..., and feedback loop"; StreamIt
         * form): joiner RR(jw0, jw1) merges the outer input (port 0) with the loop stream (port 1);
         * body; splitter (duplicate, or RR(sw0, sw1)) sends port 0 out, port 1 into the loop stream,
         * whose output returns to the joiner's port 1.  The n_enq enqueued items are the initial
         * contents of that returning edge (the loop's delay). */
        int jw0 = (int)next_int(g), jw1 = (int)next_int(g);
        char sk[8];
        next_tok(g, sk, 8);
        int st = (sk[0] == 'D') ? T_SPLIT_DUP : T_SPLIT_RR;
        int sw0 = 1, sw1 = 1;
        if (st == T_SPLIT_RR) { sw0 = (int)next_int(g); sw1 = (int)next_int(g); }
        long long nenq = next_int(g);
        if (g->err || jw0 < 0 || jw1 < 1 || sw0 < 0 || sw1 < 1 || nenq < 0) { g->err = ORC_E_PARSE; return -1; }
        word* enq = (word*)calloc((size_t)nenq + 1, sizeof(word));
        for (long long k = 0; k < nenq; k++) {
            if (g->is_i32) enq[k].i = (int32_t)next_int(g);
            else enq[k].f = next_float(g);
        }
        int jid = new_node(g);
        node* jn = &g->nodes[jid];
        jn->type = T_JOIN_RR;
        jn->nw = 2;
        jn->w = (int*)calloc(2, sizeof(int));
        jn->w[0] = jw0; jn->w[1] = jw1;
        jn->n_in = 2; jn->n_out = 1;
        jn->in = (int*)malloc(2 * sizeof(int));
        jn->out = (int*)malloc(sizeof(int));
        jn->in[0] = in_edge;
        jn->in[1] = -1;
        g->edges[in_edge].dst = jid;
        int je = new_edge(g, jid);
        g->nodes[jid].out[0] = je;
        int be = build(g, je);                         /* body */
        if (g->err) { free(enq); return -1; }
        int sid = new_node(g);
        node* sn = &g->nodes[sid];
        sn->type = st;
        sn->nw = 2;
        sn->w = (int*)calloc(2, sizeof(int));
        sn->w[0] = sw0; sn->w[1] = sw1;
        sn->n_in = 1; sn->n_out = 2;
        sn->in = (int*)malloc(sizeof(int));
        sn->out = (int*)malloc(2 * sizeof(int));
        sn->in[0] = be;
        g->edges[be].dst = sid;
        int oe = new_edge(g, sid);
        int le = new_edge(g, sid);
        g->nodes[sid].out[0] = oe;
        g->nodes[sid].out[1] = le;
        int re = build(g, le);                         /* loop stream */
        if (g->err) { free(enq); return -1; }
        g->nodes[jid].in[1] = re;
        g->edges[re].dst = jid;
        for (long long k = 0; k < nenq; k++) fifo_push(&g->edges[re].q, enq[k]);
        free(enq);
        return oe;
    }
    g->err = ORC_E_PARSE;
    return -1;
}

static void graph_free(graph* g) {
    for (int i = 0; i < g->n_nodes; i++) {
        node* n = &g->nodes[i];
        free(n->iv); free(n->fv); free(n->w); free(n->in); free(n->out);
        free(n->tw_r); free(n->tw_i);
    }
    for (int i = 0; i < g->n_edges; i++) free(g->edges[i].q.a);
    free(g->nodes);
    free(g->edges);
    memset(g, 0, sizeof(*g));
}

static int graph_parse(graph* g, const char* spec) {
    memset(g, 0, sizeof(*g));
    g->p = spec;
    char tok[64];
    next_tok(g, tok, 64);
    if (strcmp(tok, "SG1")) return ORC_E_PARSE;
    next_tok(g, tok, 64);
    if (!strcmp(tok, "i32")) g->is_i32 = 1;
    else if (strcmp(tok, "f32")) return ORC_E_PARSE;
    g->in_edge = new_edge(g, -1);
    g->out_edge = build(g, g->in_edge);
    if (g->err) { int e = g->err; graph_free(g); return e; }
    return ORC_OK;
}

/* ------------------------------------------------------- filter execution */
/* x: the `peek` items at the head of the input (oldest first); y: `push` outputs. */
static void work(const graph* g, const node* n, const word* x, word* y) {
    const int* iv = n->iv;
    const float* fv = n->fv;
    switch (n->kind) {
    case K_IDENTITY:
    case K_DELAY: y[0] = x[0]; break;
    case K_FIR: { /* acc = 0; acc = fmaf(peek(i), c[i], acc), i = 0..L-1 */
        float acc = 0.0f;
        for (int i = 0; i < iv[0]; i++) acc = fmaf(x[i].f, fv[i], acc);
        y[0].f = acc;
        break;
    }
    case K_DECIMATE: y[0] = x[0]; break;
    case K_EXPAND:
        y[0] = x[0];
        for (int i = 1; i < iv[0]; i++) y[i].u = 0u; /* +0.0f or integer 0 */
        break;
    case K_COMPARE_EXCHANGE: {
        word k1 = x[0], k2 = x[1], lo, hi;
        int le = g->is_i32 ? (k1.i <= k2.i) : (k1.f <= k2.f);
        if (le) { lo = k1; hi = k2; } else { lo = k2; hi = k1; }
        if (iv[0]) { y[0] = lo; y[1] = hi; } else { y[0] = hi; y[1] = lo; }
        break;
    }
    case K_FFT_REORDER: { /* complex items: evens first, then odds */
        int nn = iv[0], o = 0;
        for (int i = 0; i < nn; i += 2) { y[o++] = x[2 * i]; y[o++] = x[2 * i + 1]; }
        for (int i = 1; i < nn; i += 2) { y[o++] = x[2 * i]; y[o++] = x[2 * i + 1]; }
        break;
    }
    case K_COMBINE_DFT: { /* j/2 butterflies pairing complex k and k + j/2 */
        int j = iv[0], h = j / 2;
        for (int k = 0; k < h; k++) {
            float y0r = x[2 * k].f, y0i = x[2 * k + 1].f;
            float y1r = x[2 * (k + h)].f, y1i = x[2 * (k + h) + 1].f;
            float wr = n->tw_r[k], wi = n->tw_i[k];
            float p = y1i * wi;
            float tr = fmaf(y1r, wr, -p);
            float q = y1i * wr;
            float ti = fmaf(y1r, wi, q);
            y[2 * k].f = y0r + tr;
            y[2 * k + 1].f = y0i + ti;
            y[2 * (k + h)].f = y0r - tr;
            y[2 * (k + h) + 1].f = y0i - ti;
        }
        break;
    }
    case K_FM_DEMOD: {
        float p = x[0].f * x[1].f;
        y[0].f = (float)((double)fv[0] * atan((double)p));
        break;
    }
    case K_SUBTRACT: y[0].f = x[1].f - x[0].f; break;
    case K_AMPLIFY: y[0].f = x[0].f * fv[0]; break;
    case K_ADD:
        if (g->is_i32) {
            uint32_t s = 0u;
            for (int i = 0; i < iv[0]; i++) s = s + x[i].u;
            y[0].u = s;
        } else {
            float s = 0.0f;
            for (int i = 0; i < iv[0]; i++) s = s + x[i].f;
            y[0].f = s;
        }
        break;
    case K_BEAM_FIR: { /* one frame: y[t] = sum_i w_i x[t*dec - i], x[<0] = 0 within the frame */
        int L = iv[0], dec = iv[1], frame = iv[2];
        const float* wr = fv;
        const float* wi = fv + L;
        for (int to = 0; to < frame / dec; to++) {
            int t = to * dec;
            float re = 0.0f, im = 0.0f;
            for (int i = 0; i < L; i++) {
                float xr = 0.0f, xi = 0.0f;
                if (t - i >= 0) { xr = x[2 * (t - i)].f; xi = x[2 * (t - i) + 1].f; }
                re = fmaf(xr, wr[i], re);
                re = fmaf(-xi, wi[i], re);
                im = fmaf(xr, wi[i], im);
                im = fmaf(xi, wr[i], im);
            }
            y[2 * to].f = re;
            y[2 * to + 1].f = im;
        }
        break;
    }
    case K_BEAMFORM: {
        int nc = iv[0];
        const float* wr = fv;
        const float* wi = fv + nc;
        float re = 0.0f, im = 0.0f;
        for (int c = 0; c < nc; c++) {
            float xr = x[2 * c].f, xi = x[2 * c + 1].f;
            re = fmaf(xr, wr[c], re);
            re = fmaf(-xi, wi[c], re);
            im = fmaf(xr, wi[c], im);
            im = fmaf(xi, wr[c], im);
        }
        y[0].f = re;
        y[1].f = im;
        break;
    }
    case K_MAGNITUDE: {
        float a = x[0].f, b = x[1].f;
        float bb = b * b;
        y[0].f = sqrtf(fmaf(a, a, bb));
        break;
    }
    case K_MULTIPLY: y[0].f = x[0].f * x[1].f; break;
    case K_PERMUTE:
        for (int k = 1; k < n->ni; k++) y[k - 1] = x[iv[k]];
        break;
    case K_XOR:
        for (int i = 0; i < iv[0]; i++) y[i].u = x[i].u ^ x[iv[0] + i].u;
        break;
    case K_XOR_CONST:
        for (int i = 0; i < iv[0]; i++) y[i].u = x[i].u ^ (uint32_t)iv[1 + i];
        break;
    case K_SBOX: { /* FIPS 46-3: bits b1..b6 (first popped = b1); row = b1 b6, column = b2 b3 b4 b5;
                      the table is row-major (16 columns); output bits most significant first */
        uint32_t b[6];
        for (int i = 0; i < 6; i++) b[i] = x[i].u & 1u;
        uint32_t row = 2u * b[0] + b[5];
        uint32_t col = 8u * b[1] + 4u * b[2] + 2u * b[3] + b[4];
        uint32_t v = (uint32_t)iv[16 * row + col];
        for (int i = 0; i < 4; i++) y[i].u = (v >> (3 - i)) & 1u;
        break;
    }
    case K_INTO_BITS: /* most significant bit first */
        for (int k = 0; k < 32; k++) y[k].u = (x[0].u >> (31 - k)) & 1u;
        break;
    case K_BITS_TO_INT: {
        uint32_t v = 0u;
        for (int k = 0; k < 32; k++) v = 2u * v + (x[k].u & 1u);
        y[0].u = v;
        break;
    }
    default: abort();
    }
}

/* Fire node `id` as many times as its inputs allow.  Returns firings. */
static long long fire_all(graph* g, int id, word* xs, word* ys) {
    node* n = &g->nodes[id];
    long long fired = 0;
    if (n->type == T_FILTER) {
        fifo* in = &g->edges[n->in[0]].q;
        fifo* out = &g->edges[n->out[0]].q;
        if (n->prework && !n->prework_done) { /* Delay prework: k zeros, needs no input */
            word z; z.u = 0u;
            for (int i = 0; i < n->prework; i++) fifo_push(out, z);
            n->prework_done = 1;
        }
        while (fifo_avail(in) >= n->peek) {
            for (int i = 0; i < n->peek; i++) xs[i] = fifo_peek(in, i);
            work(g, n, xs, ys);
            fifo_pop(in, n->pop);
            for (int i = 0; i < n->push; i++) fifo_push(out, ys[i]);
            fired++;
        }
    } else if (n->type == T_SPLIT_DUP) {
        fifo* in = &g->edges[n->in[0]].q;
        while (fifo_avail(in) >= 1) {
            word v = fifo_peek(in, 0);
            fifo_pop(in, 1);
            for (int b = 0; b < n->n_out; b++) fifo_push(&g->edges[n->out[b]].q, v);
            fired++;
        }
    } else if (n->type == T_SPLIT_RR) {
        fifo* in = &g->edges[n->in[0]].q;
        long long tot = 0;
        for (int b = 0; b < n->nw; b++) tot += n->w[b];
        while (tot > 0 && fifo_avail(in) >= tot) {
            for (int b = 0; b < n->nw; b++)
                for (int k = 0; k < n->w[b]; k++) {
                    fifo_push(&g->edges[n->out[b]].q, fifo_peek(in, 0));
                    fifo_pop(in, 1);
                }
            fired++;
        }
    } else { /* T_JOIN_RR */
        for (;;) {
            int ok = 1;
            for (int b = 0; b < n->nw; b++)
                if (fifo_avail(&g->edges[n->in[b]].q) < n->w[b]) ok = 0;
            if (!ok) break;
            fifo* out = &g->edges[n->out[0]].q;
            for (int b = 0; b < n->nw; b++) {
                fifo* in = &g->edges[n->in[b]].q;
                for (int k = 0; k < n->w[b]; k++) {
                    fifo_push(out, fifo_peek(in, 0));
                    fifo_pop(in, 1);
                }
            }
            fired++;
        }
    }
    return fired;
}

static int max_window(const graph* g) {
    int m = 8;
    for (int i = 0; i < g->n_nodes; i++) {
        const node* n = &g->nodes[i];
        if (n->peek > m) m = n->peek;
        if (n->push > m) m = n->push;
    }
    return m;
}

/*
 * Run the program on `n_in` input items (4-byte words), collecting at most
 * `n_out_max` output items.  *n_out gets the number produced.  `chunk` input
 * items are fed per round (any positive value gives the same output: Kahn
 * determinism, pinned in tests).  `order_seed` != 0 fires the nodes of each
 * round in a different (still topological) order: sinks-first sweeps repeated
 * until quiescent -- a second valid schedule for the determinism pin.
 */
int orc_run(const char* spec, const void* input, long long n_in, void* output,
            long long n_out_max, long long* n_out, long long chunk, int order_seed) {
    graph g;
    int rc = graph_parse(&g, spec);
    if (rc) return rc;
    if (chunk <= 0) chunk = 4096;
    int mw = max_window(&g);
    word* xs = (word*)malloc(sizeof(word) * (size_t)mw);
    word* ys = (word*)malloc(sizeof(word) * (size_t)mw);
    const word* in = (const word*)input;
    word* out = (word*)output;
    long long fed = 0, produced = 0;
    fifo* qin = &g.edges[g.in_edge].q;
    fifo* qout = &g.edges[g.out_edge].q;
    for (;;) {
        long long c = n_in - fed < chunk ? n_in - fed : chunk;
        for (long long k = 0; k < c; k++) fifo_push(qin, in[fed + k]);
        fed += c;
        if (order_seed == 0) {
            /* sweeps in node order until nothing fires (one sweep suffices without feedback loops) */
            long long any;
            do {
                any = 0;
                for (int id = 0; id < g.n_nodes; id++) any += fire_all(&g, id, xs, ys);
            } while (any);
        } else {
            /* reverse sweeps until nothing fires: each sweep fires downstream nodes first */
            long long any;
            do {
                any = 0;
                for (int id = g.n_nodes - 1; id >= 0; id--) any += fire_all(&g, id, xs, ys);
            } while (any);
        }
        while (fifo_avail(qout) > 0 && produced < n_out_max) {
            out[produced++] = fifo_peek(qout, 0);
            fifo_pop(qout, 1);
        }
        if (qout != qin) fifo_pop(qout, fifo_avail(qout));
        if (produced >= n_out_max || fed >= n_in) break;
    }
    *n_out = produced;
    free(xs);
    free(ys);
    graph_free(&g);
    return ORC_OK;
}

/* ------------------------------------------------------------ rate solver */
static long long gcdll(long long a, long long b) {
    if (a < 0) a = -a;
    if (b < 0) b = -b;
    while (b) { long long t = a % b; a = b; b = t; }
    return a;
}

/* items node `id` pops from its input k / pushes to its output k per firing */
static long long pop_of(const node* n, int k) {
    if (n->type == T_FILTER) return n->pop;
    if (n->type == T_SPLIT_DUP) return 1;
    if (n->type == T_SPLIT_RR) { long long t = 0; for (int b = 0; b < n->nw; b++) t += n->w[b]; return t; }
    return n->w[k];
}
static long long push_of(const node* n, int k) {
    if (n->type == T_FILTER) return n->push;
    if (n->type == T_SPLIT_DUP) return 1;
    if (n->type == T_SPLIT_RR) return n->w[k];
    long long t = 0;
    for (int b = 0; b < n->nw; b++) t += n->w[b];
    return t;
}

/*
 * Balance equations r_u * push_u(e) = r_v * pop_v(e) for every edge
 * (PAPER.md:229-231), solved with exact fractions by propagation from node 0,
 * then scaled to the minimal positive integer vector (gcd 1).
 * reps[n_nodes]; node_info[4*n] = {type, kind, pop(in0), push(out0)}.
 */
int orc_rates(const char* spec, long long* reps, int max_nodes, int* n_nodes, int* node_info,
              long long* in_per_iter, long long* out_per_iter) {
    graph g;
    int rc = graph_parse(&g, spec);
    if (rc) return rc;
    int N = g.n_nodes;
    *n_nodes = N;
    if (N == 0 || N > max_nodes) { graph_free(&g); return N == 0 ? ORC_E_PARSE : ORC_E_NOMEM; }
    long long* num = (long long*)calloc((size_t)N, sizeof(long long));
    long long* den = (long long*)calloc((size_t)N, sizeof(long long));
    int* stack = (int*)malloc(sizeof(int) * (size_t)N);
    int sp = 0;
    num[0] = 1; den[0] = 1;
    stack[sp++] = 0;
    rc = ORC_OK;
    while (sp > 0 && rc == ORC_OK) {
        int u = stack[--sp];
        node* nu = &g.nodes[u];
        /* neighbours through output and input edges */
        for (int dir = 0; dir < 2; dir++) {
            int cnt = dir == 0 ? nu->n_out : nu->n_in;
            for (int k = 0; k < cnt; k++) {
                int e = dir == 0 ? nu->out[k] : nu->in[k];
                int v = dir == 0 ? g.edges[e].dst : g.edges[e].src;
                if (v < 0) continue;
                node* nv = &g.nodes[v];
                int kv = 0;
                if (dir == 0) { for (int q = 0; q < nv->n_in; q++) if (nv->in[q] == e) kv = q; }
                else { for (int q = 0; q < nv->n_out; q++) if (nv->out[q] == e) kv = q; }
                /* dir 0: r_v = r_u * push_u / pop_v ; dir 1: r_v = r_u * pop_u / push_v */
                long long a = dir == 0 ? push_of(nu, k) : pop_of(nu, k);
                long long b = dir == 0 ? pop_of(nv, kv) : push_of(nv, kv);
                long long n2 = num[u] * a, d2 = den[u] * b;
                long long gg = gcdll(n2, d2);
                n2 /= gg; d2 /= gg;
                if (den[v] == 0) {
                    num[v] = n2; den[v] = d2;
                    stack[sp++] = v;
                } else if (num[v] != n2 || den[v] != d2) {
                    rc = ORC_E_RATE;
                }
            }
        }
    }
    if (rc == ORC_OK) {
        long long L = 1;
        for (int i = 0; i < N; i++) L = L / gcdll(L, den[i]) * den[i];
        long long G = 0;
        for (int i = 0; i < N; i++) { reps[i] = num[i] * (L / den[i]); G = gcdll(G, reps[i]); }
        for (int i = 0; i < N; i++) reps[i] /= G;
        for (int i = 0; i < N; i++) {
            node* n = &g.nodes[i];
            node_info[4 * i + 0] = n->type;
            node_info[4 * i + 1] = n->type == T_FILTER ? n->kind : -1;
            node_info[4 * i + 2] = (int)pop_of(n, 0);
            node_info[4 * i + 3] = (int)push_of(n, 0);
        }
        int first = g.edges[g.in_edge].dst, last = g.edges[g.out_edge].src;
        *in_per_iter = reps[first] * pop_of(&g.nodes[first], 0);
        int klast = 0;
        for (int q = 0; q < g.nodes[last].n_out; q++) if (g.nodes[last].out[q] == g.out_edge) klast = q;
        *out_per_iter = reps[last] * push_of(&g.nodes[last], klast);
    }
    free(num); free(den); free(stack);
    graph_free(&g);
    return rc;
}
