// culi_eval.cuh — device side of libculi.so: heap access (16-byte nodes), warp-aggregated bump allocator,
// environment lookup, and the explicit-stack (non-recursive) eval/apply machine.  sm_100a only.
//
// The paper's evaluator is a recursive tree walk using CUDA device recursion (§III-B.c,
// L172-175).  Here one thread runs one evaluation as a state machine over two per-thread stacks held in
// HBM, interleaved across threads ("level-major": entry i of every thread is contiguous, so lanes that
// run the same code at the same stack height coalesce):
//   K-stack  (uint4 per entry) : continuation frames  {cursor, env, vsbase, depth|kind<<12|count<<16}
//   V-stack  (uint4 per entry) : values and environment frames {w.lo, w.hi, sym, tag}
// The machine replays the recursive definition of SURVEY §8(c).4 in the same order, so canonical step
// counts, depths and first errors match the oracle exactly.  Tail positions (last body form, if
// branches, macro expansions) do not keep a K-frame, but the canonical depth still increases.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "culi_internal.h"

namespace culi {

constexpr uint32_t STACK_ENV = 0x80000000u;   // env reference into the thread's V-stack

// Resident 128-thread eval blocks per SM (the register budget of __launch_bounds__) and so the default
// number of stack slots (SM count x 128 x this).  The machine is latency-bound: more warps per scheduler
// hide more of each warp's dependent-instruction latency.
// The splitting / nesting kernels (C2, C5, C0) run 9 (56 registers), the others 8 (64 registers):
// measured per kernel (tools/ab.sh, session 2): split 8 -> 9 blocks C2 62.0 -> 60.5 ms, C5 126.5 -> 123.8 ms;
// voting (C4) 0.47 -> 0.50 ms and fan-out (C3) 0.165 -> 0.170 ms at 9, so those stay at 8; 10 is worse
// everywhere.  Stack slots are sized for the larger count.
#ifndef CULI_SPLIT_BLOCKS_PER_SM
#define CULI_SPLIT_BLOCKS_PER_SM 9
#endif
#ifndef CULI_BLOCKS_PER_SM
#define CULI_BLOCKS_PER_SM 8
#endif

// Serve the persistent code segment from shared memory (see culi_machine.cuh ldnode); off by default.
#ifndef CULI_STAGE_CODE
#define CULI_STAGE_CODE 0
#endif

struct DevHeap {
  TagArr tag;                  // views of the node array (struct Node, culi_internal.h): tag.p == word.p
  WordArr word;
  unsigned long long* top;     // bump pointer (node index)
  uint64_t cap;                // node capacity
  uint8_t* gtag;               // global frame: direct-indexed by symbol id (identity hash)
  uint64_t* gword;
  uint32_t gcap;
  const char* strs;            // string bytes (offsets in STR words)
};

struct EvalArgs {
  DevHeap H;
  uint4* kst;                  // K-stack, level-major: kst[level * nslots + slot]
  uint4* vst;                  // V-stack, level-major
  uint32_t nslots;
  uint32_t stride;             // nslots * sizeof(uint4): byte distance between stack levels
  uint32_t kcap;               // K-stack entries per slot
  uint32_t vcap;               // V-stack entries per slot
  const uint32_t* roots;       // heap index of each form's datum
  const uint32_t* perm;        // optional evaluation order (binned dispatch), may be null
  uint32_t nforms;
  uint32_t* next;              // work counter (forms handed out so far)
  uint8_t* rtag;               // results, indexed by form
  uint8_t* rerr;
  uint64_t* rsteps;
  uint64_t* rword;
  uint32_t max_depth;
  uint64_t fuel;
  int define_mode;
  uint32_t mut;                // setq may run: every frame lives in the heap from creation
  uint32_t pmark;              // heap nodes below this index are persistent (read-only for a batch's setq)
  int* flags;                  // [0] heap/stack exhausted, [1] define: index of failing form + 1, [2] its err
  uint32_t voting;             // warp opcode voting on/off
  uint32_t fanout;             // top-level ||| forms fan out over threads (batch eval kernel only)
  struct FanDesc* desc;        // fan-out descriptors (device)
  uint32_t* npend;             // number of descriptors written
  uint32_t maxdesc;
  uint32_t* fallback;          // forms to re-evaluate sequentially (fan-out could not decide them)
  uint32_t* nfallback;
  uint4* payload;              // export tokens (flat ||| results are written by the fan-out stage)
  unsigned long long* pcount;
  unsigned long long pcap;
  const uint32_t* wide;        // per form: argument count of a wide top-level form, else 0 (host scan)
  uint32_t lanes;              // plain kernel: forms per warp (lanes >= this stay idle; 32 = all)
  uint32_t nest;               // nested ||| suspend + help, batch eval kernel only
  struct NestDesc* ndesc;
  uint32_t* nnest;
  uint32_t maxnest;
  uint4* kst2;                 // secondary stacks (elements run by a thread whose own form is suspended)
  uint4* vst2;
  uint32_t* finished;          // forms completed (threads without forms help until all are done)
  uint32_t code_lo, code_n;    // node range staged in shared memory (persistent code segment)
  uint32_t gst;                // global-frame entries staged in shared memory
  uint32_t split;              // argument splitting: idle warps evaluate pending arguments of busy ones
  uint32_t split_poll;         // closure calls between two polls of the idle-warp counter
  uint32_t split_first;        // closure calls before an evaluation's first poll (split the top of the tree early)
  uint32_t split_sleep;        // longest back-off (ns) of an idle warp waiting for its ticket's group
  uint32_t steal_gate;         // idle lanes steal only when their whole warp is idle
  struct SplitGroup* groups;   // SPLIT_GPW group slots per warp of the grid
  unsigned long long* gqueue;  // ring of published groups: ticket << 32 | (group + 1), gqcap entries
  uint32_t gqcap;              // power of two
  struct SplitCtl* sctl;       // queue counters, idle-warp tokens, statistics, bounded-wait diagnostics
  unsigned long long wait_ns;  // longest wait for another warp (join, queue entry, nested |||) before giving up
};

// One top-level (||| n f l1 .. lm) form whose arguments have been evaluated.
constexpr uint32_t FANOUT_MAXM = 6;
constexpr uint8_t E_PENDING = 0xfe;          // internal: record filled in by the fan-out finalizer
// FAN_PAR: (||| n f l1..lm) elements.  Wide forms (>= WIDE_MIN arguments, K12 "per warp for wide forms"):
// FAN_DATA (h a1..an) with h not applicable -> list (h v1..vn); FAN_LIST (list a1..an); FAN_FOLD (+ or *
// a1..an, op in m).  For wide kinds element i evaluates argument i (depth 2); heads[0] = first arg cell.
enum FanKind : uint32_t { FAN_PAR = 0, FAN_DATA = 1, FAN_LIST = 2, FAN_FOLD = 3 };
constexpr uint32_t WIDE_MIN = 64;
static_assert(WIDE_MIN == WIDE_LEN_MIN, "readers mark lists of the size the machine suspends on");
struct FanDesc {
  uint32_t form, n, m, spine;                // n: result cells; spine: 2n nodes (n cells, then n boxes)
  uint32_t kind, nelem;                      // FanKind; elements to evaluate
  uint32_t ftag, depth;
  uint64_t fword;
  uint64_t steps0;                           // canonical steps before the first element
  uint64_t top;                              // heap top when the descriptor was written
  uint32_t heads[FANOUT_MAXM];               // first cell of each list
  unsigned long long total;                  // sum of element steps (atomic)
  uint32_t bad;                              // bit 0: non-contiguous list, bit 1: an element errored
  uint32_t nonflat;                          // some element value is a cons (export walks it)
  unsigned long long flat_off;               // payload offset of a flat result list
};
constexpr uint8_t K_FLATREC = 12;

// A nested (||| n f l1..lm) whose evaluation is suspended until its elements are applied (§8(f)1): the
// owner thread saved {sp, vtop, steps}; any thread claims elements (next), applies f with the fuel left
// and adds their steps; when done == n the owner resumes at RET with the result spine.
constexpr uint32_t NEST_MIN = 32;
constexpr uint8_t E_SUSPEND = 0xfc;
// Warp voting (north_star "ballot for branch voting"): a lane group that diverged yields
// at a return; the kernel re-forms groups by (stack height, continuation kind) and resumes the deepest.
constexpr uint8_t E_YIELD = 0xfb;
// NEST_WIDE: a wide list — a data list or (list a1..an) with at least WIDE_MIN elements to evaluate —
// reached below the top level suspends the same way (kind NEST_EVAL): element i is the expression in
// cell heads[0] + i, evaluated in the heap environment env at depth+1; its value goes to spine cell
// off + i of the ncells-cell result spine (cell 0 of a data list holds the head value already).
enum NestKind : uint32_t { NEST_APPLY = 0, NEST_EVAL = 1 };
// The claim counter and the completion counters sit in lines of their own: every idle thread of the grid
// polls `ready`/`next` while the element threads update `done`/`total`.
struct alignas(128) NestDesc {
  uint32_t form, n, m, spine;
  uint32_t ftag, depth;
  uint64_t fword;
  uint64_t steps0;
  uint64_t top;
  uint32_t heads[FANOUT_MAXM];
  uint32_t sp, vtop;
  uint32_t kind, env, off, ncells;            // NEST_EVAL only (kind NEST_APPLY: 0)
  uint32_t ready;                             // fields published, elements claimable
  alignas(128) uint32_t next;                 // elements claimed
  alignas(128) unsigned long long total;      // sum of element steps
  uint32_t done, bad;
};

// Argument splitting.  When idle warps wait for work, the lanes of a busy warp that poll
// together turn the lowest pending argument of their K-stacks (the biggest unevaluated chunk: the next
// argument of the outermost KF_ARGS frame) into tasks, one group per poll, published with one ticket; an
// idle warp holding that ticket claims the whole group and its lanes evaluate the tasks on their own
// stacks.  Arguments are pure (no mutation inside a batch, c.3/c.13 #25), so only steps, the first error
// and fuel need care: each owner lane adds its task's steps at the join and decides errors/fuel exactly
// (c.4, c.10).  A group is claimed or taken back as a whole, so the owner lanes of a converged warp stay
// converged.  No warp-wide barrier takes part (round 1 deadlocked on one): the idle
// warps' rounds use a shared-memory counter, and the only warp intrinsics are a ballot and shuffles over
// __activemask() with no other collective in between.
struct SplitTask {
  uint32_t expr, env, depth, pad;      // argument node, heap env, depth of its evaluation
  unsigned long long budget;           // fuel left at the fork
  unsigned long long rw, rsteps;       // result word, steps
  uint32_t rt, rerr, done, pad2;
  uint32_t pad3[2];
};
static_assert(sizeof(SplitTask) == 64, "one task per 64-byte line");
struct SplitGroup {
  uint32_t state;                      // SPLIT_OPEN / SPLIT_CLAIMED / SPLIT_TAKEN
  uint32_t remaining;                  // owner lanes that have not joined yet (0: the slot is free again)
  uint32_t mask;                       // lanes with a task
  uint32_t form;
  uint32_t claimer;                    // global warp id of the thief (diagnostics)
  uint32_t pad[11];
  SplitTask t[32];
};
constexpr uint32_t SPLIT_GPW = 8;      // group slots per warp (outstanding polls of one warp)
constexpr uint32_t SPLIT_OPEN = 0, SPLIT_CLAIMED = 1, SPLIT_TAKEN = 2;
// Ticket queue (a FAA queue): an idle warp takes ticket h = head++ and waits for the entry stamped h; busy
// warps publish while head > tail (an idle warp waits) at ticket q = tail++.  Counters live across
// launches and tickets are never reused, so an entry left by an earlier launch (or lap of the ring) never
// matches; the reset kernel sets head = tail = max.  Outstanding tickets <= warps < ring capacity.
struct SplitCtl {
  unsigned long long tail;             // tickets handed out to publishers (monotonic)
  unsigned long long head;             // tickets handed out to idle lanes (monotonic)
  uint32_t published;                  // groups published in this launch (statistics)
  uint32_t timeouts;                   // bounded waits that gave up in this launch (0 in a healthy run)
  uint32_t diag[9];                    // the first one: kind, group, lane, form, state, mask, remaining, done, claimer
  uint32_t claimed;                    // groups an idle warp claimed (the rest were taken back by their owners)
  uint32_t stat[4];                    // statistics: thief rounds, rounds with < 32 lanes present, -, -
  unsigned long long t0;               // globaltimer at the launch's reset (debug watchdog, CULI_WATCHDOG builds)
  uint32_t wd[8];                      // debug watchdog: count, form, steps lo, sp, depth, root, thief, finished
};
constexpr uint32_t WAIT_JOIN = 1, WAIT_QUEUE = 2, WAIT_NEST = 3;
#ifndef CULI_WATCHDOG
#define CULI_WATCHDOG 0            // debug builds: forms running past CULI_WATCHDOG ms fail and are recorded
#endif

struct ExportArgs {
  TagArr tag;
  WordArr word;
  uint8_t* rtag;
  uint64_t* rword;
  uint32_t nforms;
  uint4* vst;                  // DFS stack (the eval V-stack, reused)
  uint32_t nslots, vcap;
  uint4* payload;              // tokens {word.lo, word.hi, tag, 0}
  unsigned long long* pcount;
  unsigned long long pcap;
  int* flags;                  // [3] payload overflow, [4] export stack overflow
  const uint32_t* list;        // optional: export only these forms
  uint32_t nlist;
};

// host-side launchers (culi_kernels.cu, culi_dispatch.cu)
cudaError_t launch_relocate(cudaStream_t s, const uint8_t* stag, const uint64_t* sword, Node* nodes, uint64_t base,
                            uint64_t n, uint32_t str_base, uint32_t* roots, uint32_t nroots, int sms);
cudaError_t launch_eval(cudaStream_t s, const EvalArgs& A, uint32_t blocks);
cudaError_t launch_lenmark(cudaStream_t s, Node* nodes, uint64_t base, const uint32_t* pairs, uint32_t npairs);
cudaError_t launch_define(cudaStream_t s, const EvalArgs& A);
cudaError_t launch_export(cudaStream_t s, const ExportArgs& X, uint32_t blocks);
cudaError_t launch_reset(cudaStream_t s, unsigned long long* top, unsigned long long top_value,
                         uint32_t* next, unsigned long long* pcount, int* flags, uint32_t* npend,
                         uint32_t* nfallback, uint32_t* nnest, struct SplitCtl* sctl);
cudaError_t launch_fanout(cudaStream_t s, const EvalArgs& A, uint32_t blocks);
cudaError_t launch_nest_clear(cudaStream_t s, struct NestDesc* d, uint32_t n);
cudaError_t launch_flat_export(cudaStream_t s, const EvalArgs& A, uint32_t blocks);
cudaError_t launch_dispatch(cudaStream_t s, const DevHeap& H, const uint32_t* roots, uint32_t nforms,
                            uint32_t* keys, uint32_t* keys_alt, uint32_t* perm, uint32_t* perm_alt,
                            void* temp, size_t temp_bytes, uint32_t** perm_out, int sms, uint32_t size_first);
size_t dispatch_temp_bytes(uint32_t nforms);
uint32_t dispatch_launches(uint32_t nforms);   // kernels launch_dispatch issues (an estimate: the graph path counts them)
// Batches of at most this many forms in which no closure can exist (no lambda / defun) are evaluated in
// input order: with <= 128 warps (fewer than the 148 SMs) the eval time is the slowest warp's either way,
// and the binning permutation scatters the warps' node loads.  Measured on C1 (1,024 forms): dispatch
// 35 us + eval 51 us binned, eval 42 us not.  Batches with closures stay binned: recursive forms of equal
// shape and argument then share warps (converged lanes), which pays for the sort.
constexpr uint32_t BIN_MIN_FORMS = 4097;

struct V {
  uint32_t t;
  uint64_t w;
};

// The halves of a node word are 32-bit node indices.  The empty asm makes each half an opaque 32-bit
// value, so `base + index` compiles to one IMAD.WIDE.U32 instead of 64-bit shift/mask arithmetic on the
// whole word (measured: 6 instructions per node address otherwise).
#ifndef CULI_OPAQUE_HALVES
#define CULI_OPAQUE_HALVES 1
#endif
__device__ __forceinline__ uint32_t lo32(uint64_t w) {
  uint32_t x = (uint32_t)w;
#if CULI_OPAQUE_HALVES
  asm("" : "+r"(x));
#endif
  return x;
}
__device__ __forceinline__ uint32_t hi32(uint64_t w) {
  uint32_t x = (uint32_t)(w >> 32);
#if CULI_OPAQUE_HALVES
  asm("" : "+r"(x));
#endif
  return x;
}
__device__ __forceinline__ bool is_ref(uint32_t k) {
  return k == K_CONS || k == K_STR || k == K_CLOSURE || k == K_MACRO;
}
__device__ __forceinline__ V mkv(uint32_t t, uint64_t w) { V v; v.t = t; v.w = w; return v; }

}  // namespace culi
