// k1_inst.cu — the hot kernel's template instances, one state mode per object file.
//
// _build.py compiles this file once per SHRED_INST value (in parallel) and links the objects
// with shred.cu:  SHRED_INST = MODE_K63 / MODE_K40 / MODE_K32 / MODE_K32B instantiates
// k1_bulk<MODE, Cfg, ceil(w/16) (0: w > 64), marker kind, funnel> for that mode, and
// SHRED_INST = 0 the dispatchers pick_k1 / pick_k1_small plus the small-input shapes.
#define SHRED_K1_ONLY
#include <type_traits>

#include "kernels.cuh"

#ifndef SHRED_INST
#error "compile k1_inst.cu with -DSHRED_INST=<0 | state mode>"
#endif

namespace shred {

template <int MODE> K1Fn pick_mode(int wch, int mk, bool fn);

#if SHRED_INST != 0
template <int MODE, class C, int MK>
static K1Fn pick_w(int wch, bool fn) {
    switch (wch * 2 + (fn ? 1 : 0)) {           // fn: w not a multiple of 16 (funnel-shifted pops)
        case 0: return k1_bulk<MODE, C, 0, MK, false>;   // wch 0: long windows (w > 64, pops by TMA)
        case 1: return k1_bulk<MODE, C, 0, MK, true>;
        case 2: return k1_bulk<MODE, C, 1, MK, false>;
        case 3: return k1_bulk<MODE, C, 1, MK, true>;
        case 4: return k1_bulk<MODE, C, 2, MK, false>;
        case 5: return k1_bulk<MODE, C, 2, MK, true>;
        case 6: return k1_bulk<MODE, C, 3, MK, false>;
        case 7: return k1_bulk<MODE, C, 3, MK, true>;
        case 8: return k1_bulk<MODE, C, 4, MK, false>;
        case 9: return k1_bulk<MODE, C, 4, MK, true>;
        default: return nullptr;
    }
}
template <int MODE>
K1Fn pick_mode(int wch, int mk, bool fn) {
    using C = typename std::conditional<MODE == MODE_K63 || MODE == MODE_K40 || MODE == MODE_K63T, CfgK63,
                                        CfgK32>::type;
    constexpr bool TP = MODE == MODE_K32T || MODE == MODE_K63T;
    if (TP && mk != MK_EQ && mk != MK_LE) return nullptr;   // other kinds: the table modes
    switch (mk) {
        case MK_EQ: return pick_w<MODE, C, MK_EQ>(wch, fn);
        case MK_LE: return pick_w<MODE, C, MK_LE>(wch, fn);
        case MK_DIV: return TP ? nullptr : pick_w<MODE, C, MK_DIV>(wch, fn);
        case MK_REM: return TP ? nullptr : pick_w<MODE, C, MK_REM>(wch, fn);
        default: return nullptr;
    }
}
template K1Fn pick_mode<SHRED_INST>(int, int, bool);
#else
// The instance for (u64 state: deg 41..63 | deg 33..40; u32 state with a whole-byte top byte |
// u32 state; ceil(w/16), marker kind, w % 16 != 0).
// tprod: P = x^k + Q with Q's terms >= 8 apart, below k - 7 (deg <= 32: MODE_K32T) or below 25
// (deg 41..63: MODE_K63T), '==' and '<=' with D = 2^m; otherwise the table modes.
K1Fn pick_k1(int k, bool byteidx, int wch, int mk, bool fn, bool tprod) {
    if (k >= 41) {
        if (tprod) {
            if (K1Fn f = pick_mode<MODE_K63T>(wch, mk, fn)) return f;
        }
        return pick_mode<MODE_K63>(wch, mk, fn);
    }
    if (k >= 33) return pick_mode<MODE_K40>(wch, mk, fn);
    if (tprod) {
        if (K1Fn f = pick_mode<MODE_K32T>(wch, mk, fn)) return f;
    }
    return byteidx ? pick_mode<MODE_K32B>(wch, mk, fn) : pick_mode<MODE_K32>(wch, mk, fn);
}
// The small-input shape (CfgSmall) exists for the paper's window with the equality marker.
K1Fn pick_k1_small(int k, bool byteidx, int wch, int mk, bool fn, bool tprod) {
    if (wch != 3 || mk != MK_EQ || fn || (k >= 33 && k <= 40)) return nullptr;
    if (k >= 41) return tprod ? k1_bulk<MODE_K63T, CfgSmall, 3, MK_EQ> : k1_bulk<MODE_K63, CfgSmall, 3, MK_EQ>;
    if (tprod) return k1_bulk<MODE_K32T, CfgSmall, 3, MK_EQ>;
    return byteidx ? k1_bulk<MODE_K32B, CfgSmall, 3, MK_EQ> : k1_bulk<MODE_K32, CfgSmall, 3, MK_EQ>;
}
#endif

}  // namespace shred
