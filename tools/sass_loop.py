"""Instruction mix of the hottest loop of one kernel in a cuobjdump -sass listing.

Usage: python tools/sass_loop.py <sass file> <function-name substring> [--all-loops]
Finds backward branches (loops), picks the one whose body holds the most LDS, and prints the
per-opcode count and the per-pipe totals (ALU: LOP3/PRMT/ISETP/SEL/IADD3/SHF/...; FMA: IMAD*;
LSU: LDS/STS/LDG/...).  Static counts: a body executed once per loop iteration.
"""
import re
import sys

ALU = ("LOP3", "PRMT", "ISETP", "SEL", "IADD3", "SHF", "LEA", "PLOP3", "FMNMX", "IMNMX",
       "POPC", "FLO", "BMSK", "SGXT", "LOP", "MOV", "VIMNMX", "R2P", "P2R", "ISCADD", "FSETP")
FMA = ("IMAD", "FFMA", "FMUL", "FADD", "HFMA2", "VIADD")   # VIADD: fmaheavy (tools/pipe_probe.cu)
LSU = ("LDS", "STS", "LDG", "STG", "LD", "ST", "LDSM", "ATOMS", "SHFL", "LDC")


def main():
    path, fn = sys.argv[1], sys.argv[2]
    text = open(path).read().split("\n")
    start = next(i for i, l in enumerate(text) if "Function :" in l and fn in l)
    end = next((i for i in range(start + 1, len(text)) if "Function :" in text[i]), len(text))
    ins = []
    for l in text[start:end]:
        m = re.match(r"\s*/\*([0-9a-f]{4,})\*/\s+(.*?);", l)
        if m:
            ins.append((int(m.group(1), 16), m.group(2).strip()))
    addr = {a: k for k, (a, _) in enumerate(ins)}
    loops = []
    for k, (a, s) in enumerate(ins):
        m = re.search(r"BRA[^0-9]*0x([0-9a-f]+)", s)
        if m:
            t = int(m.group(1), 16)
            if t <= a and t in addr:
                body = ins[addr[t]:k + 1]
                nlds = sum(1 for _, x in body if re.search(r"\bLDS", x))
                loops.append((nlds, addr[t], k))
    loops.sort(reverse=True)
    for nlds, s, e in (loops if "--all-loops" in sys.argv else loops[:1]):
        ops, pipes = {}, {"alu": 0, "fma": 0, "lsu": 0, "other": 0}
        for _, x in ins[s:e + 1]:
            x = re.sub(r"^@!?U?P\w+\s+", "", x)
            op = x.split()[0]
            base = op.split(".")[0]
            ops[op] = ops.get(op, 0) + 1
            p = "alu" if base in ALU else "fma" if base in FMA else "lsu" if base in LSU else "other"
            pipes[p] += 1
        print(f"loop {hex(ins[s][0])}-{hex(ins[e][0])}: {e - s + 1} instructions, {nlds} LDS")
        print("  pipes:", pipes)
        print("  ops:", sorted(ops.items(), key=lambda t: -t[1]))


if __name__ == "__main__":
    main()
