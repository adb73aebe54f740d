// ptxas contraction probe: mul.rn.f32x2 feeding add.rn.f32x2 becomes FFMA2 even with --fmad=false
// (kernels using mul2 directly); an fma.rn.f32x2 with a run-time -0.0 addend keeps FMUL-then-FADD2
// rounding (kC below).  Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 --fmad=false -cubin
// contract.cu && cuobjdump -sass contract.cubin | grep -E "FFMA|FMUL|FADD"
typedef unsigned long long u64;
__device__ __forceinline__ u64 add2(u64 a, u64 b) { u64 d; asm("add.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b)); return d; }
__device__ __forceinline__ u64 mulz(u64 a, u64 b, u64 z) { u64 d; asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(a), "l"(b), "l"(z)); return d; }
__global__ void kC(u64* a, const u64* b, u64 k0, u64 k1, u64 z){ int i = threadIdx.x; u64 s = add2(add2(a[i], b[i]), a[i+1]); a[i] = add2(mulz(k0, a[i+2], z), mulz(k1, s, z)); }
