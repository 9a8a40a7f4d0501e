// Mandelbrot customizing function for the Map skeleton (§IV-A,
// P:L379-397, eq. (5): z_{i+1} = z_i^2 + c, z_0 = 0).  The element is the
// pixel's position c; the result is the number of
// updates made while |z| <= 2, at most `cap` (reading R4).
// Compiled with FMA contraction off so it matches the oracle bit for bit.
struct Pos { float re, im; };
int mandelbrot(Pos c, int cap) {
    float x = 0.0f, y = 0.0f;
    int n = 0;
    while (n < cap && x * x + y * y <= 4.0f) {
        float xt = (x * x - y * y) + c.re;
        y = (2.0f * x) * y + c.im;
        x = xt;
        ++n;
    }
    return n;
}
